"""B200-native hot path of arXiv:1011.0024 (multi-GPU QUDA): even-odd Wilson-clover Dslash,
T-direction ghost-zone exchange, mixed-precision reliable-update BiCGstab.

The product is the C-ABI library libqudax.so (include/qudax.h, sources in csrc/);
`qudax` is its thin Python binding.  Build with `python -m paper_1011_0024_b200.build`.
"""
from . import qudax  # noqa: F401

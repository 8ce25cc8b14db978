"""Debug helper: where does a loopback split-dimension Dslash differ from the unsplit one?"""
import sys
import numpy as np
sys.path.insert(0, ".")
import qgen
from paper_1011_0024_b200 import qudax

dims = (8, 4, 6, 8)
U = qgen.gauge(dims, 1221)
psi = qgen.spinor(dims, 1222)
for prec in (2, 4):
    for mask in (1, 2, 4, 6, 8, 14):
        ref = qudax.Context(dims)
        loop = qudax.Context(dims, comm=qudax.COMM_NCCL, nccl_id=qudax.nccl_unique_id(), split_mask=mask)
        outs = []
        for c in (ref, loop):
            c.gauge_load(U, 0.12, 1.0, prec=prec, recon=12)
            fi, fo = c.new_field(prec), c.new_field(prec)
            c.spinor_load(fi, prec, 1, psi)
            c.dslash(fo, fi, prec, 0, dagger=False, kind=0)
            c.sync()
            outs.append(c.spinor_store(fo, prec, 0))
        d = np.abs(outs[0] - outs[1]).max(axis=(4, 5))
        bad = np.argwhere(d > 0)
        print(f"prec {prec} mask {mask:04b}: {len(bad)} sites differ, max {d.max():.3e}; first (t,z,y,x): {bad[:6].tolist()}")
        ref.close(); loop.close()

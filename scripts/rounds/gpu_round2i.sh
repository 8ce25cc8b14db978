#!/bin/bash
# Round-2 pass I: A/B of the late T x in the fused-(<t,s>,|t|^2) xpay kernel (default) vs early.
TAG=${1:-r02i}
OUT=gpurun_out/$TAG
mkdir -p $OUT
for r in 1 2; do
  for L in default earlyxdot; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    timeout 300 python bench.py --steps 20 --warmup 3 --no-extra --no-cpu-baseline --breakdown > $OUT/ab_$L.$r.json 2> $OUT/ab_$L.$r.err
  done
done
unset QUDAX_LIB
timeout 600 python -m pytest tests/gpu/test_solver.py tests/gpu/test_fullsize.py -q -p no:cacheprovider > $OUT/pytest.log 2>&1; echo rc=$? >> $OUT/pytest.log
ls -la $OUT

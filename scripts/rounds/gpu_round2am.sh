#!/bin/bash
# Round-2 pass AM: fp32/fp64 xpay output stored after the CTA published its reduction partial
# (head, QX_RED_STORE_LATE 1) vs before (lib_var/early), alternating; solver / multi-RHS tests.
TAG=${1:-r02am}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 900 python -m pytest tests/gpu/test_solver.py tests/gpu/test_multirhs.py tests/gpu/test_halo.py -x -q > $OUT/pytest.log 2>&1; echo rc=$? >> $OUT/pytest.log
for r in 1 2 3; do
  for L in default early; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    timeout 300 python bench.py --steps 20 --warmup 3 --no-extra --no-cpu-baseline --breakdown > $OUT/step_$L.$r.json 2> $OUT/step_$L.$r.err
  done
done
unset QUDAX_LIB
ls -la $OUT

#!/bin/bash
# Round-2 pass Y: packed FFMA2 site partials of the fused reductions (head) vs 6 -> 7 CTAs per SM
# (lib_var/minb7, built before the partials change); solver / multi-RHS tests.
TAG=${1:-r02y}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 900 python -m pytest tests/gpu/test_solver.py tests/gpu/test_multirhs.py -x -q > $OUT/pytest.log 2>&1; echo rc=$? >> $OUT/pytest.log
for r in 1 2; do
  for L in default minb7; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    timeout 600 python scripts/bench_dslash.py --cases f32-12,h-12 --reps 30 --nrhs 8 --tag $L > $OUT/$L.$r.jsonl 2>&1
    timeout 300 python bench.py --steps 20 --warmup 3 --no-extra --no-cpu-baseline --breakdown > $OUT/step_$L.$r.json 2> $OUT/step_$L.$r.err
  done
done
unset QUDAX_LIB
K='regex:dslash_kernel<\(int\)4, \(int\)12, \(bool\)0, \(int\)2'
timeout 900 ncu --set full --clock-control none --import-source on --kernel-name-base demangled \
    -k "$K" --launch-skip 10 -c 2 -o $OUT/xpay_solver \
    python bench.py --steps 1 --warmup 1 --iters 20 --no-extra --no-cpu-baseline > $OUT/ncu_xpay.log 2>&1
ls -la $OUT

#!/bin/bash
# Round-2 pass W: evidence of the head — bench line (full), ncu launch list of the step, ncu
# --set full of the solver's fp32-12 Dslash launches, standalone fp32-12 / half-12
# clover-inverse kernels with source counters; multi-RHS / halo GPU tests (half cross product).
TAG=${1:-r02w}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 900 python -m pytest tests/gpu/test_multirhs.py tests/gpu/test_dslash_parity.py -x -q > $OUT/pytest_part.log 2>&1; echo rc=$? >> $OUT/pytest_part.log
bash scripts/profile_round.sh $TAG
K='regex:dslash_kernel<\(int\)4, \(int\)12, \(bool\)0, \(int\)1'
timeout 600 ncu --set full --clock-control none --import-source on --kernel-name-base demangled \
  -k "$K" --launch-skip 5 --launch-count 1 -o $OUT/ci_f32 python scripts/bench_dslash.py --cases f32-12 --reps 3 > $OUT/ncu_ci_f32.log 2>&1
K='regex:dslash_kernel<\(int\)2, \(int\)12, \(bool\)0, \(int\)1'
timeout 600 ncu --set full --clock-control none --import-source on --kernel-name-base demangled \
  -k "$K" --launch-skip 5 --launch-count 1 -o $OUT/ci_h12 python scripts/bench_dslash.py --cases h-12 --reps 3 > $OUT/ncu_ci_h12.log 2>&1
timeout 600 python scripts/bench_dslash.py --cases f32-12,h-12,f32-8,f32-18,h-18,h-8,f64-18,f64-12 --reps 30 --nrhs 4,8 > $OUT/bench_dslash.jsonl 2>&1
ls -la $OUT

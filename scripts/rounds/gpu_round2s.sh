#!/bin/bash
# Round-2 pass S: lane-interleaved multi-RHS kernel (dslash_li.cuh) — correctness, A/B against
# the two-RHS-per-thread and one-RHS-per-CTA launches, ncu; ncu of the round-1 vs head
# standalone fp32-12 clover-inverse kernel.
TAG=${1:-r02s}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 900 python -m pytest tests/gpu/test_multirhs.py tests/gpu/test_solver.py -k "multi or batched" -x -q > $OUT/pytest_mr.log 2>&1; echo rc=$? >> $OUT/pytest_mr.log
for r in 1 2; do
  for F in 0 32 8; do
    timeout 600 python scripts/bench_dslash.py --cases f32-12,h-12,f64-18 --reps 10 --nrhs 2,4,6,8 --flags $F --tag flags$F > $OUT/mr_flags$F.$r.jsonl 2>&1
  done
done
K='regex:dslash_(li_)?kernel<\(int\)4, \(int\)12, \(bool\)0, \(int\)1'
timeout 600 ncu --set full --clock-control none --import-source on --kernel-name-base demangled \
  -k "$K" --launch-skip 5 --launch-count 1 -o $OUT/ci_head python scripts/bench_dslash.py --cases f32-12 --reps 3 > $OUT/ncu_ci_head.log 2>&1
(cd old_r01 && timeout 600 ncu --set full --clock-control none --import-source on --kernel-name-base demangled \
  -k "$K" --launch-skip 5 --launch-count 1 -o ../$OUT/ci_old python scripts/bench_dslash.py --cases f32-12 --reps 3 > ../$OUT/ncu_ci_old.log 2>&1)
timeout 600 ncu --set full --clock-control none --import-source on --kernel-name-base demangled \
  -k "regex:dslash_li_kernel<\(int\)4, \(int\)12, \(bool\)0, \(int\)2" --launch-skip 2 --launch-count 1 -o $OUT/li_f12_xpay \
  python scripts/bench_dslash.py --cases f32-12 --reps 3 --nrhs 8 > $OUT/ncu_li.log 2>&1
for f in ci_head ci_old li_f12_xpay; do ncu -i $OUT/$f.ncu-rep --page raw --csv > $OUT/${f}_raw.csv 2>/dev/null; done
ls -la $OUT

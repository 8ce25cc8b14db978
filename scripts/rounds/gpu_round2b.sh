#!/bin/bash
# Round-2 pass B: GPU tests (all, no -x), memcheck of the failing split-dims case, A/B of the
# pipelined hop schedule, ncu of the half-12 clover-inverse kernel, bench line.
TAG=${1:-r02b}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 1500 python -m pytest tests/gpu -q -rs > $OUT/pytest_gpu.log 2>&1; echo rc=$? >> $OUT/pytest_gpu.log
timeout 400 compute-sanitizer --tool memcheck --print-limit 20 python -m pytest tests/gpu/test_halo.py -x -q -k "split_dims_bitwise" > $OUT/memcheck_split.log 2>&1; echo rc=$? >> $OUT/memcheck_split.log
bash scripts/ab_dslash.sh $TAG "default nopipe pipe7 noclvpf" f32-12,h-12,h-18,f64-18
timeout 600 ncu --set full --clock-control none --import-source on --kernel-name-base demangled \
  -k "regex:dslash_kernel<\(int\)2, \(int\)12, \(bool\)0, \(int\)1" --launch-skip 5 --launch-count 1 -o $OUT/h12_inv \
  python scripts/bench_dslash.py --cases h-12 --reps 3 > $OUT/ncu_h12.log 2>&1
ncu -i $OUT/h12_inv.ncu-rep --page source --csv > $OUT/h12_inv_source.csv 2>/dev/null
ncu -i $OUT/h12_inv.ncu-rep --page details --csv > $OUT/h12_inv_details.csv 2>/dev/null
timeout 900 python bench.py > $OUT/bench.json 2> $OUT/bench.err
ls -la $OUT

#!/bin/bash
# Round-2 pass B: A/B of the software-pipelined hop schedule (default = half pipelined; nopipe;
# pipe7 = every precision pipelined), tests of the kernel-side allreduce (P2P mode), ncu of the
# half-12 clover-inverse kernel.
TAG=${1:-r02b}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 900 python -m pytest tests/gpu/test_halo.py tests/gpu/test_multirank.py tests/gpu/test_solver.py -x -q -rs > $OUT/pytest_p2p.log 2>&1; echo rc=$? >> $OUT/pytest_p2p.log
bash scripts/ab_dslash.sh $TAG "default nopipe pipe7" f32-12,h-12,h-18,f64-18
timeout 900 ncu --set full --clock-control none --import-source on --kernel-name-base demangled \
  -k "regex:dslash_kernel<\(int\)2, \(int\)12, \(bool\)0, \(int\)1" --launch-skip 5 --launch-count 1 -o $OUT/h12_inv \
  python scripts/bench_dslash.py --cases h-12 --reps 3 > $OUT/ncu_h12.log 2>&1
ncu -i $OUT/h12_inv.ncu-rep --page source --csv > $OUT/h12_inv_source.csv 2>/dev/null
ncu -i $OUT/h12_inv.ncu-rep --page details --csv > $OUT/h12_inv_details.csv 2>/dev/null
ls -la $OUT

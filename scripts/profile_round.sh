#!/bin/bash
# Round evidence on the GPU box: bench line, ncu launch list of a short bench, ncu --set full of
# the solver-launched fp32-12 Dslash kernels.  Outputs under gpurun_out/$TAG/ (summarise here
# with scripts/ncu_summary.py).
TAG=${1:-r01}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 600 python bench.py > $OUT/bench.json 2> $OUT/bench.err
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 2000 --csv --log-file $OUT/launches.csv \
    python bench.py --steps 2 --warmup 1 --iters 20 --no-extra --no-cpu-baseline > $OUT/launches_bench.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on --kernel-name-base demangled \
    -k "regex:dslash_kernel<\(int\)4, \(int\)12" --launch-skip 10 -c 2 -o $OUT/dslash_solver \
    python bench.py --steps 1 --warmup 1 --iters 20 --no-extra --no-cpu-baseline > $OUT/ncu_full.log 2>&1
ncu -i $OUT/dslash_solver.ncu-rep --page raw --csv > $OUT/dslash_solver_raw.csv
ncu -i $OUT/dslash_solver.ncu-rep --page details --csv > $OUT/dslash_solver_details.csv
xz -6 $OUT/dslash_solver.ncu-rep
ls -la $OUT

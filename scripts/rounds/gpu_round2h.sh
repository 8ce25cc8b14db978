#!/bin/bash
# Round-2 pass H: ncu launch list of a short bench, ncu --set full of the solver-launched fp32-12
# Dslash kernels, multi-RHS register-cap variants, strong-scaling N=1 line, reference arm.
TAG=${1:-r02h}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 3000 --csv --log-file $OUT/launches.csv \
    python bench.py --steps 2 --warmup 1 --iters 20 --no-extra --no-cpu-baseline > $OUT/launches_bench.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on --kernel-name-base demangled \
    -k "regex:dslash_kernel<\(int\)4, \(int\)12" --launch-skip 20 -c 4 -o $OUT/dslash_solver \
    python bench.py --steps 1 --warmup 1 --iters 20 --no-extra --no-cpu-baseline > $OUT/ncu_full.log 2>&1
ncu -i $OUT/dslash_solver.ncu-rep --page raw --csv > $OUT/dslash_solver_raw.csv 2>/dev/null
ncu -i $OUT/dslash_solver.ncu-rep --page details --csv > $OUT/dslash_solver_details.csv 2>/dev/null
for L in default mrminb5 mrminb3; do
  if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
  timeout 300 python scripts/bench_dslash.py --cases f32-12,h-12 --reps 20 --nrhs 8 --tag $L >> $OUT/mr.log 2>&1
done
unset QUDAX_LIB
timeout 600 python bench.py --scaling strong --no-extra --no-cpu-baseline > $OUT/bench_strong_n1.json 2> $OUT/bench_strong_n1.err
timeout 600 python bench.py --impl reference --steps 3 --warmup 1 > $OUT/bench_reference.json 2> $OUT/bench_reference.err
ls -la $OUT

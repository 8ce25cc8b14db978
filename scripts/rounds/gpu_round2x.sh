#!/bin/bash
# Round-2 pass X: graph condition set by a one-thread kernel (ncu-profilable body kernels); launch
# list of the step under ncu; 6 vs 7 CTAs per SM for the fp32 / half Dslash (lib_var/minb7).
TAG=${1:-r02x}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 900 python -m pytest tests/gpu/test_solver.py -x -q > $OUT/pytest_solver.log 2>&1; echo rc=$? >> $OUT/pytest_solver.log
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 3000 --csv --log-file $OUT/launches.csv \
    python bench.py --steps 2 --warmup 1 --iters 20 --no-extra --no-cpu-baseline > $OUT/launches_bench.log 2>&1
for r in 1 2; do
  for L in default minb7; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    timeout 600 python scripts/bench_dslash.py --cases f32-12,h-12 --reps 30 --nrhs 8 --tag $L > $OUT/$L.$r.jsonl 2>&1
  done
done
for L in default minb7; do
  if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
  timeout 300 python bench.py --steps 20 --warmup 3 --no-extra --no-cpu-baseline --breakdown > $OUT/step_$L.json 2> $OUT/step_$L.err
done
ls -la $OUT

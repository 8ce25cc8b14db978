#!/bin/bash
# Round-2 pass AJ: CTAs per SM of the eight-parameter-link Dslash (fp32 6 -> 5, half 7 -> 6;
# lib_var/r8a) vs the head, alternating.
TAG=${1:-r02aj}
OUT=gpurun_out/$TAG
mkdir -p $OUT
for r in 1 2; do
  for L in default r8a; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    timeout 600 python scripts/bench_dslash.py --cases f32-8,h-8 --reps 30 --tag $L > $OUT/$L.$r.jsonl 2>&1
  done
done
ls -la $OUT

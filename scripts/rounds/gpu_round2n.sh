#!/bin/bash
# Round-2 pass N: standalone Dslash, round-1 head vs round-2 head vs round-2 without the span
# instrumentation vs round-2 without span and halt gate (same box, alternating).
TAG=${1:-r02n}
OUT=gpurun_out/$TAG
mkdir -p $OUT
for r in 1 2; do
  (cd old_r01 && timeout 600 python scripts/bench_dslash.py --cases f32-12,f32-8,h-12,f64-18 --reps 30 --tag old > ../$OUT/old.$r.jsonl 2>&1)
  for L in default nohalt; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    timeout 600 python scripts/bench_dslash.py --cases f32-12,f32-8,h-12,f64-18 --reps 30 --tag $L > $OUT/$L.$r.jsonl 2>&1
  done
  unset QUDAX_LIB
done
ls -la $OUT

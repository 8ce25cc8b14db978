#!/bin/bash
# Round-2 pass P: which round-2 kernel change costs the standalone Dslash (variants compile one out).
TAG=${1:-r02p}
OUT=gpurun_out/$TAG
mkdir -p $OUT
for r in 1 2; do
  (cd old_r01 && timeout 600 python scripts/bench_dslash.py --cases f32-12,f32-8,h-12 --reps 30 --tag old > ../$OUT/old.$r.jsonl 2>&1)
  for L in default all4 nodar nospan; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    timeout 600 python scripts/bench_dslash.py --cases f32-12,f32-8,h-12 --reps 30 --tag $L > $OUT/$L.$r.jsonl 2>&1
  done
  unset QUDAX_LIB
done
ls -la $OUT

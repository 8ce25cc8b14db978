#!/bin/bash
# Round-2 pass AK: half recon-18 Dslash at 6 CTAs per SM (head) vs 7 (lib_var/h18m7), alternating.
TAG=${1:-r02ak}
OUT=gpurun_out/$TAG
mkdir -p $OUT
for r in 1 2; do
  for L in default h18m7; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    timeout 600 python scripts/bench_dslash.py --cases h-18,h-8,h-12 --reps 30 --tag $L > $OUT/$L.$r.jsonl 2>&1
  done
done
ls -la $OUT

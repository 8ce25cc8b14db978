#!/bin/bash
# Round-2 pass Q: roofline pass with per-launch events inside graph replay (default) vs eager
# launches while timing is on.
TAG=${1:-r02q}
OUT=gpurun_out/$TAG
mkdir -p $OUT
for r in 1 2; do
  for L in default eagertiming; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    timeout 300 python bench.py --steps 20 --warmup 3 --no-extra --no-cpu-baseline --breakdown > $OUT/ab_$L.$r.json 2> $OUT/ab_$L.$r.err
  done
done
unset QUDAX_LIB
ls -la $OUT

#!/bin/bash
# Round-2 pass K: solver-step A/B of the second Mhat kernel's reverse site order and of a 96-register
# (5 CTAs/SM) fp32 / half Dslash.
TAG=${1:-r02k}
OUT=gpurun_out/$TAG
mkdir -p $OUT
for r in 1 2; do
  for L in default norev minb5; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    timeout 300 python bench.py --steps 20 --warmup 3 --no-extra --no-cpu-baseline --breakdown > $OUT/ab_$L.$r.json 2> $OUT/ab_$L.$r.err
  done
done
unset QUDAX_LIB
ls -la $OUT

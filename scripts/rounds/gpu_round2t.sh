#!/bin/bash
# Round-2 pass T: which source change costs the head's standalone clover-inverse kernel its
# round-1 speed (register moves around FFMA2 operand pairs, r02s) — build variants, same box.
TAG=${1:-r02t}
OUT=gpurun_out/$TAG
mkdir -p $OUT
for r in 1 2; do
  (cd old_r01 && timeout 600 python scripts/bench_dslash.py --cases f32-12,h-12 --reps 30 --tag old > ../$OUT/old.$r.jsonl 2>&1)
  for L in default nohalt_nospan haltearly norpf; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    timeout 600 python scripts/bench_dslash.py --cases f32-12,h-12 --reps 30 --tag $L > $OUT/$L.$r.jsonl 2>&1
  done
  unset QUDAX_LIB
done
for L in default haltearly norpf; do
  if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
  timeout 300 python bench.py --steps 20 --warmup 3 --no-extra --no-cpu-baseline --breakdown > $OUT/step_$L.json 2> $OUT/step_$L.err
done
unset QUDAX_LIB
ls -la $OUT

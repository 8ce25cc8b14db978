#!/bin/bash
# Round-2 pass V: complex multiply-adds with the i-multiplication folded into FFMA2 operand
# modifiers (no (-1, 1) constant pair) — full GPU tests, Dslash table vs round 1, bench.
TAG=${1:-r02v}
OUT=gpurun_out/$TAG
mkdir -p $OUT
for r in 1 2; do
  (cd old_r01 && timeout 600 python scripts/bench_dslash.py --cases f32-12,h-12,f32-8,f64-18 --reps 30 --tag old > ../$OUT/old.$r.jsonl 2>&1)
  timeout 600 python scripts/bench_dslash.py --cases f32-12,h-12,f32-8,f64-18 --reps 30 --nrhs 8 --tag head > $OUT/head.$r.jsonl 2>&1
done
timeout 300 python bench.py --steps 20 --warmup 3 --no-extra --no-cpu-baseline --breakdown > $OUT/step.json 2> $OUT/step.err
timeout 1500 python -m pytest tests -m gpu -x -q > $OUT/pytest_gpu.log 2>&1; echo rc=$? >> $OUT/pytest_gpu.log
ls -la $OUT

#!/bin/bash
# Round-2 pass M: per-kind Dslash table, round-1 head (old_r01 worktree) vs round-2 head, same box.
TAG=${1:-r02m}
OUT=gpurun_out/$TAG
mkdir -p $OUT
for r in 1 2; do
  (cd old_r01 && timeout 600 python scripts/bench_dslash.py --cases f32-12,f32-8,h-12,h-8,f64-12 --reps 30 --tag old > ../$OUT/old.$r.jsonl 2>&1)
  timeout 600 python scripts/bench_dslash.py --cases f32-12,f32-8,h-12,h-8,f64-12 --reps 30 --tag new > $OUT/new.$r.jsonl 2>&1
done
ls -la $OUT

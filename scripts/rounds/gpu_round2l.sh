#!/bin/bash
# Round-2 pass L: per-kind Dslash table of the head build, wall time of the default bench.
TAG=${1:-r02l}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 900 python scripts/bench_dslash.py --cases f32-12,f32-18,f32-8,h-12,h-18,h-8,f64-18,f64-12 --reps 30 --nrhs 2,4,8 > $OUT/bench_dslash.jsonl 2> $OUT/bench_dslash.err
( time timeout 900 python bench.py > $OUT/bench.json 2> $OUT/bench.err ) 2> $OUT/bench_time.txt
ls -la $OUT

#!/bin/bash
# Round-2 pass U: solver batches as WHILE-node graphs (no in-kernel halt gate) — solver / multi-rank
# GPU tests, smoke, standalone Dslash table vs round 1, bench step.
TAG=${1:-r02u}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 900 python -m pytest tests/gpu/test_solver.py tests/gpu/test_multirank.py tests/gpu/test_halo.py -x -q > $OUT/pytest_solver.log 2>&1; echo rc=$? >> $OUT/pytest_solver.log
python -c "import __graft_entry__ as g; g.smoke()" > $OUT/smoke.log 2>&1; echo rc=$? >> $OUT/smoke.log
for r in 1 2; do
  (cd old_r01 && timeout 600 python scripts/bench_dslash.py --cases f32-12,h-12 --reps 30 --tag old > ../$OUT/old.$r.jsonl 2>&1)
  timeout 600 python scripts/bench_dslash.py --cases f32-12,h-12 --reps 30 --tag head > $OUT/head.$r.jsonl 2>&1
done
timeout 300 python bench.py --steps 20 --warmup 3 --no-extra --no-cpu-baseline --breakdown > $OUT/step.json 2> $OUT/step.err
ls -la $OUT

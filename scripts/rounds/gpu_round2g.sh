#!/bin/bash
# Round-2 pass G: full GPU tests, halo timeline (tail mode), sanitizers, bench line.
TAG=${1:-r02g}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 1500 python -m pytest tests/gpu -v -rs --timeout 300 -p no:cacheprovider > $OUT/pytest_gpu.log 2>&1; echo rc=$? >> $OUT/pytest_gpu.log
timeout 200 python scripts/halo_timeline.py > $OUT/halo_timeline.jsonl 2> $OUT/halo_timeline.err
timeout 200 python -c "import __graft_entry__ as g; g.smoke()" > $OUT/smoke.log 2>&1; echo rc=$? >> $OUT/smoke.log
timeout 600 python bench.py > $OUT/bench.json 2> $OUT/bench.err
for tool in memcheck racecheck synccheck; do
  timeout 600 compute-sanitizer --tool $tool --print-limit 50 python scripts/sanitize.py > $OUT/sanitize_$tool.log 2>&1
  echo rc=$? >> $OUT/sanitize_$tool.log
done
ls -la $OUT

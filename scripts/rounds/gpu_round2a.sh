#!/bin/bash
# Round-2 first GPU pass: full GPU test suite, smoke, compute-sanitizer, bench line.
TAG=${1:-r02a}
OUT=gpurun_out/$TAG
mkdir -p $OUT
nvidia-smi > $OUT/nvidia_smi.txt 2>&1
timeout 2400 python -m pytest tests -m gpu -x -q -rs > $OUT/pytest_gpu.log 2>&1; echo rc=$? >> $OUT/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > $OUT/smoke.log 2>&1; echo rc=$? >> $OUT/smoke.log
for tool in memcheck racecheck synccheck; do
  timeout 1200 compute-sanitizer --tool $tool --print-limit 50 python scripts/sanitize.py > $OUT/sanitize_$tool.log 2>&1
  echo rc=$? >> $OUT/sanitize_$tool.log
done
timeout 900 python bench.py > $OUT/bench.json 2> $OUT/bench.err
ls -la $OUT

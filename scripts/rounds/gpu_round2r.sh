#!/bin/bash
# Round-2 pass R (re-entry session): head evidence on a fresh box — GPU tests, bench line,
# and the roofline-pass A/B (per-launch events inside graph replay vs eager launches).
TAG=${1:-r02r}
OUT=gpurun_out/$TAG
mkdir -p $OUT
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm,power.limit --format=csv > $OUT/smi.csv
timeout 600 python bench.py > $OUT/bench.json 2> $OUT/bench.err
bash scripts/rounds/gpu_round2q.sh $TAG
timeout 1200 python -m pytest tests -m gpu -x -q > $OUT/pytest_gpu.log 2>&1; echo rc=$? >> $OUT/pytest_gpu.log
ls -la $OUT

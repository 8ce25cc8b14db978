#!/bin/bash
# Round-2 pass J: GPU tests, bench line, ncu launch list of an NCCL-loopback solve (NCCL kernels
# inside the replayed solver graphs), launch list of the bench step.
TAG=${1:-r02j}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 1500 python -m pytest tests/gpu -v -rs --timeout 300 -p no:cacheprovider > $OUT/pytest_gpu.log 2>&1; echo rc=$? >> $OUT/pytest_gpu.log
timeout 600 python bench.py > $OUT/bench.json 2> $OUT/bench.err
timeout 300 ncu --metrics gpu__time_duration.sum --clock-control none -c 5000 --csv --log-file $OUT/loopback_launches.csv \
    python scripts/loopback_solve.py > $OUT/loopback_solve.log 2>&1
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 3000 --csv --log-file $OUT/launches.csv \
    python bench.py --steps 2 --warmup 1 --iters 20 --no-extra --no-cpu-baseline > $OUT/launches_bench.log 2>&1
ls -la $OUT

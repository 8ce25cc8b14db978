#!/bin/bash
# Round-2 pass AF: split-path (halo loopback) cost table and the halo/interior overlap timeline
# on the head build.
TAG=${1:-r02af}
OUT=gpurun_out/$TAG
mkdir -p $OUT
for P in 4 2 8; do timeout 600 python scripts/bench_halo.py --prec $P > $OUT/halo_p$P.log 2>&1; done
timeout 300 python scripts/halo_timeline.py > $OUT/halo_timeline.jsonl 2> $OUT/halo_timeline.err
ls -la $OUT

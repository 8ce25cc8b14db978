#!/bin/bash
OUT=gpurun_out/r02f
mkdir -p $OUT
for v in nograph nograph_noov graph_noov graph poll1_graph; do
  echo "=== $v" >> $OUT/debug.log
  NCCL_DEBUG=WARN timeout 70 python scripts/debug_nccl_solve.py $v >> $OUT/debug.log 2>&1; echo "rc=$?" >> $OUT/debug.log
done

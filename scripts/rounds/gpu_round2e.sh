#!/bin/bash
# Round-2 pass E: A/B of the shared-memory staging of the fused-reduction operand (fp32 xpay),
# in-step breakdown for both, halo-overlap timeline, new GPU tests.
TAG=${1:-r02e}
OUT=gpurun_out/$TAG
mkdir -p $OUT
for t in "tests/gpu/test_halo.py::test_loopback_split_dims_solve" "tests/gpu/test_solver.py::test_loopback_nccl_solve_bitwise_with_allreduce_in_graph" "tests/gpu/test_solver.py::test_loopback_solve_matches_unsplit"; do
  timeout 180 python -m pytest "$t" -q -p no:cacheprovider >> $OUT/pytest_nccl.log 2>&1; echo "$t rc=$?" >> $OUT/pytest_nccl.log
done
for r in 1 2; do
  for L in default nostage; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    timeout 300 python bench.py --steps 20 --warmup 3 --no-extra --no-cpu-baseline --breakdown > $OUT/ab_$L.$r.json 2> $OUT/ab_$L.$r.err
  done
done
unset QUDAX_LIB
timeout 300 python scripts/halo_timeline.py > $OUT/halo_timeline.jsonl 2> $OUT/halo_timeline.err
timeout 1200 python -m pytest tests/gpu -v -rs --timeout 300 -p no:cacheprovider > $OUT/pytest_sel.log 2>&1; echo rc=$? >> $OUT/pytest_sel.log
ls -la $OUT

#!/bin/bash
# Round-2 pass AH: programmatic dependent launch for the solver iteration's kernels (head, QX_PDL 1)
# vs none (lib_var/nopdl), alternating; GPU tests of the solver / halo / multi-RHS / parity paths.
TAG=${1:-r02ah}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 1200 python -m pytest tests/gpu/test_solver.py tests/gpu/test_halo.py tests/gpu/test_multirhs.py tests/gpu/test_dslash_parity.py tests/gpu/test_multirank.py -x -q > $OUT/pytest.log 2>&1; echo rc=$? >> $OUT/pytest.log
for r in 1 2 3; do
  for L in default nopdl; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    timeout 300 python bench.py --steps 20 --warmup 3 --no-extra --no-cpu-baseline --breakdown > $OUT/step_$L.$r.json 2> $OUT/step_$L.$r.err
  done
done
unset QUDAX_LIB
timeout 900 python scripts/diag_batch_overhead.py > $OUT/batch_overhead.jsonl 2> $OUT/batch_overhead.err
ls -la $OUT

#!/bin/bash
# Round-2 pass AC: the xpay's x loaded with L1 evict-last priority when the (<t,s>, |t|^2)
# reduction re-reads it (head) vs plain read-only loads (lib_var/nokeep), alternating; tests.
TAG=${1:-r02ac}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 900 python -m pytest tests/gpu/test_solver.py tests/gpu/test_dslash_parity.py -x -q > $OUT/pytest.log 2>&1; echo rc=$? >> $OUT/pytest.log
for r in 1 2 3; do
  for L in default nokeep; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    timeout 300 python bench.py --steps 20 --warmup 3 --no-extra --no-cpu-baseline --breakdown > $OUT/step_$L.$r.json 2> $OUT/step_$L.$r.err
  done
done
unset QUDAX_LIB
ls -la $OUT

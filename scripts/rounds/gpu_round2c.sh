#!/bin/bash
# Round-2 pass C: GPU tests with per-test timeouts (find the hang of r02b), A/B of the solver-batch
# halt check (late = after the first hop's loads; early = kernel entry), bench line.
TAG=${1:-r02c}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 1800 python -m pytest tests/gpu -v -rs --timeout 240 -p no:cacheprovider > $OUT/pytest_gpu.log 2>&1; echo rc=$? >> $OUT/pytest_gpu.log
for r in 1 2; do
  for L in default haltearly; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    timeout 300 python bench.py --steps 10 --warmup 3 --no-extra --no-cpu-baseline > $OUT/ab_$L.$r.json 2>&1
  done
done
unset QUDAX_LIB
timeout 900 python bench.py > $OUT/bench.json 2> $OUT/bench.err
ls -la $OUT

#!/bin/bash
# Round-2 pass D: GPU tests; solver-step A/B against the round-1 head (old_r01 worktree, same box);
# step time without per-launch events; in-step per-kind breakdown; multi-RHS register-cap variants.
TAG=${1:-r02d}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 1500 python -m pytest tests/gpu -v -rs --timeout 240 -p no:cacheprovider > $OUT/pytest_gpu.log 2>&1; echo rc=$? >> $OUT/pytest_gpu.log
for r in 1 2; do
  (cd old_r01 && timeout 300 python bench.py --steps 20 --warmup 3 --no-extra --no-cpu-baseline > ../$OUT/ab_old.$r.json 2>&1)
  timeout 300 python bench.py --steps 20 --warmup 3 --no-extra --no-cpu-baseline > $OUT/ab_new.$r.json 2>&1
  timeout 300 python bench.py --steps 20 --warmup 3 --no-extra --no-cpu-baseline --no-kernel-timing > $OUT/ab_new_noev.$r.json 2>&1
done
timeout 300 python bench.py --steps 20 --warmup 3 --no-extra --no-cpu-baseline --breakdown > $OUT/breakdown.json 2> $OUT/breakdown.err
for L in default mrminb5 mrminb3; do
  if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
  timeout 300 python scripts/bench_dslash.py --cases f32-12,h-12 --reps 20 --nrhs 8 --tag $L >> $OUT/mr.log 2>&1
done
unset QUDAX_LIB
ls -la $OUT

#!/bin/bash
# Round-2 pass AE: final evidence of the head — full GPU tests, smoke, bench line (full), strong
# N=1, reference arm, launch list, ncu of the solver Dslash, per-kind Dslash table; ncu of the
# fp32 recon-8 clover-inverse kernel, head and round 1 (the remaining standalone regression).
TAG=${1:-r02ae}
OUT=gpurun_out/$TAG
mkdir -p $OUT
timeout 1500 python -m pytest tests/gpu -q -rs --timeout 600 -p no:cacheprovider > $OUT/pytest_gpu.log 2>&1; echo rc=$? >> $OUT/pytest_gpu.log
timeout 200 python -c "import __graft_entry__ as g; g.smoke()" > $OUT/smoke.log 2>&1; echo rc=$? >> $OUT/smoke.log
bash scripts/profile_round.sh $TAG
timeout 600 python bench.py --scaling strong --no-extra > $OUT/bench_strong_n1.json 2> $OUT/bench_strong.err
timeout 600 python bench.py --impl reference --steps 3 --warmup 3 > $OUT/bench_reference.json 2> $OUT/bench_reference.err
timeout 600 python scripts/bench_dslash.py --cases f32-12,f32-18,f32-8,h-12,h-18,h-8,f64-18,f64-12 --reps 30 --nrhs 2,4,8 > $OUT/bench_dslash.jsonl 2>&1
K='regex:dslash_kernel<\(int\)4, \(int\)8, \(bool\)0, \(int\)1'
timeout 600 ncu --set full --clock-control none --import-source on --kernel-name-base demangled \
  -k "$K" --launch-skip 5 --launch-count 1 -o $OUT/ci_f8 python scripts/bench_dslash.py --cases f32-8 --reps 3 > $OUT/ncu_ci_f8.log 2>&1
(cd old_r01 && timeout 600 ncu --set full --clock-control none --import-source on --kernel-name-base demangled \
  -k "$K" --launch-skip 5 --launch-count 1 -o ../$OUT/ci_f8_old python scripts/bench_dslash.py --cases f32-8 --reps 3 > ../$OUT/ncu_ci_f8_old.log 2>&1)
ls -la $OUT

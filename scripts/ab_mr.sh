# multi-RHS Dslash: NR right-hand sides per thread (default) vs one (QUDAX_MR_OFF), 2 alternating rounds
mkdir -p gpurun_out/$1
for r in 1 2; do
  timeout 300 python scripts/bench_dslash.py --cases ${2:-f32-12,h-12} --reps 20 --nrhs 2,4,8 --tag mr >> gpurun_out/$1/ab.log 2>&1
  QUDAX_MR_OFF=1 timeout 300 python scripts/bench_dslash.py --cases ${2:-f32-12,h-12} --reps 20 --nrhs 2,4,8 --tag off >> gpurun_out/$1/ab.log 2>&1
done

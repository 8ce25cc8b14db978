# End-of-round evidence: GPU tests, bench line + launch list + ncu of the solver Dslash
# (profile_round.sh), per-kernel Dslash table, ncu of the half and multi-RHS kernels.
TAG=${1:-r01g}
mkdir -p gpurun_out/$TAG
timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/$TAG/pytest_gpu.log 2>&1; echo rc=$? >> gpurun_out/$TAG/pytest_gpu.log
bash scripts/profile_round.sh $TAG
timeout 600 python scripts/bench_dslash.py --cases f32-12,f32-18,f32-8,h-12,h-18,h-8,f64-18,f64-12 --reps 30 --nrhs 2,4,8 > gpurun_out/$TAG/bench_dslash.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on --kernel-name-base demangled \
  -k "regex:dslash_kernel<\(int\)2, \(int\)12, \(bool\)0, \(int\)1" --launch-skip 5 --launch-count 1 -o gpurun_out/$TAG/h12_inv \
  python scripts/bench_dslash.py --cases h-12 --reps 3 > gpurun_out/$TAG/ncu_h12.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on --kernel-name-base demangled \
  -k "regex:dslash_mr_kernel<\(int\)4, \(int\)12, \(bool\)0, \(int\)2" --launch-skip 2 --launch-count 1 -o gpurun_out/$TAG/mr_f12_xpay \
  python scripts/bench_dslash.py --cases f32-12 --reps 3 --nrhs 8 > gpurun_out/$TAG/ncu_mr.log 2>&1
for f in h12_inv mr_f12_xpay; do ncu -i gpurun_out/$TAG/$f.ncu-rep --page source --csv > gpurun_out/$TAG/${f}_source.csv 2>/dev/null; done
ls -la gpurun_out/$TAG

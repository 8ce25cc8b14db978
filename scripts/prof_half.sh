mkdir -p gpurun_out/h1
python scripts/bench_dslash.py --cases f32-12,h-12,h-18,f64-18 --reps 30 > gpurun_out/h1/bench_dslash.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on --kernel-name-base demangled \
  -k "regex:dslash_kernel<\(int\)2, \(int\)12" --launch-skip 5 --launch-count 1 -o gpurun_out/h1/h12_hop \
  python scripts/bench_dslash.py --cases h-12 --reps 3 > gpurun_out/h1/ncu1.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on --kernel-name-base demangled \
  -k "regex:dslash_kernel<\(int\)4, \(int\)12" --launch-skip 5 --launch-count 1 -o gpurun_out/h1/f12_hop \
  python scripts/bench_dslash.py --cases f32-12 --reps 3 > gpurun_out/h1/ncu2.log 2>&1
ls -la gpurun_out/h1

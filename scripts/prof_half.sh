# ncu --set full of the half / fp32 recon-12 clover-inverse Dslash (bench_dslash launches)
mkdir -p gpurun_out/h2
for spec in "h-12:2, \(int\)12, \(bool\)0, \(int\)1" "f32-12:4, \(int\)12, \(bool\)0, \(int\)1"; do
  c=${spec%%:*}; k=${spec#*:}
  timeout 900 ncu --set full --clock-control none --import-source on --kernel-name-base demangled \
    -k "regex:dslash_kernel<\(int\)$k" --launch-skip 5 --launch-count 1 -o gpurun_out/h2/$c \
    python scripts/bench_dslash.py --cases $c --reps 3 > gpurun_out/h2/ncu_$c.log 2>&1
  ncu -i gpurun_out/h2/$c.ncu-rep --page source --csv > gpurun_out/h2/${c}_source.csv 2>/dev/null
done
ls -la gpurun_out/h2

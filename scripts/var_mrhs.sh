# multi-RHS variant study (experiment builds under paper_1011_0024_b200/lib_var)
mkdir -p gpurun_out/mrhs
for v in default w wl l; do
  if [ $v = default ]; then L=""; else L=paper_1011_0024_b200/lib_var/$v/libqudax.so; fi
  QUDAX_LIB=$L python scripts/bench_dslash.py --cases f32-12,h-12 --reps 30 --nrhs 2,4,8 --tag $v >> gpurun_out/mrhs/var.log 2>&1
done

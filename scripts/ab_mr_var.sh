# multi-RHS variants (lib_var builds) vs default, 2 alternating rounds: bash scripts/ab_mr_var.sh TAG "libs"
mkdir -p gpurun_out/$1
for r in 1 2; do
  for L in default $2; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    timeout 300 python scripts/bench_dslash.py --cases f32-12,h-12 --reps 20 --nrhs 2,4,8 --tag $L >> gpurun_out/$1/ab.log 2>&1
  done
done
unset QUDAX_LIB

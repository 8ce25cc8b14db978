# A/B of Dslash kernel variants (bench_dslash.py, alternating libraries, 2 rounds)
# usage: bash scripts/ab_dslash.sh TAG "lib1 lib2 ..." [cases] [nrhs]
TAG=$1; LIBS=$2; CASES=${3:-f32-12,h-12,h-18,f64-18}; NRHS=${4:-}
mkdir -p gpurun_out/$TAG
for r in 1 2; do
  for L in $LIBS; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    timeout 300 python scripts/bench_dslash.py --cases $CASES --reps 30 ${NRHS:+--nrhs $NRHS} --tag $L >> gpurun_out/$TAG/ab.log 2>&1
  done
done
unset QUDAX_LIB

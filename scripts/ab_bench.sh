# A/B of the solver step: default lib vs an experiment build (alternating, 3 rounds)
mkdir -p gpurun_out/ab
for i in 1 2 3; do
  python bench.py --no-extra --no-cpu-baseline > gpurun_out/ab/a$i.json 2>/dev/null
  QUDAX_LIB=$1 python bench.py --no-extra --no-cpu-baseline > gpurun_out/ab/b$i.json 2>/dev/null
done

# A/B of the solver step (bench.py --no-extra) across library variants, per-kind Dslash times
# (QUDAX_TIMING_BREAKDOWN), 2 alternating rounds: bash scripts/ab_step.sh TAG "libs"
mkdir -p gpurun_out/$1
for r in 1 2; do
  for L in $2; do
    if [ "$L" = default ]; then unset QUDAX_LIB; else export QUDAX_LIB=paper_1011_0024_b200/lib_var/$L/libqudax.so; fi
    QUDAX_TIMING_BREAKDOWN=1 timeout 300 python bench.py --no-extra --no-cpu-baseline --steps 5 --warmup 3 > gpurun_out/$1/$L.$r.json 2> gpurun_out/$1/$L.$r.err
    echo "$L $r $(python -c "import json;d=json.load(open('gpurun_out/$1/$L.$r.json'));print(round(d['value']),round(d['ms_per_step'],2),d['clocks']['sm_mhz'])") $(grep 'qudax timing: prec 4' gpurun_out/$1/$L.$r.err | awk '{print $9}' | tr '\n' ' ')" >> gpurun_out/$1/summary.txt
  done
done
unset QUDAX_LIB
cat gpurun_out/$1/summary.txt

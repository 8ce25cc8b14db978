# A/B of the solver step under two environment settings (2 alternating rounds):
#   bash scripts/ab_env.sh TAG "VAR=a" "VAR=b"
mkdir -p gpurun_out/$1
for r in 1 2; do
  for E in "$2" "$3"; do
    env $E QUDAX_TIMING_BREAKDOWN=1 timeout 300 python bench.py --no-extra --no-cpu-baseline --steps 5 --warmup 3 > gpurun_out/$1/run.json 2> gpurun_out/$1/run.err
    echo "$E $r $(python -c "import json;d=json.load(open('gpurun_out/$1/run.json'));print(round(d['value']),round(d['ms_per_step'],2),d['clocks']['sm_mhz'])") $(grep 'qudax timing: prec 4' gpurun_out/$1/run.err | awk '{print $12}' | tr '\n' ' ')" >> gpurun_out/$1/summary.txt
  done
done
cat gpurun_out/$1/summary.txt

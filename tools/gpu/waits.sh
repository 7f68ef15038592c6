# wait-strategy A/B (OCL_WAIT=<producer><consumer>) on C4 and C5 points
TAG=${TAG:-waits}
mkdir -p gpurun_out/$TAG
for w in 00 10 12 22 11; do
  for a in "--workload c4" "--workload c5 --c5-groups 16" "--workload c5 --c5-groups 256" "--workload c5 --c5-groups 4"; do
    OCL_WAIT=$w timeout 300 python bench.py --no-cpu --no-e2e --steps 20 $a > /tmp/b.json 2>&1
    python -c "
import json,sys
d=json.loads(open('/tmp/b.json').read().strip().splitlines()[-1]); print('$w', '$a', round(d['ms_per_step'],4), round(d['roofline']['kernel_ms'],4), d['roofline']['kernel'])" >> gpurun_out/$TAG/waits.txt 2>&1 || tail -3 /tmp/b.json >> gpurun_out/$TAG/waits.txt
  done
done
cat gpurun_out/$TAG/waits.txt

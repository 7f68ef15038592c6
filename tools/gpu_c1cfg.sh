for rep in 1 2; do for c in 7 5 3 6; do
  OCL_BULK=$c timeout 200 python bench.py --workload c1 --no-e2e --no-cpu --steps 100 > /tmp/c1_$c.json 2>&1
  echo c1 $c $(python -c "import json,sys;d=json.loads(open('/tmp/c1_$c.json').read().strip().splitlines()[-1]);print(d['ms_per_step'],d['roofline']['kernel_ms'])")
done; done

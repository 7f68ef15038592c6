summ() { python -c "import json,sys; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('$1', d['ms_per_step'], d['value']/1e9, d['roofline']['kernel_ms'])"; }
timeout 900 python -m pytest tests/test_gpu_sorted.py tests/test_gpu_radix.py -x -q 2>&1 | tail -1
for k in 4 8; do OCL_SORTED_K=$k timeout 300 python bench.py --workload c3c --no-cpu --no-e2e --steps 20 2>&1 | summ c3c-K$k; done
timeout 300 python bench.py --workload c3s --no-cpu --no-e2e --steps 10 2>&1 | summ c3s

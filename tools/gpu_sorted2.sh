summ() { python -c "import json,sys; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('$1', d['ms_per_step'], d['value']/1e9, d['roofline']['kernel_ms'])"; }
timeout 900 python -m pytest tests/test_gpu_sorted.py -x -q 2>&1 | tail -2
for k in 4 8; do OCL_SORTED_K=$k timeout 300 python bench.py --workload c3c --no-cpu --no-e2e --steps 20 2>&1 | summ c3c-K$k; done
timeout 300 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum,smsp__inst_executed.sum --clock-control none --csv python bench.py --workload c3c --steps 1 --warmup 1 --no-e2e --no-cpu > gpurun_out/c3c_launches.csv 2>/dev/null
python tools/launches.py gpurun_out/c3c_launches.csv 2>&1 | tail -4

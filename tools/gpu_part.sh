summ() { python -c "import json,sys; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('$1', d['ms_per_step'], d['value']/1e9, d['config']['groups'])"; }
timeout 900 python -m pytest tests/test_gpu_parity.py -x -q 2>&1 | tail -3
timeout 300 python bench.py --workload c3 --no-cpu --no-e2e --steps 10 2>&1 | summ c3
for g in 65536 16777216; do for z in 0.0 1.0; do timeout 200 python bench.py --workload c5 --c5-groups $g --c5-zipf $z --no-cpu --no-e2e --steps 5 2>&1 | summ "c5_G=${g}_z=$z"; done; done
timeout 300 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv python bench.py --workload c3 --steps 1 --warmup 0 --no-e2e --no-cpu > gpurun_out/c3_launches.csv 2>/dev/null
python tools/launches.py gpurun_out/c3_launches.csv 14 | grep -v elementwise

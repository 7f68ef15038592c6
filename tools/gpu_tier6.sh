summ() { python -c "import json,sys; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('$1', d['ms_per_step'], d['value']/1e9, d['roofline']['kernel'])"; }
for t in 0 6; do timeout 300 python bench.py --workload c3 --tier $t --no-cpu --no-e2e --steps 10 2>&1 | summ c3-tier$t; done
timeout 300 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv python bench.py --workload c3 --tier 6 --steps 1 --warmup 0 --no-e2e --no-cpu > gpurun_out/c3t6_launches.csv 2>/dev/null
python tools/launches.py gpurun_out/c3t6_launches.csv 60 | grep -v elementwise | awk '{print $1, $2, $3, $4, $(NF-3), $(NF-2), $(NF-1), $NF}' | head -60

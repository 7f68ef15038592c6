# scratch driver for gpurun iterations (tests + high-cardinality benches + launch list)
summ() { python -c "import json,sys; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('$1', d['ms_per_step'], d['value']/1e9, d['roofline']['kernel'])"; }
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -x -q -k "partitioned or many_groups or c3 or sweep" 2>&1 | tail -2
for w in c3 c3c; do timeout 300 python bench.py --workload $w --no-cpu --no-e2e --steps 10 2>&1 | summ $w; done
for g in 65536 16777216; do for z in 0.0 1.5; do timeout 200 python bench.py --workload c5 --c5-groups $g --c5-zipf $z --no-cpu --no-e2e --steps 10 2>&1 | summ "c5_G=${g}_z=$z"; done; done
timeout 300 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv python bench.py --workload c5 --c5-groups 16777216 --c5-zipf 0 --no-cpu --no-e2e --steps 1 --warmup 0 > gpurun_out/c5_launches.csv 2>/dev/null

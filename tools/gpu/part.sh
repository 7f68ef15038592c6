TAG=${TAG:-part}
mkdir -p gpurun_out/$TAG
timeout 1200 python -m pytest -q -m gpu tests/test_gpu_parity.py -k "partitioned or c3 or many_groups or sweep or routed" tests/test_gpu_c5_grid.py > gpurun_out/$TAG/pytest.log 2>&1; tail -3 gpurun_out/$TAG/pytest.log
for w in c3 c3s; do timeout 300 python bench.py --workload $w --no-e2e --no-cpu > gpurun_out/$TAG/bench_$w.json 2>&1; python -c "
import json; d=json.loads(open('gpurun_out/$TAG/bench_$w.json').read().strip().splitlines()[-1]); print('$w', round(d['ms_per_step'],4), d['roofline']['kernel'])"; done
for g in 16384 1048576 16777216; do timeout 300 python bench.py --workload c5 --c5-groups $g --no-e2e --no-cpu > gpurun_out/$TAG/bench_c5_$g.json 2>&1; python -c "
import json; d=json.loads(open('gpurun_out/$TAG/bench_c5_$g.json').read().strip().splitlines()[-1]); print('c5 $g', round(d['ms_per_step'],4), d['roofline']['kernel'])"; done

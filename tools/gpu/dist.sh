# distributed path + timed-kernel parity tests, the default bench and the --dist overhead bench
TAG=${TAG:-dist}
mkdir -p gpurun_out/$TAG
timeout 1500 python -m pytest -q tests/test_gpu_distributed.py tests/test_gpu_timed.py tests/test_gpu_parity.py > gpurun_out/$TAG/pytest.log 2>&1
tail -5 gpurun_out/$TAG/pytest.log
timeout 400 python bench.py --no-cpu > gpurun_out/$TAG/bench_c4.json 2> gpurun_out/$TAG/bench_c4.err
timeout 400 python bench.py --no-cpu --dist > gpurun_out/$TAG/bench_c4_dist.json 2> gpurun_out/$TAG/bench_c4_dist.err
timeout 400 python bench.py --no-cpu --no-e2e --workload c1 > gpurun_out/$TAG/bench_c1.json 2> gpurun_out/$TAG/bench_c1.err
timeout 400 python bench.py --no-cpu --no-e2e --workload c1 --dist > gpurun_out/$TAG/bench_c1_dist.json 2> gpurun_out/$TAG/bench_c1_dist.err
tail -2 gpurun_out/$TAG/*.err
true

# parity of the signature kernels, then bench lines and a C5 sweep subset; logs under gpurun_out/$TAG
TAG=${TAG:-c5}
mkdir -p gpurun_out/$TAG
timeout 1200 python -m pytest -q -x tests/test_gpu_timed.py > gpurun_out/$TAG/pytest.log 2>&1
tail -3 gpurun_out/$TAG/pytest.log
for w in c4 c4mm c2; do OCL_DEBUG=1 timeout 400 python bench.py --no-cpu --no-e2e --workload $w > gpurun_out/$TAG/bench_$w.json 2>&1; done
timeout 900 python tools/sweep_c5.py --steps 5 --groups ${C5G:-2,4,5,6,8,10,11} --out gpurun_out/$TAG/c5.json > gpurun_out/$TAG/c5.log 2>&1
cat gpurun_out/$TAG/c5.md
true

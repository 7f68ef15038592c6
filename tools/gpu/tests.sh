# GPU test suite (+ optional pytest args) and the default bench line; logs under gpurun_out/$TAG.
TAG=${TAG:-tests}
mkdir -p gpurun_out/$TAG
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv > gpurun_out/$TAG/gpu.txt 2>&1
timeout ${PYT_TIMEOUT:-1800} python -m pytest tests -m gpu -q -x ${PYTEST_ARGS} > gpurun_out/$TAG/pytest_gpu.log 2>&1
tail -5 gpurun_out/$TAG/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/$TAG/smoke.log 2>&1; tail -1 gpurun_out/$TAG/smoke.log
[ -n "$BENCH" ] && timeout 400 python bench.py > gpurun_out/$TAG/bench_c4.json 2> gpurun_out/$TAG/bench_c4.err
true

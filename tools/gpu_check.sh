# Confirmation pass: GPU parity suite, smoke, default bench line.
mkdir -p gpurun_out/check
timeout 1500 python -m pytest tests -m gpu -x -q > gpurun_out/check/pytest_gpu.log 2>&1; echo "pytest rc=$?"
tail -3 gpurun_out/check/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -2
timeout 400 python bench.py > gpurun_out/check/bench_c4.json 2> gpurun_out/check/bench_c4.err; tail -c 600 gpurun_out/check/bench_c4.json

mkdir -p gpurun_out/last
timeout 1500 python -m pytest tests -m gpu -q > gpurun_out/last/pytest_gpu.log 2>&1; tail -1 gpurun_out/last/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -1
timeout 400 python bench.py > gpurun_out/last/bench_c4.json 2> gpurun_out/last/bench_c4.err; tail -c 300 gpurun_out/last/bench_c4.json
timeout 1200 python tools/sweep_c5.py --steps 5 --out gpurun_out/last/c5_sweep.json > gpurun_out/last/c5_sweep.log 2>&1; tail -1 gpurun_out/last/c5_sweep.log

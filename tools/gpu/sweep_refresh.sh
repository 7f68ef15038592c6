TAG=r02g
O=gpurun_out/$TAG
mkdir -p $O
timeout 900 python -m pytest -q -x tests/test_gpu_parity.py -m gpu -k "partition or c3 or many_groups or sweep_c5 or partial" > $O/pytest.log 2>&1; tail -1 $O/pytest.log
timeout 900 python -m pytest -q -x tests/test_gpu_c5_grid.py -m gpu 2>&1 | tail -1
b() { n=$1; shift; timeout 600 python bench.py "$@" > $O/bench_$n.json 2> $O/bench_$n.err; tail -c 120 $O/bench_$n.json; echo; }
for g in 4096 65536 1048576; do b c5_g$g --workload c5 --c5-groups $g --no-e2e --no-cpu; done
timeout 1800 python tools/sweep_c5.py --steps 5 --out $O/c5_sweep.json > $O/c5_sweep.log 2>&1
ls $O | wc -l

# End-of-round checks: full GPU suite, smoke, default bench line, reference arm, J3 line + launch list
TAG=${TAG:-r02e}
O=gpurun_out/$TAG
mkdir -p $O
timeout 1800 python -m pytest tests -m gpu -q -x > $O/pytest_gpu.log 2>&1; tail -1 $O/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" > $O/smoke.log 2>&1; tail -1 $O/smoke.log
b() { n=$1; shift; timeout 600 python bench.py "$@" > $O/bench_$n.json 2> $O/bench_$n.err; tail -c 160 $O/bench_$n.json; echo; }
b c4
b reference --impl reference --steps 3 --warmup 1
b j3 --workload j3 --no-cpu
b c3 --workload c3 --no-e2e --no-cpu
M=gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum,lts__t_sectors_op_atom.sum,lts__t_sectors_op_red.sum,l1tex__data_pipe_lsu_wavefronts_mem_shared_op_atom.sum
timeout 600 ncu --metrics $M --clock-control none --csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu --workload j3 > $O/j3_launches.csv 2>/dev/null; python tools/launches.py $O/j3_launches.csv 40 > $O/j3_launches.txt 2>&1
timeout 600 ncu --metrics $M --clock-control none --csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu > $O/c4_launches.csv 2>/dev/null; python tools/launches.py $O/c4_launches.csv 40 > $O/c4_launches.txt 2>&1
ls $O | wc -l

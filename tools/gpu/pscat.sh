# Partitioned tier pass-1b A/B: parity of the tier-5 tests and the C5 grid, C3 timing per OCL_PSCAT mode,
# eager vs lazy table zeroing, and the C3 launch list.
TAG=${TAG:-pscat}
O=gpurun_out/$TAG
mkdir -p $O
timeout 1500 python -m pytest -q -x tests/test_gpu_parity.py -m gpu -k "partition or c3 or many_groups or sweep_c5 or near_full or partials" > $O/pytest.log 2>&1; tail -2 $O/pytest.log
[ -z "$NOGRID" ] && { timeout 1500 python -m pytest -q -x tests/test_gpu_c5_grid.py -m gpu > $O/grid.log 2>&1; tail -2 $O/grid.log; }
for r in 1 2; do
for e in "OCL_PSCAT=0" "OCL_PSCAT=1" "OCL_PSCAT=2" "OCL_PSCAT=0 OCL_PART_EAGER=1" ${EXTRA}; do
  env $e timeout 300 python bench.py --workload c3 --no-e2e --no-cpu --steps 20 2>/dev/null | python -c "import json,sys; d=json.loads(sys.stdin.read()); print('$e', round(d['ms_per_step'],4), round(d['roofline']['kernel_ms'],4))"
done
done | tee $O/ab.txt
M=gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum,lts__t_sectors_op_atom.sum,lts__t_sectors_op_red.sum,l1tex__data_pipe_lsu_wavefronts_mem_shared_op_atom.sum
timeout 600 ncu --metrics $M --clock-control none --csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu --workload c3 > $O/c3_launches.csv 2>/dev/null
python tools/launches.py $O/c3_launches.csv 40 > $O/c3_launches.txt 2>&1; head -30 $O/c3_launches.txt

# ncu launch lists (per-kernel time, DRAM bytes, L2 atomic / reduction sectors) for bench workloads
TAG=${TAG:-launches}
mkdir -p gpurun_out/$TAG
M=gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum,lts__t_sectors_op_atom.sum,lts__t_sectors_op_red.sum,l1tex__data_pipe_lsu_wavefronts_mem_shared_op_atom.sum
for pair in $PAIRS; do
  name=${pair%%=*}; args=${pair#*=}
  timeout 900 ncu --metrics $M --clock-control none --csv python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu ${args//,/ } \
    > gpurun_out/$TAG/${name}_launches.csv 2> gpurun_out/$TAG/${name}.err
done
ls -la gpurun_out/$TAG

# Evidence refresh for the paths the partitioned-tier work changed: C3 / C5 bench lines, launch lists,
# full ncu of the C3 passes, the C5 sweep
TAG=${TAG:-r02c}
O=gpurun_out/$TAG
mkdir -p $O
b() { n=$1; shift; timeout 600 python bench.py "$@" > $O/bench_$n.json 2> $O/bench_$n.err; tail -c 200 $O/bench_$n.json; echo; }
b c3 --workload c3 --no-e2e
for g in 4096 65536 1048576 16777216; do b c5_g$g --workload c5 --c5-groups $g --no-e2e --no-cpu; done
b c5_g256_sel1 --workload c5 --c5-groups 256 --c5-sel 0.01 --no-e2e --no-cpu
b c5_g1024_sel1 --workload c5 --c5-groups 1024 --c5-sel 0.01 --no-e2e --no-cpu
b c5_g65536_sel1 --workload c5 --c5-groups 65536 --c5-sel 0.01 --no-e2e --no-cpu
b c5_g16777216_sel1 --workload c5 --c5-groups 16777216 --c5-sel 0.01 --no-e2e --no-cpu
M=gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum,lts__t_sectors_op_atom.sum,lts__t_sectors_op_red.sum,l1tex__data_pipe_lsu_wavefronts_mem_shared_op_atom.sum
l() { n=$1; shift; timeout 900 ncu --metrics $M --clock-control none --csv python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu "$@" > $O/${n}_launches.csv 2>/dev/null; python tools/launches.py $O/${n}_launches.csv 60 > $O/${n}_launches.txt 2>&1; }
l c3 --workload c3
for g in 65536 16777216; do l c5_g$g --workload c5 --c5-groups $g; done
f() { n=$1; k=$2; shift 2; timeout 900 ncu --set full --import-source on --clock-control none -k regex:$k -s 1 -c 1 -o $O/$n -f python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu "$@" > /dev/null 2>&1
  ncu -i $O/$n.ncu-rep --page details --csv > $O/${n}_details.csv 2>/dev/null; rm -f $O/$n.ncu-rep; }
f c3_agg_full k_part_agg --workload c3; f c3_l1_full k_part_scatter_l1 --workload c3; f c3_s2_full k_part_scatter2 --workload c3; f c5_g65536_agg_full k_part_agg --workload c5 --c5-groups 65536
timeout 1800 python tools/sweep_c5.py --steps 5 --out $O/c5_sweep.json > $O/c5_sweep.log 2>&1
ls $O | wc -l

# ncu --set full of the unfused a7 / a4 kernels (tools/bench_ops.py at $ROWS rows), hot-line summaries
TAG=${TAG:-ncuops2}
O=gpurun_out/$TAG
mkdir -p $O
timeout 600 python tools/bench_ops.py --steps 5 --warmup 2 --rows ${ROWS:-600000000} > $O/ops.json 2>&1; python -c "
import json; d=json.loads(open('$O/ops.json').read())
print({k: (round(v['ms'],3), round(v['frac'],3)) for k,v in d['ops'].items()})"
for spec in "a7:k_group_aggregate" "a4:k_group_build" "a2:k_prefix_compact" "a1_select_bitmap_u8:k_select_bitmap"; do
  only=${spec%%:*}; k=${spec##*:}
  timeout 900 ncu --set full --import-source on --clock-control none -k regex:$k -s 2 -c 1 -o $O/$only -f \
    python tools/bench_ops.py --only $only --steps 1 --warmup 1 --rows ${ROWS:-200000000} > $O/$only.log 2>&1
  ncu -i $O/$only.ncu-rep --page details --csv > $O/${only}_details.csv 2>/dev/null
  ncu -i $O/$only.ncu-rep --page source --csv --print-source cuda,sass > $O/${only}_src.csv 2>/dev/null
  python tools/src_hot.py $O/${only}_src.csv 30 > $O/${only}_hot.txt 2>&1; gzip -f $O/${only}_src.csv; rm -f $O/$only.ncu-rep
done
ls $O

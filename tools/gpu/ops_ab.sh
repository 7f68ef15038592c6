# Unfused operators: A/B of env settings ($ENVS, ';'-separated) on tools/bench_ops.py --only $ONLY; optional ncu of $K
TAG=${TAG:-opsab}
O=gpurun_out/$TAG
mkdir -p $O
IFS=';' read -ra LIST <<< "$ENVS"
for r in 1 2; do
for e in "${LIST[@]}"; do
  lab="$e"; [ "$e" = "-" ] && e=""
  env $e timeout 600 python tools/bench_ops.py --only ${ONLY:-a} --steps 5 --warmup 2 > $O/o.json 2>&1
  python -c "
import json; d=json.loads(open('$O/o.json').read())
print('$lab', {k: (round(v['ms'],3), round(v['frac'],3)) for k,v in d['ops'].items()})" || tail -3 $O/o.json
done
done | tee $O/ab.txt
if [ -n "$K" ]; then
  timeout 900 ncu --set full --import-source on --clock-control none -k regex:$K -s ${SKIP:-1} -c 1 -o $O/k -f \
    python tools/bench_ops.py --only $ONLY --steps 1 --warmup 1 --rows ${ROWS:-200000000} > $O/ncu.log 2>&1
  ncu -i $O/k.ncu-rep --page details --csv > $O/k_details.csv 2>/dev/null
  ncu -i $O/k.ncu-rep --page source --csv --print-source cuda,sass > $O/k_src.csv 2>/dev/null
  python tools/src_hot.py $O/k_src.csv 40 > $O/k_hot.txt 2>&1; gzip -f $O/k_src.csv; rm -f $O/k.ncu-rep
fi

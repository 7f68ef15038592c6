# C3 A/B over env settings ($ENVS, ';'-separated, "-" = none) + optional ncu of one kernel ($K)
TAG=${TAG:-c3ab}
O=gpurun_out/$TAG
mkdir -p $O
[ -n "$TESTS" ] && { timeout 1500 python -m pytest -q -x tests/test_gpu_parity.py -m gpu -k "$TESTS" > $O/pytest.log 2>&1; tail -2 $O/pytest.log; }
IFS=';' read -ra LIST <<< "$ENVS"
for r in 1 2; do
for e in "${LIST[@]}"; do
  lab="$e"; [ "$e" = "-" ] && e=""
  env $e timeout 300 python bench.py --workload ${WL:-c3} ${BARGS} --no-e2e --no-cpu --steps 20 2>/dev/null | python -c "import json,sys; d=json.loads(sys.stdin.read()); print('$lab', round(d['ms_per_step'],4), round(d['roofline']['kernel_ms'],4))"
done
done | tee $O/ab.txt
if [ -n "$K" ]; then
  timeout 900 ncu --set full --import-source on --clock-control none -k regex:$K -s 1 -c 1 -o $O/k -f \
    python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu --workload ${WL:-c3} ${BARGS} > $O/ncu.log 2>&1
  ncu -i $O/k.ncu-rep --page details --csv > $O/k_details.csv 2>/dev/null
  ncu -i $O/k.ncu-rep --page source --csv --print-source cuda,sass > $O/k_src.csv 2>/dev/null
  ncu -i $O/k.ncu-rep --page raw --csv > $O/k_raw.csv 2>/dev/null
  python tools/src_hot.py $O/k_src.csv 40 > $O/k_hot.txt 2>&1; gzip -f $O/k_src.csv; rm -f $O/k.ncu-rep
fi

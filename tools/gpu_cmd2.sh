summ() { python -c "import json,sys; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('$1', d['ms_per_step'], d['value']/1e9, d['roofline']['kernel'])"; }
for t in 0 1 2 5; do for w in c3 c3c; do timeout 300 python bench.py --workload $w --tier $t --no-cpu --no-e2e --steps 5 2>&1 | summ "$w-tier$t"; done; done
for t in 1 5; do for g in 4096 65536 1048576 16777216; do for z in 0.0 1.0; do timeout 300 python bench.py --workload c5 --tier $t --c5-groups $g --c5-zipf $z --no-cpu --no-e2e --steps 5 2>&1 | summ "c5-tier$t-G$g-z$z"; done; done; done

summ() { python -c "import json,sys; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('$1', round(d['ms_per_step'],3), d['roofline']['kernel'][:40])"; }
for g in 1024 2048 4096; do for t in 0 5; do for sel in 0.5 1.0; do timeout 200 python bench.py --workload c5 --tier $t --c5-groups $g --c5-sel $sel --no-cpu --no-e2e --steps 5 2>&1 | summ "G=$g tier=$t sel=$sel"; done; done; done

summ() { python -c "import json,sys; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('$1', round(d['ms_per_step'],3), d['roofline']['kernel'][:32])"; }
timeout 900 python -m pytest tests/test_gpu_parity.py -x -q 2>&1 | tail -1
for g in 4 16 256 1024; do for sel in 0.01 0.5 1.0; do timeout 200 python bench.py --workload c5 --c5-groups $g --c5-sel $sel --no-cpu --no-e2e --steps 5 2>&1 | summ "G=$g sel=$sel"; done; done

timeout 600 python -m pytest tests -m gpu -x -q 2>&1 | tail -2
for rep in 1 2; do for c in 0 2 3 4 5 6 7; do OCL_BULK=$c timeout 200 python bench.py --no-cpu --no-e2e --steps 30 2>&1 | python -c "import json,sys; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('cfg','$c', d['ms_per_step'], d['roofline']['kernel_ms'], d['roofline']['frac'], d['roofline']['kernel'])"; done; done

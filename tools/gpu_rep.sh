summ() { python -c "import json,sys; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('$1', round(d['ms_per_step'],3), d['roofline']['kernel'][:40])"; }
timeout 900 python -m pytest tests/test_gpu_parity.py -x -q 2>&1 | tail -1
for g in 16 64 256 1024; do for z in 0.0 1.5; do for rep in 1 0; do if [ $rep = 1 ]; then E="OCL_CTA_REP=1"; else E=""; fi; env $E timeout 200 python bench.py --workload c5 --c5-groups $g --c5-zipf $z --no-cpu --no-e2e --steps 5 2>&1 | summ "G=$g z=$z ${E:-auto}"; done; done; done

# Partitioned tier A/B: current build vs build/base (OCL_LIB_PATH) on C3 and C5 high-G points; parity subset
TAG=${TAG:-partab}
O=gpurun_out/$TAG
mkdir -p $O
[ -n "$TESTS" ] && { timeout 1500 python -m pytest -q -x tests/test_gpu_parity.py -m gpu -k "$TESTS" > $O/pytest.log 2>&1; tail -1 $O/pytest.log; [ -n "$GRID" ] && timeout 900 python -m pytest -q -x tests/test_gpu_c5_grid.py -m gpu 2>&1 | tail -1; }
for r in 1 2; do
for L in "-" "$PWD/build/base/libocelot_b200.so"; do
  lp=""; [ "$L" != "-" ] && lp="OCL_LIB_PATH=$L"
  for w in "c3" "c5 --c5-groups 4096" "c5 --c5-groups 65536" "c5 --c5-groups 1048576" "c5 --c5-groups 16777216" "c5 --c5-groups 65536 --c5-sel 0.01" "c5 --c5-groups 65536 --c5-zipf 1.5"; do
    env $lp timeout 300 python bench.py --workload $w --no-e2e --no-cpu --steps 10 2>/dev/null | python -c "import json,sys; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('$(basename $(dirname $L))', '$w', round(d['ms_per_step'],4))"
  done
done
done | tee $O/ab.txt

# Full GPU suite + sanitizers over the partitioned-tier cases + the C3 bench line
TAG=${TAG:-vpart}
O=gpurun_out/$TAG
mkdir -p $O
timeout 1800 python -m pytest tests -m gpu -q -x > $O/pytest_gpu.log 2>&1; tail -2 $O/pytest_gpu.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -1
for t in memcheck racecheck synccheck; do
  timeout 1200 /usr/local/cuda/bin/compute-sanitizer --tool $t --error-exitcode 1 --print-limit 20 python tools/sanitize_cases.py ${CASES:-partitioned_two_level fused_groupby_tiers} > $O/sanitize_$t.log 2>&1; echo "$t rc=$?"; tail -2 $O/sanitize_$t.log
done
timeout 300 python bench.py --workload c3 --no-e2e > $O/bench_c3.json 2> $O/bench_c3.err; tail -c 600 $O/bench_c3.json

# select-compact-gather: new parity tests, sanitizers on its case, full GPU suite, A/B vs build/ab/lib_head.so
TAG=${TAG:-sparse}
mkdir -p gpurun_out/$TAG
timeout 900 python -m pytest tests/test_gpu_timed.py -q -x -k "compact_gather or sparse" > gpurun_out/$TAG/pytest_sparse.log 2>&1
tail -3 gpurun_out/$TAG/pytest_sparse.log
for t in memcheck racecheck synccheck; do
  timeout 900 /usr/local/cuda/bin/compute-sanitizer --tool $t --error-exitcode 1 --print-limit 20 \
    python tools/sanitize_cases.py fused_select_compact_gather > gpurun_out/$TAG/sanitize_$t.log 2>&1
  echo "$t rc=$? $(tail -1 gpurun_out/$TAG/sanitize_$t.log)"
done
TAG=$TAG bash tools/gpu/tests.sh
TAG=$TAG LIBS="- build/ab/lib_head.so" ENVS="-" SPECS="${SPECS:-c4 c5:16 c5:256 c5:4:0:0.01 c5:16:1.0:0.01 c5:256:1.0:0.01 c5:1024:1.0:0.01 c5:256:1.0:0.03 c5:256:1.5:0.01 c5:256:1.0:0.05}" bash tools/gpu/abenvs.sh > /dev/null
awk '{print $1, $3, $4}' gpurun_out/$TAG/ab.txt | sort -k2,2 -k1,1 | awk '{a[$1" "$2]=a[$1" "$2]" "$3} END{for(k in a) print k, a[k]}' | sort -k2,2 -k1,1

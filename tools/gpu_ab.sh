summ() { python -c "import json,sys; d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('$1', d['ms_per_step'], d['value']/1e9)"; }
for rep in 1 2; do
for lib in build/oldlib/libocelot_b200.so paper_journals_pvldb_heimelspmm13_b200/_lib/libocelot_b200.so; do
  for w in "c3" "c5 --c5-groups 16777216" "c5 --c5-groups 65536"; do OCL_LIB_PATH=$lib timeout 300 python bench.py --workload $w --no-cpu --no-e2e --steps 5 2>&1 | summ "$lib $w"; done
done; done

TAG=${TAG:-abops}
mkdir -p gpurun_out/$TAG
for so in "" build/ab/*.so; do
  if [ -z "$so" ]; then lib=paper_journals_pvldb_heimelspmm13_b200/_lib/libocelot_b200.so; else lib=$PWD/$so; fi
  OCL_LIB_PATH=$PWD/${lib#$PWD/} timeout 600 python tools/bench_ops.py --only ${ONLY:-a} --steps 5 --warmup 2 > /tmp/o.json 2>&1
  python -c "
import json; d=json.loads(open('/tmp/o.json').read())
print('$(basename $lib)', {k: (round(v['ms'],3), round(v['frac'],3)) for k,v in d['ops'].items()})" >> gpurun_out/$TAG/ab.txt 2>&1 || tail -3 /tmp/o.json >> gpurun_out/$TAG/ab.txt
done
cat gpurun_out/$TAG/ab.txt

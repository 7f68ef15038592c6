"""Summarise an `ncu --metrics gpu__time_duration.sum,dram__bytes_* --csv` launch list (scratch tool)."""
import csv
import io
import sys

lines = [ln for ln in open(sys.argv[1]) if ln.startswith('"')]
rows = list(csv.reader(io.StringIO("".join(lines))))
h = rows[0]
ki, mi, vi, ii = h.index("Kernel Name"), h.index("Metric Name"), h.index("Metric Value"), h.index("ID")
d = {}
for r in rows[1:]:
    d.setdefault((int(r[ii]), r[ki][:48]), {})[r[mi]] = r[vi]
last = int(sys.argv[2]) if len(sys.argv) > 2 else 12
for (i, k), m in sorted(d.items())[-last:]:
    print(i, k, m.get("gpu__time_duration.sum"), "R", m.get("dram__bytes_read.sum"), "W", m.get("dram__bytes_write.sum"))

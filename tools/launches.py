"""Summarise an ncu `--metrics ... --csv` launch list: per kernel launch of the LAST step (the
launches after the last `k_*` table memset marker are not separable, so give the number of launches
per step): time, DRAM read / write bytes, L2 atomic / reduction sectors, shared atomic wavefronts."""
import csv
import io
import sys

lines = [ln for ln in open(sys.argv[1]) if ln.startswith('"')]
rows = list(csv.reader(io.StringIO("".join(lines))))
h = rows[0]
ki, mi, vi, ii = h.index("Kernel Name"), h.index("Metric Name"), h.index("Metric Value"), h.index("ID")
d = {}
for r in rows[1:]:
    d.setdefault((int(r[ii]), r[ki].split("(")[0][:60]), {})[r[mi]] = r[vi].replace(",", "")
last = int(sys.argv[2]) if len(sys.argv) > 2 else 12
tot = {}
print(f"{'id':>4} {'kernel':60s} {'us':>9} {'DRAM R MB':>10} {'DRAM W MB':>10} {'L2 atom':>10} {'L2 red':>10} {'smem atom':>10}")
for (i, k), m in sorted(d.items())[-last:]:
    f = lambda key, s=1.0: float(m.get(key, 0) or 0) / s
    t = f("gpu__time_duration.sum")
    unit = 1e3 if t > 1e3 else 1.0          # ncu reports ns or us depending on version
    row = (t / unit, f("dram__bytes_read.sum", 1e6), f("dram__bytes_write.sum", 1e6), f("lts__t_sectors_op_atom.sum"),
           f("lts__t_sectors_op_red.sum"), f("l1tex__data_pipe_lsu_wavefronts_mem_shared_op_atom.sum"))
    for j, x in enumerate(row):
        tot[j] = tot.get(j, 0) + x
    print(f"{i:4d} {k:60s} {row[0]:9.1f} {row[1]:10.1f} {row[2]:10.1f} {row[3]:10.0f} {row[4]:10.0f} {row[5]:10.0f}")
print(f"{'':4s} {'total':60s} {tot[0]:9.1f} {tot[1]:10.1f} {tot[2]:10.1f} {tot[3]:10.0f} {tot[4]:10.0f} {tot[5]:10.0f}")

"""Top source lines by executed instructions / stall samples from `ncu --page source --csv --print-source cuda,sass` (scratch tool)."""
import csv
import sys

rows = list(csv.reader(open(sys.argv[1])))
n = int(sys.argv[2]) if len(sys.argv) > 2 else 30
agg, fname = [], ""
hdr = None
for r in rows:
    if r and r[0] == "File Path":
        fname = r[1].split("/")[-1]
        continue
    if r and "Instructions Executed" in r:
        hdr = r
        ie, sm = r.index("Instructions Executed"), r.index("Warp Stall Sampling (All Samples)")
        continue
    if hdr and len(r) > ie and r[0] and r[ie] not in ("-", ""):
        try:
            agg.append((int(r[ie]), int(r[sm] or 0), f"{fname}:{r[0]}", r[1][:80]))
        except ValueError:
            pass
ti = sum(a[0] for a in agg) or 1
ts = sum(a[1] for a in agg) or 1
print("total inst", ti, "samples", ts)
for a in sorted(agg, key=lambda a: -a[1])[:n]:
    print(f"{a[0] / ti * 100:5.1f}% inst {a[1] / ts * 100:5.1f}% smp  {a[2]:>22} {a[3]}")

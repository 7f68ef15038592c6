"""Summarise an ncu `--page source --csv --print-source sass` dump: instructions executed and stall samples
per opcode, and the hottest address windows (debug aid)."""
import collections
import csv
import gzip
import io
import sys


def load(path):
    data = (gzip.open(path, "rt") if path.endswith(".gz") else open(path)).read()
    rows = list(csv.reader(io.StringIO(data)))
    for hi, r in enumerate(rows):
        if "Source" in r and any("Instructions Executed" in c for c in r):
            break
    hdr = rows[hi]
    ie = [i for i, c in enumerate(hdr) if c.startswith("Instructions Executed")][0]
    st = [i for i, c in enumerate(hdr) if c.startswith("Warp Stall Sampling (All")][0]
    src = hdr.index("Source")
    recs = []
    for r in rows[hi + 1:]:
        try:
            recs.append((int(r[0], 16), int(r[ie] or 0), int(r[st] or 0), r[src].strip()))
        except (ValueError, IndexError):
            pass
    return recs


def main(path, units=None, top=24, windows=12):
    recs = load(path)
    op, ops = collections.Counter(), collections.Counter()
    for a, n, s, t in recs:
        o = (t.split()[1] if t.startswith("@") else t.split()[0]).split(".")[0]
        op[o] += n
        ops[o] += s
    tot, tots = sum(op.values()), sum(ops.values())
    print(f"{path}: {tot:.3e} warp instructions, {tots} stall samples" +
          (f", {tot / units:.1f} per unit" if units else ""))
    for k, v in op.most_common(top):
        print(f"  {k:12s} {v / tot:6.3f} instr  {ops[k] / max(tots, 1):6.3f} stalls")
    recs.sort()
    W = 64
    win = collections.Counter()
    for i in range(0, len(recs), W):
        chunk = recs[i:i + W]
        win[(chunk[0][0], chunk[-1][0])] = (sum(x[1] for x in chunk), sum(x[2] for x in chunk))
    print("hottest windows (by stall samples):")
    for (a0, a1), (n, s) in sorted(win.items(), key=lambda kv: -kv[1][1])[:windows]:
        print(f"  {a0:#x}-{a1:#x}: {n:.3e} instr, {s} stalls")


if __name__ == "__main__":
    main(sys.argv[1], float(sys.argv[2]) if len(sys.argv) > 2 else None)

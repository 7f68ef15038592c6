"""Hashing ablation: the paper's optimistic / verify / pessimistic scheme with six
hash functions and a 1.4x table (ocl_group_build_paper) against the B200 group build
(ocl_group_build: one pessimistic CAS round, CTA key cache, warp-deduplicated claims, 2x table).

Workload shaped like the paper's Fig. 5(e)/(f) (hash table creation over a 4-byte column, 100 distinct
values; then a sweep of distinct values): n int32 keys, uniform over G distinct values (seeded).
Device time per build (CUDA events, median of --reps after 2 warm-ups), L2 flushed between reps.
"""
import argparse
import json
import os
import statistics
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_journals_pvldb_heimelspmm13_b200 as ocl  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--rows", type=int, default=100_000_000)       # 400 MB of 4-byte keys (Fig. 5 x-axis)
    ap.add_argument("--groups", default="100,1000,10000,100000,1000000,10000000")
    ap.add_argument("--reps", type=int, default=5)
    ap.add_argument("--out", default="")
    args = ap.parse_args()
    dev = torch.device("cuda", 0)
    g = torch.Generator(device=dev).manual_seed(20130826)
    flush = torch.empty(512 << 20, dtype=torch.uint8, device=dev)
    res = []
    for G in [int(x) for x in args.groups.split(",")]:
        keys = torch.randint(0, G, (args.rows,), generator=g, device=dev, dtype=torch.int32)
        line = {"rows": args.rows, "groups": G}
        for scheme in ("b200", "paper"):
            ts = []
            for rep in range(args.reps + 2):
                flush.zero_()
                a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
                a.record()
                gids, kout, ng, st = ocl.group_build([keys], expected_groups=G, out_capacity=G, scheme=scheme)
                b.record()
                torch.cuda.synchronize()
                assert int(st.item()) == 0 and int(ng.item()) <= G, (scheme, G, int(st.item()))
                if rep >= 2:
                    ts.append(a.elapsed_time(b))
            ms = statistics.median(ts)
            line[scheme] = {"ms": ms, "rows_per_s": args.rows / (ms / 1e3), "G_found": int(ng.item())}
        line["paper_over_b200"] = line["paper"]["ms"] / line["b200"]["ms"]
        print(json.dumps(line), flush=True)
        res.append(line)
        del keys
    if args.out:
        with open(args.out, "w") as f:
            json.dump(res, f, indent=1)


if __name__ == "__main__":
    main()

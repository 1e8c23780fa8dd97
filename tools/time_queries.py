"""Per-query K1 device time of prepared plans at SF (repeated), for A/B tuning.

    python tools/time_queries.py [--sf 10] [--queries q2.1,q3.1] [--reps 5]
"""
import argparse
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
sys.path.insert(0, os.path.join(ROOT, "tools"))

import torch  # noqa: E402

import ssbgen  # noqa: E402
from paper_journals_pvldb_chrysogeloskaa19_b200 import hx, ssb  # noqa: E402
from prof_query import device_db  # noqa: E402

ap = argparse.ArgumentParser()
ap.add_argument("--sf", type=float, default=10)
ap.add_argument("--queries", default="all")
ap.add_argument("--reps", type=int, default=5)
ap.add_argument("--join", default="auto", choices=["auto", "hash"], help="HX_OPT_JOIN_LAYOUT")
ap.add_argument("--lo-rows", type=int, default=0, help="first rows of lineorder only (SF1000 dims)")
a = ap.parse_args()
ctx = hx.Context(0)
if a.join == "hash":
    ctx.set_option(hx._hx.HX_OPT_JOIN_LAYOUT, hx._hx.HX_JOIN_HASH)
qs = ssb.QUERIES if a.queries == "all" else a.queries.split(",")
need = set().union(*(ssb.FACT_COLS[q] for q in qs))
dims, fact = device_db(ctx, ssbgen.sizes(a.sf), lo_rows=a.lo_rows or None,
                       lo_cols=[c for c in ssbgen.TABLE_COLS["lineorder"] if ssbgen.COLS[c] in need])
eng = ssb.SsbEngine(ctx, dims, fact)
plans = {q: eng.plan(q) for q in qs}
tot = 0.0
for q in qs:
    ts = []
    for _ in range(a.reps):
        plans[q].enqueue()
        plans[q].rows()
        ts.append(plans[q].hp.k1_time()[0])
    ts.sort()
    tot += ts[len(ts) // 2]
    n = fact.n_rows
    print(f"{q} {n * 4 * len(ssb.FACT_COLS[q]) / (ts[len(ts) // 2] / 1e3) / 1e9:7.0f} GB/s  k1 median {ts[len(ts) // 2]:.4f} ms  min {ts[0]:.4f}  all {' '.join(f'{t:.3f}' for t in ts)}")
print(f"sum of medians {tot:.4f} ms")
for pl in plans.values():
    pl.close()
ctx.close()

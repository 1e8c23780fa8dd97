"""Run selected SSB queries on device-generated SF data (for ncu / nsight captures).

    python tools/prof_query.py --sf 10 --queries q1.1,q2.1 --reps 2
"""
import argparse
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import torch  # noqa: E402

import ssbgen  # noqa: E402
from paper_journals_pvldb_chrysogeloskaa19_b200 import _hx, hx, ssb  # noqa: E402


def device_db(ctx, sz, seed=42, lo_rows=None, lo_cols=None):
    keep, stream = [], torch.cuda.current_stream().cuda_stream

    def table(cols, n):
        spec = []
        for c in cols:
            t = torch.empty(max(n, 1), dtype=torch.int32, device="cuda")
            ssbgen.column_device(seed, sz, c, t.data_ptr(), 0, n, stream)
            keep.append(t)
            spec.append((ssbgen.COLS[c], t.data_ptr(), n))
        return hx.load_columns(ctx, spec, placement=_hx.HX_PLACE_VIEW, keep=keep)

    dims = {t: table(ssbgen.TABLE_COLS[t], ssbgen.table_rows(sz, ssbgen.TABLE_COLS[t][0]))
            for t in ("date", "customer", "supplier", "part")}
    n = sz["n_lineorder"] if lo_rows is None else min(lo_rows, sz["n_lineorder"])
    fact = table(lo_cols or ssbgen.TABLE_COLS["lineorder"], n)
    torch.cuda.synchronize()
    return dims, fact


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--sf", type=float, default=10)
    ap.add_argument("--queries", default="q1.1,q2.1,q3.1,q4.1")
    ap.add_argument("--reps", type=int, default=2)
    ap.add_argument("--lo-rows", type=int, default=0, help="first rows of lineorder only")
    ap.add_argument("--join", default="auto", choices=["auto", "hash"], help="HX_OPT_JOIN_LAYOUT")
    a = ap.parse_args()
    ctx = hx.Context(0, torch.cuda.current_stream().cuda_stream)
    if a.join == "hash":
        ctx.set_option(_hx.HX_OPT_JOIN_LAYOUT, _hx.HX_JOIN_HASH)
    qs = ssb.QUERIES if a.queries == "all" else a.queries.split(",")
    need = set().union(*(ssb.FACT_COLS[q] for q in qs))
    dims, fact = device_db(ctx, ssbgen.sizes(a.sf), lo_rows=a.lo_rows or None,
                           lo_cols=[c for c in ssbgen.TABLE_COLS["lineorder"] if ssbgen.COLS[c] in need])
    eng = ssb.SsbEngine(ctx, dims, fact)
    plans = {q: eng.plan(q) for q in qs}  # the bench's execution path (prepared plans)
    for _ in range(a.reps):
        for q in qs:
            plans[q].enqueue()
            plans[q].rows()
    torch.cuda.synchronize()
    print("ok")


if __name__ == "__main__":
    main()

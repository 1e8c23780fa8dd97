"""SURVEY.md §8(e) "pick by measurement": a replicated dimension build on every GPU (K2 over
the replicated dimension columns) vs build-on-root + ncclBroadcast of the built table.
Times every SSB query's builds at a given SF (device events) and reports the bytes a
broadcast would move (the table's allocation) with the NVLink time at 900 GB/s per direction.

    python tools/build_vs_bcast.py [--sf 1000]
"""
import argparse
import json
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
ap.add_argument("--sf", type=float, default=1000)
a = ap.parse_args()
s = torch.cuda.Stream()
torch.cuda.set_stream(s)
ctx = hx.Context(0, s.cuda_stream)
dims, fact = device_db(ctx, ssbgen.sizes(a.sf), lo_rows=16, lo_cols=["lo_orderdate"])
eng = ssb.SsbEngine(ctx, dims, fact)
out = {"sf": a.sf, "builds": []}
for q in ssb.QUERIES:
    for _, b in ssb.PLANS[q].joins:
        for _ in range(2):  # second run timed (allocator warm)
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record(s)
            ht = eng.build(b)
            e1.record(s)
            torch.cuda.synchronize()
            info = ht.info()
            ms = e0.elapsed_time(e1)
            ht.close()
        slot_bytes = info["n_slots"] * 8
        out["builds"].append({"query": q, "dim": b.table, "rows": dims[b.table].n_rows,
                              "passing": info["n_keys"], "build_ms": round(ms, 4),
                              "bcast_bytes_slots": slot_bytes,
                              "bcast_ms_at_900GBs": round(slot_bytes / 900e9 * 1e3, 4)})
tot_b = sum(x["build_ms"] for x in out["builds"])
tot_c = sum(x["bcast_ms_at_900GBs"] for x in out["builds"])
out["total_build_ms"], out["total_bcast_ms_lower_bound"] = round(tot_b, 3), round(tot_c, 3)
print(json.dumps(out))
ctx.close()

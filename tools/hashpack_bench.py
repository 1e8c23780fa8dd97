"""Throughput of the hash-partitioned join's pieces on one GPU.

    python tools/hashpack_bench.py [--sf 10] [--parts 8]

K3 hash-pack of the lineorder columns a query references (HBM-bound: the key column read
twice, every column read once and written once), and an SSB query with its customer join
hash-partitioned into n parts vs the broadcast join, both through the C-ABI.
"""
import argparse
import json
import os
import sys
import time

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
sys.path.insert(0, os.path.join(ROOT, "tools"))

import torch  # noqa: E402

import ssbgen  # noqa: E402
from paper_journals_pvldb_chrysogeloskaa19_b200 import hx, ssb  # noqa: E402
from prof_query import device_db  # noqa: E402

ap = argparse.ArgumentParser()
ap.add_argument("--sf", type=float, default=10)
ap.add_argument("--parts", type=int, default=8)
ap.add_argument("--reps", type=int, default=5)
ap.add_argument("--no-join", action="store_true", help="time the hash-pack only")
a = ap.parse_args()
s = torch.cuda.Stream()
torch.cuda.set_stream(s)
ctx = hx.Context(0, s.cuda_stream)
cols = ["lo_orderdate", "lo_custkey", "lo_partkey", "lo_suppkey", "lo_revenue", "lo_supplycost"]
dims, fact = device_db(ctx, ssbgen.sizes(a.sf), lo_cols=cols)
n = fact.n_rows
out = {"sf": a.sf, "rows": n, "parts": a.parts, "columns": len(cols)}
best = 1e9
for _ in range(a.reps):
    torch.cuda.synchronize()
    t0 = time.perf_counter()
    t, offs = hx.hash_partition(ctx, fact, ssbgen.COLS["lo_custkey"], a.parts)  # synchronises
    best = min(best, time.perf_counter() - t0)
    t.close()
alg = n * 4 * (2 * len(cols) + 1)  # key read twice, every column read + written once
out["hashpack_ms"] = best * 1e3
out["hashpack_gbps"] = alg / best / 1e9
out["hashpack_alg_bytes"] = alg
eng = ssb.SsbEngine(ctx, dims, fact)
for q in (() if a.no_join else ("q3.1", "q4.1")):
    for mode in ("broadcast", "partitioned"):
        ts = []
        for _ in range(a.reps):
            torch.cuda.synchronize()
            t0 = time.perf_counter()
            if mode == "broadcast":
                eng.run(q)
            else:
                eng.run_hash_partitioned(q, "customer", a.parts)
            ts.append(time.perf_counter() - t0)
        out[f"{q}_{mode}_ms"] = sorted(ts)[len(ts) // 2] * 1e3
print(json.dumps(out))
ctx.close()

"""Where does the e2e step (bench.py's e2e leg) go? H2D loads alone vs loads + 13 queries."""
import os
import sys
import time

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import torch  # noqa: E402

import ssbgen  # noqa: E402
from paper_journals_pvldb_chrysogeloskaa19_b200 import hx, ssb  # noqa: E402

C = ssbgen.COLS
sz = ssbgen.sizes(10)
s = torch.cuda.Stream()
torch.cuda.set_stream(s)
ctx = hx.Context(0, s.cuda_stream)
host = {}
for t in ("lineorder", "date", "customer", "supplier", "part"):
    host[t] = {}
    for c in ssbgen.TABLE_COLS[t]:
        n = ssbgen.table_rows(sz, c)
        buf = torch.empty(n, dtype=torch.int32, pin_memory=True)
        ssbgen.column(42, sz, c, 0, n, out=buf.numpy())
        host[t][c] = (buf, n)


def load(t):
    return hx.load_columns(ctx, [(C[c], b.data_ptr(), n) for c, (b, n) in host[t].items()])


def loads_only():
    tabs = [load(t) for t in ("date", "customer", "supplier", "part", "lineorder")]
    torch.cuda.synchronize()
    for tb in tabs:
        tb.close()


def full(plans=False):
    d = {t: load(t) for t in ("date", "customer", "supplier", "part")}
    f = load("lineorder")
    e = ssb.SsbEngine(ctx, d, f)
    if plans:
        out = [e.run(q) for q in ssb.QUERIES]
    else:
        pend = [e.start(q) for q in ssb.QUERIES]
        out = [e.finish(p) for p in pend]
    for tb in list(d.values()) + [f]:
        tb.close()
    return out


for name, fn in (("loads only", loads_only), ("loads + 13 queries (bench e2e)", full)):
    fn()
    torch.cuda.synchronize()
    ts = []
    for _ in range(5):
        t0 = time.perf_counter()
        fn()
        torch.cuda.synchronize()
        ts.append((time.perf_counter() - t0) * 1e3)
    print(f"{name}: median {sorted(ts)[2]:.2f} ms  {[round(x, 1) for x in ts]}")
ctx.close()

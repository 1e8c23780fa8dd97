"""Where does a bench step go? device time of the captured graph vs the host result reads."""
import sys, time
sys.path.insert(0, '/root/repo'); sys.path.insert(0, '/root/repo/tools')
import torch
import ssbgen
from paper_journals_pvldb_chrysogeloskaa19_b200 import hx, ssb
from prof_query import device_db
s = torch.cuda.Stream()
torch.cuda.set_stream(s)
ctx = hx.Context(0, s.cuda_stream)  # a real stream: torch events bracket the library's work
assert ctx.stream == s.cuda_stream
dims, fact = device_db(ctx, ssbgen.sizes(10))
eng = ssb.SsbEngine(ctx, dims, fact)
plans = {q: eng.plan(q) for q in ssb.QUERIES}
order = [plans[q].hp for q in ssb.QUERIES]
g = hx.capture(ctx, lambda: hx.plans_enqueue(ctx, order))
for _ in range(3):
    g.launch(); [plans[q].rows() for q in ssb.QUERIES]
torch.cuda.synchronize()
# device-only: graph launches back to back
e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
e0.record(s)
for _ in range(20): g.launch()
e1.record(s); torch.cuda.synchronize()
print('graph device ms/step', e0.elapsed_time(e1) / 20)
# with host result reads
t0 = time.perf_counter(); e0.record(s)
for _ in range(20):
    g.launch(); [plans[q].rows() for q in ssb.QUERIES]
e1.record(s); torch.cuda.synchronize()
print('step ms (launch+rows)', e0.elapsed_time(e1) / 20, 'host', (time.perf_counter() - t0) / 20 * 1e3)
# host cost of rows() alone (results already there)
t0 = time.perf_counter()
for _ in range(20): [plans[q].rows() for q in ssb.QUERIES]
print('rows() only ms', (time.perf_counter() - t0) / 20 * 1e3)
t0 = time.perf_counter()
for _ in range(20): [plans[q].hp.result() for q in ssb.QUERIES]
print('hp.result() only ms', (time.perf_counter() - t0) / 20 * 1e3)
k = sum(plans[q].hp.k1_time()[0] for q in ssb.QUERIES)
span = order[0].k1_span(order[-1])
print('K1 sum ms', k, 'K1 span ms', span, 'gaps ms', span - k)
# single launches, each synchronised
ts = []
for _ in range(10):
    torch.cuda.synchronize()
    e0.record(s); g.launch(); e1.record(s); torch.cuda.synchronize()
    ts.append(e0.elapsed_time(e1))
print('single launch + sync ms', sorted(ts)[len(ts)//2], ts[:4])
want = {q: plans[q].rows() for q in ssb.QUERIES}
for _ in range(5): g.launch()
torch.cuda.synchronize()
print('results after back-to-back launches equal:', all(plans[q].rows() == want[q] for q in ssb.QUERIES))
t0 = time.perf_counter()
for _ in range(10):
    g.launch(); torch.cuda.synchronize()
print('launch+sync host ms', (time.perf_counter() - t0) / 10 * 1e3)
for q in ssb.QUERIES:
    plans[q].enqueue(); plans[q].rows()
    print(q, 'k1', round(plans[q].hp.k1_time()[0], 3))

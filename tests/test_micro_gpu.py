"""GPU parity of the §6.4 micro-benchmark pipelines against
oracle/micro.py, through the C-ABI: the pure scan (SUM over one column, K1 without a join)
and the non-partitioned 1:N join (K2 build + K1 probe; COUNT and SUM of the matches).
Bit-exact int64 results; small ragged sizes on both the plain (hash table) and the planned
(direct map) path, and the paper's full size (23 GB probe column, 7.7 MB build column) in
the launch configuration bench.py --workload times."""
import os

import numpy as np
import pytest

import ssbgen
from oracle import micro as omicro

pytestmark = pytest.mark.gpu

torch = pytest.importorskip("torch")
if not torch.cuda.is_available():
    pytest.skip("needs a CUDA GPU", allow_module_level=True)

from paper_journals_pvldb_chrysogeloskaa19_b200 import _hx, hx, micro  # noqa: E402

C = ssbgen.COLS


@pytest.fixture(scope="module")
def ctx():
    c = hx.Context(0)
    yield c
    c.close()


def device_tables(ctx, sz, seed, keep):
    stream = torch.cuda.current_stream().cuda_stream

    def table(cols, n):
        spec = []
        for c in cols:
            t = torch.empty(max(n, 1), dtype=torch.int32, device="cuda")
            ssbgen.column_device(seed, sz, c, t.data_ptr(), 0, n, stream)
            keep.append(t)
            spec.append((C[c], t.data_ptr(), n))
        return hx.load_columns(ctx, spec, placement=_hx.HX_PLACE_VIEW)

    fact = table(["mb_value", "mb_probekey"], sz["n_lineorder"])
    build = table(["mb_buildkey"], sz["n_part"])
    torch.cuda.synchronize()
    return fact, build


def oracle_results(sz, seed, chunk=1 << 27):
    n = sz["n_lineorder"]
    build = ssbgen.column(seed, sz, "mb_buildkey")

    def vals():
        for r in range(0, n, chunk):
            yield ssbgen.column(seed, sz, "mb_value", r, min(chunk, n - r))

    def pairs():
        for r in range(0, n, chunk):
            k = min(chunk, n - r)
            yield ssbgen.column(seed, sz, "mb_probekey", r, k), ssbgen.column(seed, sz, "mb_value", r, k)

    return omicro.sum_column(vals()), omicro.join_count(build, pairs())


@pytest.mark.parametrize("n_rows,n_build", [(0, 10), (1, 1), (5, 3), (2561, 100),
                                            (1_000_003, 5_000), (3_000_001, 200_000)])
def test_micro_parity_small(ctx, n_rows, n_build):
    sz = ssbgen.micro_sizes(n_rows, n_build)
    keep = []
    fact, build = device_tables(ctx, sz, 21, keep)
    want_sum, want_join = oracle_results(sz, 21)
    eng = micro.MicroEngine(ctx, fact, build)
    assert eng.run_sum() == want_sum
    assert eng.run_join() == want_join
    for kind, pl in (("sum", eng.plan_sum()), ("join", eng.plan_join())):
        for _ in range(2):
            pl.enqueue()
            assert eng.plan_value(pl, kind) == (want_sum if kind == "sum" else want_join), kind
        pl.close()


def test_micro_parity_paper_size(ctx):
    """a 23 GB column (5.75 G int32 rows) and a 7.7 MB build column, in
    HBM; prepared plans in a CUDA graph as bench.py --workload sum/join runs them."""
    sz = ssbgen.micro_sizes(ssbgen.MICRO_PAPER_ROWS, ssbgen.MICRO_PAPER_BUILD)
    keep = []
    fact, build = device_tables(ctx, sz, 42, keep)
    eng = micro.MicroEngine(ctx, fact, build)
    ps, pj = eng.plan_sum(), eng.plan_join()
    graph = hx.capture(ctx, lambda: hx.plans_enqueue(ctx, [ps, pj]))
    graph.launch()
    got_sum, got_join = eng.plan_value(ps, "sum"), eng.plan_value(pj, "join")
    want_sum, want_join = oracle_results(sz, 42, chunk=1 << 28)
    assert got_sum == want_sum
    assert got_join == want_join
    graph.close()
    ps.close()
    pj.close()
    del keep

"""The multi-GPU (NCCL) call sequences on ONE GPU: a 1-rank communicator with
HX_FORCE_COLLECTIVES=1 makes libhx issue every collective it would issue with N ranks — the
union-router allreduce / reduce of hx_merge_aggregates, the per-plan allreduces of a
multi-plan step (on the finalize stream, inside a captured CUDA graph), the mem-move broadcast of a built hash table, and the
hash-routing exchange's allgather + send/recv — and the results are checked bit-exactly
against the oracle. A 1-rank allreduce or broadcast is an identity whatever its count, so the
element counts and byte sizes libhx issues are checked separately, from its collective trace
(hx_comm_trace), against values computed independently with numpy. (NCCL refuses two ranks on
one device: the 2-rank NCCL run is tests/test_multigpu_gpu.py, skipped with fewer than 2 GPUs.)
"""
import numpy as np
import pytest

import oracle
import ssbgen

pytestmark = pytest.mark.gpu

torch = pytest.importorskip("torch")
if not torch.cuda.is_available():
    pytest.skip("needs a CUDA GPU", allow_module_level=True)

from paper_journals_pvldb_chrysogeloskaa19_b200 import hx, ssb  # noqa: E402

QUERIES = ssb.QUERIES


@pytest.fixture(scope="module")
def nctx():
    import os
    os.environ["HX_FORCE_COLLECTIVES"] = "1"
    try:
        c = hx.Context(0)
        c.comm_init(1, 0, hx.comm_unique_id())
    finally:
        del os.environ["HX_FORCE_COLLECTIVES"]
    assert c.comm_info() == (0, 1)
    yield c
    c.close()


@pytest.fixture(scope="module")
def db():
    return ssbgen.database(13, ssbgen.sizes(0.02))


@pytest.mark.parametrize("root", [-1, 0])
def test_merge_allreduce_and_reduce(nctx, db, root):
    dims, fact = ssb.load_db_numpy(nctx, db)
    eng = ssb.SsbEngine(nctx, dims, fact)
    for q in QUERIES:
        assert eng.finish(eng.start(q), root) == oracle.run_query(q, db), (q, root)


def test_plans_allreduce_in_graph(nctx, db):
    """Each plan's union-router allreduce on the finalize stream, inside a captured graph."""
    dims, fact = ssb.load_db_numpy(nctx, db)
    eng = ssb.SsbEngine(nctx, dims, fact)
    plans = {q: eng.plan(q) for q in QUERIES}
    order = [plans[q].hp for q in QUERIES]
    want = {q: oracle.run_query(q, db) for q in QUERIES}
    hx.plans_enqueue(nctx, order)
    for q in QUERIES:
        assert plans[q].rows() == want[q], q
    graph = hx.capture(nctx, lambda: hx.plans_enqueue(nctx, order))
    for _ in range(2):
        graph.launch()
        for q in QUERIES:
            assert plans[q].rows() == want[q], q
    graph.close()
    for pl in plans.values():
        pl.close()


def test_ht_broadcast(nctx, db):
    """Build on the root, broadcast (mem-move multicast), probe with the broadcast tables."""
    dims, fact = ssb.load_db_numpy(nctx, db)
    eng = ssb.SsbEngine(nctx, dims, fact)
    for q in ("q2.1", "q3.2", "q4.3"):
        plan = ssb.PLANS[q]
        hts = [eng.build(b) for _, b in plan.joins]
        for t in hts:
            t.broadcast(0)
        agg = hx.pipeline_probe_agg(nctx, fact, eng.shape(plan), hts)
        assert eng.finish(ssb.Pending(plan, hts, agg)) == oracle.run_query(q, db), q


def test_hash_routing_exchange(nctx, db):
    dims, fact = ssb.load_db_numpy(nctx, db)
    eng = ssb.SsbEngine(nctx, dims, fact)
    for q, dim in (("q2.1", "part"), ("q3.1", "customer"), ("q4.3", "supplier")):
        assert eng.run_hash_routed(q, dim) == oracle.run_query(q, db), (q, dim)


def test_hash_routing_exchange_partitioned_dimension(nctx, db):
    """Both join inputs through the hash-routing router: the dimension is NOT replicated for
    the routed join (dim_local = this rank's rows, here all of them), so it is hash-packed
    and exchanged like lineorder."""
    dims, fact = ssb.load_db_numpy(nctx, db)
    eng = ssb.SsbEngine(nctx, dims, fact)
    for q, dim in (("q2.1", "part"), ("q3.1", "customer"), ("q4.3", "supplier"), ("q4.1", "date")):
        local = hx.load_numpy(nctx, {ssbgen.COLS[c]: v for c, v in db[dim].items()})
        nctx.comm_trace(reset=True)
        assert eng.run_hash_routed(q, dim, dim_local=local) == oracle.run_query(q, db), (q, dim)
        ops = [r["op"] for r in nctx.comm_trace(reset=True)]
        assert ops.count("allgather") == 2, ops  # lineorder's and the dimension's part sizes
        local.close()


# ---- the sizes of the collectives, from the collective trace (hx_comm_trace) ----------------
# A 1-rank allreduce / broadcast is an identity whatever its count, so the counts libhx
# issues are checked here against values computed independently from the generated tables
# with numpy, following the query texts: a grouping dimension contributes the
# number of distinct group codes among its rows that pass the dimension's filter (the dense
# ranks, R17), and the group array is their product.
from ssb_groups import n_groups as _groups  # noqa: E402


def test_trace_merge_counts(nctx, db):
    """hx_merge_aggregates: an error-status allreduce (2 int64) on every rank, then the sums
    and the counts, n_groups elements each (allreduce, or reduce to the root)."""
    dims, fact = ssb.load_db_numpy(nctx, db)
    eng = ssb.SsbEngine(nctx, dims, fact)
    for root in (-1, 0):
        for q in QUERIES:
            nctx.comm_trace(reset=True)
            eng.finish(eng.start(q), root)
            tr = nctx.comm_trace(reset=True)
            ng = _groups(db, q)
            op = "allreduce" if root < 0 else "reduce"
            assert [(r["op"], r["count"], r["elem_bytes"]) for r in tr] == [
                ("allreduce", 2, 8), (op, ng, 8), (op, ng, 8)], (q, root, tr)


def test_trace_plan_allreduce_counts(nctx, db):
    """A multi-plan step: one union-router allreduce per plan over its adjacent {sums, counts}
    arrays, 2 x n_groups uint64 elements, issued in plan order."""
    dims, fact = ssb.load_db_numpy(nctx, db)
    eng = ssb.SsbEngine(nctx, dims, fact)
    plans = {q: eng.plan(q) for q in QUERIES}
    nctx.comm_trace(reset=True)
    hx.plans_enqueue(nctx, [plans[q].hp for q in QUERIES])
    for q in QUERIES:
        plans[q].rows()
    tr = nctx.comm_trace(reset=True)
    assert [(r["op"], r["count"], r["elem_bytes"]) for r in tr] == [
        ("allreduce", 2 * _groups(db, q), 8) for q in QUERIES]
    for pl in plans.values():
        pl.close()


def _next_pow2(x):
    return 1 << max(0, int(x - 1).bit_length())


def test_trace_ht_broadcast_sizes(nctx, db):
    """hx_ht_broadcast moves the header + rank maps, then the slots in use (8 B each, a power
    of two >= 4 per passing key, at least 16) and the Bloom filter (a power of two of 32-bit
    words >= 16 bits per passing key), from the root."""
    dims, fact = ssb.load_db_numpy(nctx, db)
    eng = ssb.SsbEngine(nctx, dims, fact)
    c, s = db["customer"], db["supplier"]
    cases = [("q3.1", "customer", int(np.sum(c["c_region"] == 2))),     # ASIA
             ("q3.2", "supplier", int(np.sum(s["s_nation"] == 23))),    # UNITED STATES
             ("q4.1", "customer", int(np.sum(c["c_region"] == 1)))]     # AMERICA
    for q, dim, n_pass in cases:
        plan = ssb.PLANS[q]
        (b,) = [b for _, b in plan.joins if b.table == dim]
        t = eng.build(b)
        nctx.comm_trace(reset=True)
        t.broadcast(0)
        tr = nctx.comm_trace(reset=True)
        assert [r["op"] for r in tr] == ["broadcast"] * 3 and all(r["root_or_peer"] == 0 for r in tr)
        assert tr[0]["count"] % 256 == 0
        assert tr[1]["count"] == 8 * max(16, _next_pow2(4 * n_pass)), (q, dim, tr)
        assert tr[2]["count"] == 4 * max(1, _next_pow2(16 * n_pass) // 32), (q, dim, tr)
        assert t.info()["n_keys"] == n_pass
        t.close()

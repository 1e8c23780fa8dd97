"""The multi-GPU (NCCL) call sequences on ONE GPU: a 1-rank communicator with
HX_FORCE_COLLECTIVES=1 makes libhx issue every collective it would issue with N ranks — the
union-router allreduce / reduce of hx_merge_aggregates, the per-plan allreduces of a
multi-plan step (on the finalize stream, inside a captured CUDA graph), the mem-move broadcast of a built hash table, and the
hash-routing exchange's allgather + send/recv — so their buffers, sizes and ordering are
checked bit-exactly against the oracle. (NCCL refuses two ranks on one device; the N-rank
data flow is covered by the gloo tests in test_hx_cpu.py.)
"""
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

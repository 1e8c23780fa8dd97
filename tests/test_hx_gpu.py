"""GPU parity of libhx against the oracle, through the C-ABI (ctypes binding).

Bar: bit-exact — the set of (group codes, int64 SUM, int64 COUNT) rows
and their ORDER BY order — for all 13 SSB queries. Inputs are seeded (ssbgen / ssb_tiny).
"""
import numpy as np
import pytest

import oracle
import ssbgen
from ssb_tiny import tiny_db

pytestmark = pytest.mark.gpu

torch = pytest.importorskip("torch")
if not torch.cuda.is_available():
    pytest.skip("needs a CUDA GPU", allow_module_level=True)

from paper_journals_pvldb_chrysogeloskaa19_b200 import _hx, hx, ssb  # noqa: E402

QUERIES = ssb.QUERIES
C = ssbgen.COLS


@pytest.fixture(scope="module")
def ctx():
    c = hx.Context(0)
    yield c
    c.close()


def run_all(ctx, db, queries=QUERIES):
    dims, fact = ssb.load_db_numpy(ctx, db)
    eng = ssb.SsbEngine(ctx, dims, fact)
    return {q: eng.run(q) for q in queries}


# ---- small SSB databases: several tiles and a ragged tail ------------------------------
@pytest.mark.parametrize("sf,seed", [(0.01, 42), (0.05, 7)])
def test_parity_small_sf(ctx, sf, seed):
    db = ssbgen.database(seed, ssbgen.sizes(sf))
    got = run_all(ctx, db)
    for q in QUERIES:
        assert got[q] == oracle.run_query(q, db), q


@pytest.fixture(scope="module")
def sf005():
    db = ssbgen.database(7, ssbgen.sizes(0.05))
    return db, {q: oracle.run_query(q, db) for q in QUERIES}


@pytest.mark.parametrize("seq_min", [None, "0", "99"])
@pytest.mark.parametrize("layout", ["auto", "hash"])
@pytest.mark.parametrize("warps", ["20", "26"])
def test_k1_instances_and_probe_schedules(sf005, monkeypatch, warps, layout, seq_min):
    """Both consumer-warp instances (HX_K1_W), the direct maps and the hash tables
    (HX_OPT_JOIN_LAYOUT, prepared plans), and the hash-table stage-C schedules: the planner's choice, every
    plan probing its likeliest-miss join alone first (HX_HT_FIRST_MIN=0), and all joins in one
    round trip (=99) — all bit-exact against the oracle over 30 K1 tiles plus a ragged tail."""
    db, want = sf005
    monkeypatch.setenv("HX_K1_W", warps)
    if seq_min is not None:
        monkeypatch.setenv("HX_HT_FIRST_MIN", seq_min)
    c = hx.Context(0)
    try:
        if layout == "hash":
            c.set_option(_hx.HX_OPT_JOIN_LAYOUT, _hx.HX_JOIN_HASH)
        dims, fact = ssb.load_db_numpy(c, db)
        eng = ssb.SsbEngine(c, dims, fact)
        for q in QUERIES:  # prepared plans (the bench's path; they pick direct maps under auto)
            pl = eng.plan(q)
            pl.enqueue()
            assert pl.rows() == want[q], (q, warps, layout, seq_min)
            pl.close()
        for q in QUERIES:  # the unprepared calls (hash tables)
            assert eng.run(q) == want[q], (q, warps, layout, seq_min)
    finally:
        c.close()


@pytest.mark.parametrize("rule", ["1", "2"])
def test_hash_plans_join_probed_in_place(sf005, monkeypatch, capfd, rule):
    """Hash-table plans that move a selective unfiltered join to the front of the probe order
    so that stage B probes it in place after the stage-F Bloom filter (HX_HT_INPLACE; with
    HX_HT_FIRST_MIN=0 every multi-join plan qualifies for rule 1): under rule 1 the rotation must
    happen for some plan (HX_DEBUG prints it); every query stays bit-exact against the oracle."""
    db, want = sf005
    monkeypatch.setenv("HX_HT_INPLACE", rule)
    monkeypatch.setenv("HX_HT_FIRST_MIN", "0")
    monkeypatch.setenv("HX_DEBUG", "1")
    c = hx.Context(0)
    try:
        c.set_option(_hx.HX_OPT_JOIN_LAYOUT, _hx.HX_JOIN_HASH)
        dims, fact = ssb.load_db_numpy(c, db)
        eng = ssb.SsbEngine(c, dims, fact)
        for q in QUERIES:
            pl = eng.plan(q)
            pl.enqueue()
            assert pl.rows() == want[q], (q, rule)
            pl.close()
    finally:
        c.close()
    err = capfd.readouterr().err
    moved = [ln for ln in err.splitlines() if "inplace=" in ln and "inplace=-1" not in ln]
    if rule == "1":  # (rule 2 needs a selective join too large for a Bloom filter: SF100-sized)
        assert moved, "no plan probed a moved join in place"


def test_parity_handcrafted(ctx, handcrafted):
    db, expect = handcrafted
    got = run_all(ctx, db)
    for q in QUERIES:
        assert got[q] == expect[q], q


@pytest.mark.parametrize("seed", [1, 2, 3])
def test_parity_tiny_skewed(ctx, seed):
    """Missing FKs, boundary dates, dense group domains (every query non-empty)."""
    db = tiny_db(seed, n_lo=20011)
    got = run_all(ctx, db)
    for q in QUERIES:
        assert got[q] == oracle.run_query(q, db), q


@pytest.mark.parametrize("n_lo", [0, 1, 3, 4, 5, 2047, 2048, 2049, 4096 * 3 + 1])
def test_ragged_sizes(ctx, n_lo):
    db = tiny_db(11, n_lo=max(n_lo, 1))
    if n_lo == 0:
        db["lineorder"] = {k: v[:0] for k, v in db["lineorder"].items()}
    got = run_all(ctx, db)
    for q in QUERIES:
        assert got[q] == oracle.run_query(q, db), (q, n_lo)


def test_duplicate_dimension_key_is_reported(ctx):
    db = tiny_db(3, dup_keys=True)
    dims, fact = ssb.load_db_numpy(ctx, db)
    eng = ssb.SsbEngine(ctx, dims, fact)
    with pytest.raises(_hx.HxError) as ei:
        eng.run("q4.1")
    assert ei.value.code == _hx.HX_EDUPKEY


# ---- hash-table self-check (K2) ------------------------------------------------------------
def test_hash_table_contents(ctx):
    sz = ssbgen.sizes(0.1)
    db = ssbgen.database(5, sz)
    dims, _ = ssb.load_db_numpy(ctx, {**db, "lineorder": {k: v[:1] for k, v in db["lineorder"].items()}})
    cust = db["customer"]
    ht = hx.build_dim_ht(ctx, dims["customer"], C["c_custkey"],
                         [hx.pred(C["c_region"], 1, 1)], C["c_nation"], 0, 24)
    info = ht.info(with_codes=True)
    passing = cust["c_region"] == 1
    assert info["n_keys"] == int(passing.sum())
    assert info["n_slots"] >= 2 * info["n_keys"] and info["n_slots"] & (info["n_slots"] - 1) == 0
    assert info["rank_to_code"] == sorted(set(cust["c_nation"][passing].tolist()))
    # probe every key through a one-join pipeline: COUNT per nation rank == dimension counts
    keys = cust["c_custkey"]
    fact = hx.load_numpy(ctx, {C["lo_custkey"]: keys, C["lo_revenue"]: np.ones_like(keys)})
    shape = hx.query_shape(joins=[(C["lo_custkey"], 0)], agg_a=C["lo_revenue"], gdims=[0])
    agg = hx.pipeline_probe_agg(ctx, fact, shape, [ht])
    k, s, c = hx.merge_aggregates(ctx, agg)
    want = {n: int((cust["c_nation"][passing] == n).sum()) for n in info["rank_to_code"]}
    assert {int(a): int(b) for a, b in zip(k[:, 0], c)} == want
    assert int(c.sum()) == int(passing.sum())  # every passing key hit, every other key missed


# ---- router / partition invariance (fake multi-GPU on one device) ----------------------
@pytest.mark.parametrize("n_parts,block_rows,policy", [(2, 4097, 0), (3, 1000, 1), (4, 1 << 22, 0)])
def test_partition_invariance(ctx, n_parts, block_rows, policy):
    db = ssbgen.database(9, ssbgen.sizes(0.02))
    n = len(db["lineorder"]["lo_orderdate"])
    part = hx.router_partition(n, n_parts, block_rows, policy)
    blocks = part.blocks()
    assert sum(e - b for b, e, _ in blocks) == n
    assert sum(part.rows(i) for i in range(n_parts)) == n
    dims, _ = ssb.load_db_numpy(ctx, {**db, "lineorder": {k: v[:1] for k, v in db["lineorder"].items()}})
    facts = [hx.load_numpy(ctx, {C[c]: v for c, v in db["lineorder"].items()}, part, i)
             for i in range(n_parts)]
    eng = ssb.SsbEngine(ctx, dims, facts[0])
    for q in QUERIES:
        plan = ssb.PLANS[q]
        hts = [eng.build(b) for _, b in plan.joins]
        shape = eng.shape(plan)
        agg = hx.pipeline_probe_agg(ctx, facts[0], shape, hts)
        for f in facts[1:]:
            hx.pipeline_probe_agg_into(ctx, f, shape, hts, agg)
        keys, sums, cnts = hx.merge_aggregates(ctx, agg)
        rows = ssb.order_by(plan, [tuple(int(x) for x in keys[i]) + (int(sums[i]), int(cnts[i]))
                                   for i in range(len(sums))])
        assert rows == oracle.run_query(q, db), (q, n_parts)


@pytest.mark.parametrize("offset", [1, 2, 3, 5])
def test_misaligned_views(ctx, offset):
    """Slices at a row offset are not 16-byte aligned: head rows take the direct path."""
    db = ssbgen.database(4, ssbgen.sizes(0.01))
    dims, fact = ssb.load_db_numpy(ctx, db)
    n = fact.n_rows
    sl = fact.slice(offset, n - 7)
    eng = ssb.SsbEngine(ctx, dims, sl)
    for q in QUERIES:
        assert eng.run(q) == oracle.run_query(q, db, offset, n - 7), q


@pytest.mark.parametrize("seg_tiles,offset", [(1, 0), (3, 3), (7, 1)])
def test_k1_launch_segments(ctx, monkeypatch, seg_tiles, offset):
    """A fact table beyond 32-bit row offsets (one GPU's SF1000 partition, 6e9 rows) runs as
    consecutive K1 launches over whole-tile segments accumulating into the same groups.
    HX_K1_SEG_TILES shrinks the segment to 1-7 tiles so that SF0.05 (117 tiles, a ragged
    tail, misaligned head rows) crosses dozens of boundaries; gathered measures included."""
    monkeypatch.setenv("HX_K1_SEG_TILES", str(seg_tiles))
    db = ssbgen.database(9, ssbgen.sizes(0.05))
    dims, fact = ssb.load_db_numpy(ctx, db)
    n = fact.n_rows
    sl = fact.slice(offset, n) if offset else fact
    eng = ssb.SsbEngine(ctx, dims, sl)
    for q in QUERIES:
        want = oracle.run_query(q, db, offset, n)
        assert eng.run(q) == want, q
        pl = eng.plan(q)
        pl.enqueue()
        assert pl.rows() == want, q
        pl.close()


@pytest.mark.parametrize("seed", [3, 8])
def test_plans_and_graph_replay(ctx, seed):
    """Prepared plans (device finalize) and a CUDA graph of all 13 executions, replayed
    twice, give the oracle's rows every time."""
    db = tiny_db(seed, n_lo=30001)
    dims, fact = ssb.load_db_numpy(ctx, db)
    eng = ssb.SsbEngine(ctx, dims, fact)
    plans = {q: eng.plan(q) for q in QUERIES}
    want = {q: oracle.run_query(q, db) for q in QUERIES}
    for q, pl in plans.items():  # plain enqueue
        pl.enqueue()
        assert pl.rows() == want[q], q
    graph = hx.capture(ctx, lambda: [pl.enqueue() for pl in plans.values()])
    for _ in range(2):
        graph.launch()
        for q, pl in plans.items():
            assert pl.rows() == want[q], q
    # one step: every build first (overlapping earlier pipelines), then the pipelines
    ordered = [pl.hp for pl in plans.values()]
    hx.plans_enqueue(ctx, ordered)
    for q, pl in plans.items():
        assert pl.rows() == want[q], q
    graph2 = hx.capture(ctx, lambda: hx.plans_enqueue(ctx, ordered))
    graph2.launch()
    for q, pl in plans.items():
        assert pl.rows() == want[q], q
    graph2.close()
    ms, nbytes = plans["q2.1"].hp.k1_time()
    # streamed columns (4 B per row each), or 3 streamed + lo_revenue gathered for the rows
    # that passed every join (one 32-byte sector each)
    n_pass = sum(r[-1] for r in want["q2.1"])
    assert ms > 0 and nbytes in (30001 * 16, 30001 * 12 + 32 * n_pass)
    graph.close()
    for pl in plans.values():
        pl.close()


@pytest.mark.parametrize("sf", [0.002, 0.4])
def test_host_resident_streaming(ctx, sf):
    """§8(a) a8: lineorder in pinned host memory, streamed over PCIe in 2^21-row blocks
    (SF0.4 = 2.4 M rows: two blocks, the second partial), plain and planned paths."""
    db = ssbgen.database(13, ssbgen.sizes(sf))
    pin = lambda n: torch.empty(n, dtype=torch.int32, pin_memory=True)
    dims, fact = ssb.load_db_host_resident(ctx, db, pin)
    eng = ssb.SsbEngine(ctx, dims, fact)
    for q in ("q1.1", "q2.1", "q3.1", "q4.1", "q4.3"):
        want = oracle.run_query(q, db)
        assert eng.run(q) == want, q
        pl = eng.plan(q)
        pl.enqueue()
        assert pl.rows() == want, q
        pl.enqueue()  # re-execution reuses the staging ring
        assert pl.rows() == want, q
        pl.close()


@pytest.mark.parametrize("sf", [0.002, 0.4])
def test_host_mapped_zero_copy(ctx, sf):
    """§8(f) NEXT-3: lineorder in mapped pinned host memory read in place by K1's bulk copies
    through UVA (HX_PLACE_HOST_MAPPED), plain and planned paths, every query."""
    db = ssbgen.database(17, ssbgen.sizes(sf))
    pin = lambda n: torch.empty(n, dtype=torch.int32, pin_memory=True)
    dims, fact = ssb.load_db_host_resident(ctx, db, pin, _hx.HX_PLACE_HOST_MAPPED)
    eng = ssb.SsbEngine(ctx, dims, fact)
    for q in QUERIES:
        want = oracle.run_query(q, db)
        assert eng.run(q) == want, q
        pl = eng.plan(q)
        pl.enqueue()
        assert pl.rows() == want, q
        pl.close()


def test_host_mapped_rejects_device_memory(ctx):
    t = torch.zeros(16, dtype=torch.int32, device="cuda")
    with pytest.raises(_hx.HxError):
        hx.load_columns(ctx, [(C["lo_orderdate"], t.data_ptr(), 16)],
                        placement=_hx.HX_PLACE_HOST_MAPPED)


@pytest.mark.parametrize("sf", [10, 100])
def test_parity_full_size_bench_configuration(ctx, sf):
    """BASELINE.json configs[1] (SF10, 60 M lineorder rows) and configs[2]'s 1-GPU leg (SF100,
    600 M rows) at full size in the launch configuration bench.py times: columns generated in
    HBM, prepared plans, one CUDA graph for the 13 queries (hx_plans_enqueue). Bit-exact
    against the oracle run over the host's cores in row ranges merged by summation (the
    union-router merge)."""
    import os
    sz = ssbgen.sizes(sf)
    stream = torch.cuda.current_stream().cuda_stream
    keep = []

    def table(cols, n):
        spec = []
        for c in cols:
            t = torch.empty(n, dtype=torch.int32, device="cuda")
            ssbgen.column_device(42, sz, c, t.data_ptr(), 0, n, stream)
            keep.append(t)
            spec.append((C[c], t.data_ptr(), n))
        return hx.load_columns(ctx, spec, placement=_hx.HX_PLACE_VIEW, keep=keep)

    dims = {t: table(ssbgen.TABLE_COLS[t], ssbgen.table_rows(sz, ssbgen.TABLE_COLS[t][0]))
            for t in ("date", "customer", "supplier", "part")}
    fact = table(ssbgen.TABLE_COLS["lineorder"], sz["n_lineorder"])
    torch.cuda.synchronize()
    eng = ssb.SsbEngine(ctx, dims, fact)
    plans = {q: eng.plan(q) for q in QUERIES}
    order = [plans[q].hp for q in QUERIES]
    graph = hx.capture(ctx, lambda: hx.plans_enqueue(ctx, order))
    graph.launch()
    got = {q: plans[q].rows() for q in QUERIES}
    db = ssbgen.database(42, sz)
    for q in QUERIES:
        want = oracle.run_query_ranges(q, db, os.cpu_count() or 8)
        assert {tuple(r[:-2]): (r[-2], r[-1]) for r in got[q]} == want, q
        plan = ssb.PLANS[q]
        assert got[q] == ssb.order_by(plan, got[q]), q  # ORDER BY holds
    graph.close()
    for pl in plans.values():
        pl.close()


@pytest.mark.parametrize("sf", [0.02, 100])
def test_device_generated_columns_match_host(ctx, sf):
    """ssbgen's device fill is bit-identical to the host fill (the bench's inputs): every
    column of every dimension, and a 4 M-row slice of every lineorder column."""
    sz = ssbgen.sizes(sf)
    for col in ssbgen.COLS:
        n = min(ssbgen.table_rows(sz, col), 4_000_000)
        r0 = ssbgen.table_rows(sz, col) - n  # the tail of the table (largest row counters)
        t = torch.empty(n, dtype=torch.int32, device="cuda")
        ssbgen.column_device(42, sz, col, t.data_ptr(), r0, n, torch.cuda.current_stream().cuda_stream)
        torch.cuda.synchronize()
        assert np.array_equal(t.cpu().numpy(), ssbgen.column(42, sz, col, r0, n)), col


# ---- direct maps (plans over dense keys, R20) vs hash tables -----------------------
def _remap_keys(db, mul, off):
    """Apply k -> k*mul + off to every customer / supplier / part key and its foreign key
    (a bijection: the query results are unchanged); mul=1, off=0 keeps the dense keys."""
    out = {t: dict(cols) for t, cols in db.items()}
    for dim, pk, fk in (("customer", "c_custkey", "lo_custkey"), ("supplier", "s_suppkey", "lo_suppkey"),
                        ("part", "p_partkey", "lo_partkey")):
        for t, c in ((dim, pk), ("lineorder", fk)):
            v = out[t][c].astype(np.int64) * mul + off
            assert v.min() >= -(1 << 31) and v.max() < (1 << 31) and not (v == -1).any()
            out[t][c] = v.astype(np.int32)
    return out


@pytest.mark.parametrize("no_gather", [False, True])
@pytest.mark.parametrize("no_dm", [False, True])
@pytest.mark.parametrize("mul,off", [(1, 0), (7919, -500000), (1 << 25, -(1 << 30))])
def test_plans_key_encodings(ctx, monkeypatch, mul, off, no_dm, no_gather):
    """Plans choose a direct map (dense or moderately sparse keys, negative keys included) or
    the hash table (span >= 2^27, or HX_NO_DM=1), and gather the measure columns of the
    passing rows or stream them (HX_NO_GATHER=1); every combination gives the oracle's rows."""
    if no_dm:
        monkeypatch.setenv("HX_NO_DM", "1")
    if no_gather:
        monkeypatch.setenv("HX_NO_GATHER", "1")
    db = _remap_keys(tiny_db(5, n_lo=20011), mul, off)
    dims, fact = ssb.load_db_numpy(ctx, db)
    eng = ssb.SsbEngine(ctx, dims, fact)
    plans = {q: eng.plan(q) for q in QUERIES}
    order = [plans[q].hp for q in QUERIES]
    graph = hx.capture(ctx, lambda: hx.plans_enqueue(ctx, order))
    for _ in range(2):
        graph.launch()
        for q in QUERIES:
            assert plans[q].rows() == oracle.run_query(q, db), (q, mul, no_dm)
    graph.close()
    for pl in plans.values():
        pl.close()


def test_plan_detects_changed_dimension(ctx):
    """A direct map is sized from the passing keys a plan observed at creation: if the
    dimension (a VIEW) later gains a passing key outside that range the execution reports
    HX_ECAPACITY instead of writing outside the map."""
    db = tiny_db(6, n_lo=5000)
    keep = []

    def view(cols):
        spec = []
        for c, v in cols.items():
            t = torch.from_numpy(np.ascontiguousarray(v)).cuda()
            keep.append(t)
            spec.append((C[c], t.data_ptr(), len(v)))
        return hx.load_columns(ctx, spec, placement=_hx.HX_PLACE_VIEW, keep=keep), keep[-len(cols):]

    dims, tensors = {}, {}
    for t in ("date", "customer", "supplier", "part"):
        dims[t], ts = view(db[t])
        tensors[t] = dict(zip(db[t].keys(), ts))
    fact, _ = view(db["lineorder"])
    torch.cuda.synchronize()
    eng = ssb.SsbEngine(ctx, dims, fact)
    pl = eng.plan("q3.1")  # customer c_region = ASIA, grouped by c_nation
    pl.enqueue()
    assert pl.rows() == oracle.run_query("q3.1", db)
    cust = tensors["customer"]
    asia = int(np.flatnonzero(db["customer"]["c_region"] == 2)[0])
    cust["c_custkey"][asia] = 1 << 30  # a passing key far outside the observed range
    torch.cuda.synchronize()
    pl.enqueue()
    with pytest.raises(_hx.HxError) as ei:
        pl.rows()
    assert ei.value.code == _hx.HX_ECAPACITY
    pl.close()


# ---- probe-order invariance (the join order cannot change the result) --------
@pytest.mark.parametrize("seed", [0, 1])
def test_probe_order_permutations(ctx, seed):
    """Every permutation of a query's joins (probe order = array order; the group key keeps
    the SELECT order through gdim_join) gives the oracle's rows."""
    import itertools
    db = ssbgen.database(21 + seed, ssbgen.sizes(0.01))
    dims, fact = ssb.load_db_numpy(ctx, db)
    eng = ssb.SsbEngine(ctx, dims, fact)
    rng = np.random.default_rng(seed)
    for q in ("q2.1", "q3.1", "q3.3", "q4.1", "q4.2", "q4.3"):
        plan = ssb.PLANS[q]
        want = oracle.run_query(q, db)
        hts = [eng.build(b) for _, b in plan.joins]
        perms = list(itertools.permutations(range(len(plan.joins))))
        for perm in [perms[i] for i in rng.choice(len(perms), size=min(6, len(perms)), replace=False)]:
            pos = {j: i for i, j in enumerate(perm)}  # original join j probed at position pos[j]
            shape = hx.query_shape(
                preds=[ssb._hx_pred(t) for t in plan.fact_preds],
                joins=[(C[plan.joins[j][0]], j) for j in perm],
                agg_op=plan.agg[0], agg_a=C[plan.agg[1]], agg_b=C[plan.agg[2]],
                gdims=[pos[g] for g in plan.gdims])
            agg = hx.pipeline_probe_agg(ctx, fact, shape, hts)
            keys, sums, cnts = hx.merge_aggregates(ctx, agg)
            rows = ssb.order_by(plan, [tuple(int(x) for x in keys[i]) + (int(sums[i]), int(cnts[i]))
                                       for i in range(len(sums))])
            agg.close()
            assert rows == want, (q, perm)
        for t in hts:
            t.close()


def test_table_write_read_and_plans_on_refreshed_data(ctx):
    """hx_table_write refreshes the HBM columns under prepared plans (the serving pattern of
    bench.py's e2e leg): rewrite every lineorder column from host memory (first with another
    seed's lineorder rows, then the original ones) and the same plan returns each database's
    oracle rows; hx_table_read returns what was written."""
    db1 = ssbgen.database(31, ssbgen.sizes(0.01))
    db2 = ssbgen.database(32, ssbgen.sizes(0.01))
    dims, fact = ssb.load_db_numpy(ctx, db1)
    eng = ssb.SsbEngine(ctx, dims, fact)
    plans = {q: eng.plan(q) for q in ("q1.1", "q2.1", "q4.3")}
    # (the dimension tables stay db1's: the second database contributes its lineorder rows)
    for db in (dict(db1, lineorder=db2["lineorder"]), db1):
        keep = []
        for c, v in db["lineorder"].items():
            v = np.ascontiguousarray(v, dtype=np.int32)
            keep.append(v)
            fact.write(C[c], v.ctypes.data, len(v))
        torch.cuda.synchronize()
        for c, v in db["lineorder"].items():
            assert np.array_equal(fact.read(C[c]), v), c
        for q, pl in plans.items():
            pl.enqueue()
            assert pl.rows() == oracle.run_query(q, db), q
    for pl in plans.values():
        pl.close()


@pytest.mark.parametrize("case", ["no_passing_part", "empty_supplier", "empty_date"])
def test_degenerate_dimensions(ctx, case):
    """A dimension filter that passes nothing, and empty dimension tables: every dependent
    query yields the oracle's (empty, or count-0) result — plain calls and prepared plans."""
    db = tiny_db(29, n_lo=9001)
    db = {t: dict(cols) for t, cols in db.items()}
    if case == "no_passing_part":
        db["part"]["p_category"] = np.full_like(db["part"]["p_category"], 24)
        db["part"]["p_brand1"] = np.full_like(db["part"]["p_brand1"], 24 * 40)
        db["part"]["p_mfgr"] = np.full_like(db["part"]["p_mfgr"], 4)
    else:
        t = case.split("_")[1]
        db[t] = {k: v[:0] for k, v in db[t].items()}
    dims, fact = ssb.load_db_numpy(ctx, db)
    eng = ssb.SsbEngine(ctx, dims, fact)
    for q in QUERIES:
        want = oracle.run_query(q, db)
        assert eng.run(q) == want, (case, q)
        pl = eng.plan(q)
        pl.enqueue()
        assert pl.rows() == want, (case, q)
        pl.close()


# ---- an empty BETWEEN on lineorder (lo > hi) selects nothing, with and without joins ------
@pytest.mark.parametrize("q", ["q1.1", "q2.1", "q4.3"])
def test_empty_fact_range_selects_nothing(ctx, q):
    """SQL `x BETWEEN 30 AND 20` is empty. K1 tests ranges with one unsigned compare, so
    k1_setup must compile lo > hi to always-false (it used to wrap and pass
    nearly every row of a pipeline with joins)."""
    import dataclasses
    db = tiny_db(5, n_lo=20011)
    dims, fact = ssb.load_db_numpy(ctx, db)
    eng = ssb.SsbEngine(ctx, dims, fact)
    base = ssb.PLANS[q]
    plan = dataclasses.replace(base, fact_preds=list(base.fact_preds) + [("lo_quantity", 30, 20)])
    hts = [eng.build(b) for _, b in plan.joins]
    agg = hx.pipeline_probe_agg(ctx, fact, eng.shape(plan), hts)
    rows = eng.finish(ssb.Pending(plan, hts, agg))
    # ungrouped: one row, count 0 (SQL NULL sum, R7); grouped: no group at all
    assert rows == ([(0, 0)] if not plan.gdims else []), (q, rows[:3])


@pytest.mark.parametrize("table,col", [("customer", "c_custkey"), ("date", "d_datekey")])
def test_reserved_key_minus_one_rejected(ctx, table, col):
    """Key -1 is the empty-slot marker (R18): a dimension holding it is refused
    with HX_EINVAL by the plain calls and by plan creation, never silently mis-joined."""
    db = tiny_db(4, n_lo=4097)
    db[table][col] = db[table][col].copy()
    db[table][col][3] = -1
    if table == "customer":  # the row must pass Q3.1's customer filter (c_region = ASIA)
        db[table]["c_region"] = db[table]["c_region"].copy()
        db[table]["c_region"][3] = 2
    dims, fact = ssb.load_db_numpy(ctx, db)
    eng = ssb.SsbEngine(ctx, dims, fact)
    q = "q3.1"
    with pytest.raises(_hx.HxError) as ei:
        eng.run(q)
    assert ei.value.code == _hx.HX_EINVAL
    with pytest.raises(_hx.HxError) as ei:
        eng.plan(q)
    assert ei.value.code == _hx.HX_EINVAL


def test_host_resident_shared_router(ctx):
    """Host-resident lineorder streamed in the blocks a shared router hands out
    (hx_pipeline_probe_agg_routed): every block once, bit-exact."""
    import os
    db = ssbgen.database(21, ssbgen.sizes(0.05))  # 300 K rows
    n = len(db["lineorder"]["lo_orderdate"])
    pin = lambda k: torch.empty(k, dtype=torch.int32, pin_memory=True)
    dims, fact = ssb.load_db_host_resident(ctx, db, pin)
    eng = ssb.SsbEngine(ctx, dims, fact)
    block = 4096 * 3 + 4  # ragged blocks; the last one partial
    n_blocks = (n + block - 1) // block
    r = hx.SharedRouter(f"/hx_test_routed_{os.getpid()}", n_blocks, create=True)
    for q in ("q1.1", "q2.1", "q3.1", "q4.3"):
        r.reset()
        rows, nb = eng.run_routed(q, r, block)
        assert nb == n_blocks, (q, nb)
        assert rows == oracle.run_query(q, db), q
    r.close(unlink=True)

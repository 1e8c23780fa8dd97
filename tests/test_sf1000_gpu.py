"""SF1000 on ONE B200: 6e9 lineorder rows (BASELINE.json configs[3]; SURVEY.md §8(d) C4's
1-GPU per-query-columns baseline of the 1 -> 8 GPU scaling run).

All 9 referenced lineorder columns (216 GB) do not fit one GPU's HBM, so the 13 queries run
in two phases over the columns they reference, generated in HBM by ssbgen (seed 42):
Q2.x-Q4.x over 6 columns (144 GB), Q1.x over 4 (96 GB). The launch configuration is
bench.py's (prepared plans, one CUDA graph of the phase's queries via hx_plans_enqueue).

What is checked:
* every query bit-exact against the oracle on sampled row ranges of the SAME 6e9-row table
  (its head, the rows around 2^31, 2^32 and the first K1 launch-segment boundary, its
  tail), each evaluated on the GPU as a view of the full table and summed — the oracle
  regenerates exactly those rows on the host;
* the full-table result equals the sum of the results over a partition of the table into
  three views (partition invariance: the full table runs as three
  segmented K1 launches of 2^31+ rows, each view as one launch);
* with HX_TEST_SF1000_FULL=1, every query over ALL 6e9 rows against the oracle run over
  the host's cores (regenerating 120 M rows at a time; ~10 min on 16 cores).
"""
import os

import pytest

import oracle
import ssbgen

pytestmark = pytest.mark.gpu

torch = pytest.importorskip("torch")
if not torch.cuda.is_available():
    pytest.skip("needs a CUDA GPU", allow_module_level=True)

from paper_journals_pvldb_chrysogeloskaa19_b200 import _hx, hx, ssb  # noqa: E402

SF = 1000
SEED = 42
C = ssbgen.COLS
PHASES = {"q2-q4": [q for q in ssb.QUERIES if not q.startswith("q1")],
          "q1": [q for q in ssb.QUERIES if q.startswith("q1")]}
K1_SEG_ROWS = 2560 << 20  # hx_probe.cu kSegRows


def lo_cols(queries):
    need = set().union(*(ssb.FACT_COLS[q] for q in queries))
    return [c for c in ssbgen.TABLE_COLS["lineorder"] if C[c] in need]


def sample_ranges(n):
    w = 2_000_000
    centres = [1 << 31, 1 << 32, K1_SEG_ROWS]
    return [(0, w)] + [(c - w // 2, c + w // 2) for c in centres] + [(n - w - 3, n)]


def as_rows_dict(rows):
    return {tuple(r[:-2]): (r[-2], r[-1]) for r in rows}


@pytest.mark.parametrize("phase", list(PHASES))
def test_sf1000_one_gpu(phase):
    queries = PHASES[phase]
    cols = lo_cols(queries)
    sz = ssbgen.sizes(SF)
    n = sz["n_lineorder"]
    torch.cuda.empty_cache()
    free, _ = torch.cuda.mem_get_info()
    need = n * 4 * len(cols) + (12 << 30)  # columns + dims, hash tables, group arrays
    if free < need:
        pytest.skip(f"needs {need / 2**30:.0f} GiB free HBM, have {free / 2**30:.0f}")
    ctx = hx.Context(0)
    stream = torch.cuda.current_stream().cuda_stream
    keep = []

    def table(names, rows):
        spec = []
        for c in names:
            t = torch.empty(rows, dtype=torch.int32, device="cuda")
            ssbgen.column_device(SEED, sz, c, t.data_ptr(), 0, rows, stream)
            keep.append(t)
            spec.append((C[c], t.data_ptr(), rows))
        return hx.load_columns(ctx, spec, placement=_hx.HX_PLACE_VIEW, keep=keep)

    objs = []
    try:
        dims = {t: table(ssbgen.TABLE_COLS[t], ssbgen.table_rows(sz, ssbgen.TABLE_COLS[t][0]))
                for t in ("date", "customer", "supplier", "part")}
        fact = table(cols, n)
        objs += list(dims.values()) + [fact]
        torch.cuda.synchronize()
        eng = ssb.SsbEngine(ctx, dims, fact)

        # the full table in the bench's launch configuration
        plans = {q: eng.plan(q) for q in queries}
        graph = hx.capture(ctx, lambda: hx.plans_enqueue(ctx, [plans[q].hp for q in queries]))
        graph.launch()
        full = {q: plans[q].rows() for q in queries}
        graph.close()
        for pl in plans.values():
            pl.close()
        for q in queries:
            assert full[q] == ssb.order_by(ssb.PLANS[q], full[q]), q  # ORDER BY holds

        # partition invariance: three views, each one K1 launch
        cuts = [0, 2_000_000_003, 4_100_000_001, n]
        parts = {q: [] for q in queries}
        for a, b in zip(cuts, cuts[1:]):
            sl = fact.slice(a, b)
            e = ssb.SsbEngine(ctx, dims, sl)
            for q in queries:
                parts[q].append(as_rows_dict(e.run(q)))
            sl.close()
        for q in queries:
            m = oracle.merge(parts[q])
            if oracle.N_KEYS[q] > 0:
                m = {k: v for k, v in m.items() if v[1] > 0}
            assert as_rows_dict(full[q]) == m, q

        # sampled rows against the oracle
        ranges = sample_ranges(n)
        got = {q: [] for q in queries}
        for a, b in ranges:
            sl = fact.slice(a, b)
            e = ssb.SsbEngine(ctx, dims, sl)
            for q in queries:
                got[q].append(as_rows_dict(e.run(q)))
            sl.close()
        dims_db = {t: {c: ssbgen.column(SEED, sz, c) for c in ssbgen.TABLE_COLS[t]}
                   for t in ("date", "customer", "supplier", "part")}

        def gen(b, k):
            return {c: ssbgen.column(SEED, sz, c, b, k) for c in cols}

        threads = min(os.cpu_count() or 8, 16)
        want = oracle.run_queries_generated(queries, dims_db, gen, ranges, threads)
        for q in queries:
            g = oracle.merge(got[q])
            if oracle.N_KEYS[q] > 0:
                g = {k: v for k, v in g.items() if v[1] > 0}
            assert g == want[q], q

        if os.environ.get("HX_TEST_SF1000_FULL") == "1":
            allrows = oracle.run_queries_generated(queries, dims_db, gen, [(0, n)],
                                                   os.cpu_count() or 8)
            for q in queries:
                assert as_rows_dict(full[q]) == allrows[q], q
            print(f"SF1000 full oracle parity ({phase}): {len(queries)} queries bit-exact")
    finally:
        for o in objs:
            o.close()
        ctx.close()
        keep.clear()
        torch.cuda.empty_cache()

"""Hash-partitioned join on the GPU, through the C-ABI.

* hx_hash_partition (hash-pack, K3) returns a permutation of the input rows in which part p
  holds exactly the rows whose key maps to p under the documented part function (restated
  here from include/hx.h), parts in order;
* identity-rank builds (HX_BUILD_IDENTITY_RANKS) rank every code of the static domain;
* an SSB query whose join with one dimension is hash-partitioned into n parts (lineorder
  part p meets only dimension part p; the other dimensions broadcast) gives the oracle's
  rows bit-exactly, for 1..16 parts, on every dimension a query can partition;
* the multi-GPU form with one rank (hx_exchange_partitions keeps part 0) likewise.
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

C = ssbgen.COLS


@pytest.fixture(scope="module")
def ctx():
    c = hx.Context(0)
    yield c
    c.close()


def part_of(keys: np.ndarray, n_parts: int) -> np.ndarray:
    """include/hx.h part function: fmix32 (murmur3 finaliser), then ((uint64)h * n_parts) >> 32."""
    m = np.uint64(0xFFFFFFFF)
    h = keys.astype(np.int64).astype(np.uint64) & m
    h ^= h >> np.uint64(16)
    h = (h * np.uint64(0x85EBCA6B)) & m
    h ^= h >> np.uint64(13)
    h = (h * np.uint64(0xC2B2AE35)) & m
    h ^= h >> np.uint64(16)
    return ((h * np.uint64(n_parts)) >> np.uint64(32)).astype(np.int64)


@pytest.mark.parametrize("kernel", ["tma", "ldg", "misaligned"])
@pytest.mark.parametrize("n_rows", [0, 1, 1000, 300_001])
@pytest.mark.parametrize("n_parts", [1, 3, 8, 64])
def test_hash_partition_is_a_grouped_permutation(ctx, monkeypatch, n_rows, n_parts, kernel):
    """Both K3 scatters: the bulk-copy one (aligned columns), the load-based one (HX_K3_LDG=1,
    and automatically for a view at an odd row offset)."""
    if kernel == "ldg":
        monkeypatch.setenv("HX_K3_LDG", "1")
    rng = np.random.default_rng(n_rows * 7 + n_parts)
    key = rng.integers(-2**31, 2**31 - 1, n_rows, dtype=np.int64).astype(np.int32)
    key[: n_rows // 3] = rng.integers(0, 50, n_rows // 3)  # heavy duplicates too
    a = rng.integers(-1000, 1000, n_rows).astype(np.int32)
    b = np.arange(n_rows, dtype=np.int32)
    full = None
    if kernel == "misaligned":  # the same rows behind one leading row: 4-byte aligned only
        pad = lambda v: np.concatenate([np.zeros(1, np.int32), v])
        full = hx.load_numpy(ctx, {10: pad(key), 11: pad(a), 12: pad(b)})
        t = full.slice(1, n_rows + 1)
    else:
        t = hx.load_numpy(ctx, {10: key, 11: a, 12: b})
    out, offs = hx.hash_partition(ctx, t, 10, n_parts)
    assert len(offs) == n_parts + 1 and offs[0] == 0 and offs[-1] == n_rows
    assert all(x <= y for x, y in zip(offs, offs[1:]))
    k2, a2, b2 = out.read(10), out.read(11), out.read(12)
    want_part = part_of(key, n_parts)
    got_part = np.repeat(np.arange(n_parts), np.diff(offs))
    assert np.array_equal(part_of(k2, n_parts), got_part)
    assert np.array_equal(np.bincount(want_part, minlength=n_parts), np.diff(offs))
    # a permutation of the rows: column b is the row id
    assert np.array_equal(np.sort(b2), b)
    assert np.array_equal(k2, key[b2]) and np.array_equal(a2, a[b2])
    out.close()
    t.close()
    if full is not None:
        full.close()


def test_identity_ranks(ctx):
    db = ssbgen.database(3, ssbgen.sizes(0.01))
    dims, _ = ssb.load_db_numpy(ctx, {**db, "lineorder": {k: v[:10] for k, v in db["lineorder"].items()}})
    # customers of ASIA grouped by nation: 5 codes present of the domain 0..24
    pr = [_hx.pred(C["c_region"], lo=2, hi=2)]
    dense = hx.build_dim_ht(ctx, dims["customer"], C["c_custkey"], pr, C["c_nation"], 0, 24)
    ident = hx.build_dim_ht(ctx, dims["customer"], C["c_custkey"], pr, C["c_nation"], 0, 24,
                            flags=_hx.HX_BUILD_IDENTITY_RANKS)
    d, i = dense.info(with_codes=True), ident.info(with_codes=True)
    assert d["n_keys"] == i["n_keys"] > 0 and d["n_ranks"] == 5 and i["n_ranks"] == 25
    assert i["rank_to_code"] == list(range(25))
    assert d["rank_to_code"] == sorted(set(d["rank_to_code"]))


# (query, dimension whose join is hash-partitioned): every dimension a query joins with a
# group column, a membership-only join, a single join (Q1.1's date)
CASES = [("q1.1", "date"), ("q2.1", "part"), ("q2.2", "supplier"), ("q3.1", "customer"),
         ("q3.2", "customer"), ("q3.3", "supplier"), ("q4.1", "customer"), ("q4.2", "part"),
         ("q4.3", "supplier"), ("q4.3", "date")]


@pytest.mark.parametrize("n_parts", [1, 2, 5, 16])
def test_hash_partitioned_join_parity(ctx, n_parts):
    db = ssbgen.database(11, ssbgen.sizes(0.05))
    dims, fact = ssb.load_db_numpy(ctx, db)
    eng = ssb.SsbEngine(ctx, dims, fact)
    for q, dim in CASES:
        assert eng.run_hash_partitioned(q, dim, n_parts) == oracle.run_query(q, db), (q, dim)


def test_hash_partitioned_join_missing_keys(ctx):
    """Foreign keys without a dimension row (tiny skewed databases) fall in some part and
    match nothing there, as in the broadcast join."""
    db = tiny_db(5, n_lo=20011)
    dims, fact = ssb.load_db_numpy(ctx, db)
    eng = ssb.SsbEngine(ctx, dims, fact)
    for q, dim in CASES:
        assert eng.run_hash_partitioned(q, dim, 7) == oracle.run_query(q, db), (q, dim)


def test_hash_routed_one_rank(ctx):
    db = ssbgen.database(2, ssbgen.sizes(0.01))
    dims, fact = ssb.load_db_numpy(ctx, db)
    eng = ssb.SsbEngine(ctx, dims, fact)
    for q, dim in CASES[:5]:
        assert eng.run_hash_routed(q, dim) == oracle.run_query(q, db), (q, dim)

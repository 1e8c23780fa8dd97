"""Pins of the CPU oracle (oracle/ssb_oracle.cpp) against things other than itself
(SURVEY.md §8(c) "What pins each part"):

  (a) hand-computed results on the handcrafted database  tests/golden/handcrafted_ssb.txt
  (b) brute-force nested-loop joins on tiny skewed databases (missing FKs, duplicate PKs)
  (c) closed forms: when every predicate passes, the query reduces to numpy dot / bincount
  (d) invariants: partition invariance (union-router merge); survivors
      conserved; group sums add to the total
  (e) SSB selectivities: survivor counts at SF1 match the analytic filter factors within 5 sigma
"""
import numpy as np
import pytest

import oracle
import ssbgen
import ssb_bruteforce as bf
from ssb_tiny import tiny_db

QUERIES = oracle.QUERIES


# ---- (a) dictionary and handcrafted results --------------------------------------------
@pytest.mark.parametrize("kind,literal,code", [
    ("region", "AFRICA", 0), ("region", "AMERICA", 1), ("region", "ASIA", 2),
    ("region", "EUROPE", 3), ("region", "MIDDLE EAST", 4),
    ("nation", "UNITED KINGDOM", 22), ("nation", "UNITED STATES", 23), ("nation", "CHINA", 4),
    ("city", "UNITED KI1", 221), ("city", "UNITED KI5", 225), ("city", "UNITED ST0", 230),
    ("mfgr", "MFGR#1", 0), ("mfgr", "MFGR#2", 1),
    ("category", "MFGR#12", 1), ("category", "MFGR#14", 3),
    ("brand1", "MFGR#2221", 260), ("brand1", "MFGR#2228", 267), ("brand1", "MFGR#2239", 278),
])
def test_encoding_table(kind, literal, code):
    """SURVEY.md §8(c) encoding table; oracle and generator dictionaries both agree with it."""
    assert oracle.encode(kind, literal) == code
    assert getattr(ssbgen, kind)(literal) == code


def test_generator_region_map_matches_tpch():
    sz = ssbgen.sizes(0.01)
    nat = ssbgen.column(1, sz, "c_nation")
    reg = ssbgen.column(1, sz, "c_region")
    for n, r in zip(nat, reg):
        assert ssbgen.REGIONS[r] == ssbgen.NATION_REGION[ssbgen.NATIONS[n]]


@pytest.mark.parametrize("q", QUERIES)
def test_handcrafted(handcrafted, q):
    db, expect = handcrafted
    got = oracle.run_query(q, db)
    assert got == expect[q], f"{q}: {got} != {expect[q]}"


@pytest.mark.parametrize("q", QUERIES)
def test_handcrafted_bruteforce_agrees(handcrafted, q):
    """The brute-force transcription also reproduces the hand-computed results."""
    db, expect = handcrafted
    want = {tuple(r[:-2]): (r[-2], r[-1]) for r in expect[q]}
    got = bf.run(q, db)
    if not got and oracle.N_KEYS[q] == 0:
        got = {(): (0, 0)}
    assert got == want


# ---- (b) brute force on tiny skewed databases -------------------------------------------
@pytest.mark.parametrize("seed,dups", [(1, False), (2, False), (3, True)])
def test_bruteforce_tiny(seed, dups):
    db = tiny_db(seed, dup_keys=dups)
    nonempty = 0
    for q in QUERIES:
        want = bf.run(q, db)
        got = oracle.as_dict(oracle.run_query(q, db))
        if oracle.N_KEYS[q] == 0:
            want = want or {(): (0, 0)}
        assert got == want, q
        nonempty += any(c > 0 for _, c in got.values())
    assert nonempty >= 11  # the skewed generator exercises (almost) every query


def test_oracle_order_by_q3_revenue_desc():
    db = tiny_db(5)
    rows = oracle.run_query("q3.1", db)
    assert rows, "need groups"
    for a, b in zip(rows, rows[1:]):
        # ORDER BY d_year asc, revenue desc (ties: codes ascending, reading R8)
        assert (a[2], -a[3], a[:3]) <= (b[2], -b[3], b[:3])


# ---- (c) closed forms --------------------------------------------------------------------
def _all_pass_db(seed, n=20000):
    sz = {"n_lineorder": n, "n_customer": 50, "n_supplier": 20, "n_part": 100, "n_date": 2557}
    db = ssbgen.database(seed, sz)
    lo = db["lineorder"]
    lo["lo_orderdate"][:] = 19930115
    lo["lo_discount"][:] = 2
    lo["lo_quantity"][:] = 10
    db["part"]["p_category"][:] = 1
    db["part"]["p_mfgr"][:] = 0
    db["supplier"]["s_region"][:] = 1
    db["customer"]["c_region"][:] = 1
    return db


def test_closed_form_q1_1_dot():
    db = _all_pass_db(11)
    lo = db["lineorder"]
    (s, c), = oracle.as_dict(oracle.run_query("q1.1", db)).values()
    assert c == len(lo["lo_orderdate"])
    assert s == int(np.dot(lo["lo_extendedprice"].astype(np.int64), lo["lo_discount"].astype(np.int64)))


def test_closed_form_q2_1_bincount():
    db = _all_pass_db(12)
    lo = db["lineorder"]
    got = oracle.as_dict(oracle.run_query("q2.1", db))
    brand = db["part"]["p_brand1"][lo["lo_partkey"] - 1]  # PKs are dense 1..P
    sums = np.bincount(brand, weights=None, minlength=1000)
    assert sum(c for _, c in got.values()) == len(brand)
    for b in np.unique(brand):
        m = brand == b
        assert got[(1993, int(b))] == (int(lo["lo_revenue"][m].astype(np.int64).sum()), int(sums[b]))


def test_closed_form_q4_1_total_profit():
    db = _all_pass_db(13)
    lo = db["lineorder"]
    got = oracle.as_dict(oracle.run_query("q4.1", db))
    total = int((lo["lo_revenue"].astype(np.int64) - lo["lo_supplycost"]).sum())
    assert sum(s for s, _ in got.values()) == total
    nat = db["customer"]["c_nation"][lo["lo_custkey"] - 1]
    assert set(got) == {(1993, int(n)) for n in np.unique(nat)}


def test_empty_lineorder():
    db = tiny_db(4)
    for q in QUERIES:
        rows = oracle.run_query(q, db, 0, 0)
        assert rows == ([(0, 0)] if oracle.N_KEYS[q] == 0 else [])


# ---- (d) invariants ----------------------------------------------------------------------
@pytest.mark.parametrize("q", QUERIES)
def test_partition_invariance(q):
    db = tiny_db(21, n_lo=6000)
    whole = oracle.as_dict(oracle.run_query(q, db))
    merged = oracle.run_query_ranges(q, db, 7)
    assert merged == whole


# ---- (e) selectivities at SF1 against the SSB filter factors -------------------------------
ORDER_DAYS = 2406  # 1992-01-01 .. 1998-08-02


@pytest.fixture(scope="module")
def sf1():
    return ssbgen.database(42, ssbgen.sizes(1))


def _expected_fraction(q, db):
    f = lambda col, pred: float(np.mean(pred(col)))  # realised fraction of dimension rows
    c, s, p = db["customer"], db["supplier"], db["part"]
    y9297 = (366 + 365 + 365 + 365 + 366 + 365) / ORDER_DAYS
    y9798 = (365 + 214) / ORDER_DAYS
    return {
        "q1.1": 365 / ORDER_DAYS * 3 / 11 * 24 / 50,
        "q1.2": 31 / ORDER_DAYS * 3 / 11 * 10 / 50,
        "q1.3": 7 / ORDER_DAYS * 3 / 11 * 10 / 50,
        "q2.1": f(p["p_category"], lambda x: x == 1) * f(s["s_region"], lambda x: x == 1),
        "q2.2": f(p["p_brand1"], lambda x: (x >= 260) & (x <= 267)) * f(s["s_region"], lambda x: x == 2),
        "q2.3": f(p["p_brand1"], lambda x: x == 278) * f(s["s_region"], lambda x: x == 3),
        "q3.1": f(c["c_region"], lambda x: x == 2) * f(s["s_region"], lambda x: x == 2) * y9297,
        "q3.2": f(c["c_nation"], lambda x: x == 23) * f(s["s_nation"], lambda x: x == 23) * y9297,
        "q3.3": f(c["c_city"], lambda x: np.isin(x, [221, 225])) * f(s["s_city"], lambda x: np.isin(x, [221, 225])) * y9297,
        "q3.4": f(c["c_city"], lambda x: np.isin(x, [221, 225])) * f(s["s_city"], lambda x: np.isin(x, [221, 225])) * 31 / ORDER_DAYS,
        "q4.1": f(c["c_region"], lambda x: x == 1) * f(s["s_region"], lambda x: x == 1) * f(p["p_mfgr"], lambda x: x <= 1),
        "q4.2": f(c["c_region"], lambda x: x == 1) * f(s["s_region"], lambda x: x == 1) * f(p["p_mfgr"], lambda x: x <= 1) * y9798,
        "q4.3": f(c["c_region"], lambda x: x == 1) * f(s["s_nation"], lambda x: x == 23) * f(p["p_category"], lambda x: x == 3) * y9798,
    }[q]


@pytest.mark.parametrize("q", QUERIES)
def test_selectivity_sf1(sf1, q):
    n = len(sf1["lineorder"]["lo_orderdate"])
    rows = oracle.run_query(q, sf1)
    survivors = sum(r[-1] for r in rows)
    pf = _expected_fraction(q, sf1)
    mu, sigma = n * pf, np.sqrt(n * pf * (1 - pf))
    assert abs(survivors - mu) < 5 * sigma + 1, (q, survivors, mu, sigma)


def test_dim_index_chunks_equal_run_query():
    """oracle.DimIndex (dimension maps built once, lineorder evaluated chunk by chunk on
    threads, partials summed) gives run_query's result: the SF1000 parity helper."""
    sz = ssbgen.sizes(0.2)
    db = ssbgen.database(5, sz)
    lo = db["lineorder"]
    n = sz["n_lineorder"]
    got = oracle.run_queries_generated(oracle.QUERIES, db, lambda b, k: {c: v[b:b + k] for c, v in lo.items()},
                                       [(0, 400_000), (400_000, n)], 3, chunk_rows=300_001)
    for q in oracle.QUERIES:
        assert got[q] == oracle.as_dict(oracle.run_query(q, db)), q

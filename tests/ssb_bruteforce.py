"""Brute-force nested-loop evaluator of the 13 SSB queries [SSB-spec] — an independent
transcription used to pin the oracle on tiny inputs (SURVEY.md §8(c) pin (i)).

It shares nothing with oracle/ssb_oracle.cpp: no hash maps, no std::map, no dictionary
functions. Every lineorder row is compared with EVERY row of each dimension (the textbook
nested-loop join: each matching combination contributes once), then the WHERE clause is
tested and the measure added to a dict keyed by the GROUP BY codes. Literal codes are typed
directly from SURVEY.md §8(c)'s encoding table. Use only at tiny sizes: O(N * |dims|).
"""
import itertools

import numpy as np

AMERICA, ASIA, EUROPE = 1, 2, 3
US = 23
KI1, KI5 = 221, 225


def _q(dims, where, key, measure):
    return {"dims": dims, "where": where, "key": key, "measure": measure}


def _ext_disc(lo):
    return lo["lo_extendedprice"] * lo["lo_discount"]


def _rev(lo):
    return lo["lo_revenue"]


def _profit(lo):
    return lo["lo_revenue"] - lo["lo_supplycost"]


QUERIES = {
    "q1.1": _q("d", lambda lo, d, c, s, p: d["d_year"] == 1993 and 1 <= lo["lo_discount"] <= 3
               and lo["lo_quantity"] < 25, lambda lo, d, c, s, p: (), _ext_disc),
    "q1.2": _q("d", lambda lo, d, c, s, p: d["d_yearmonthnum"] == 199401
               and 4 <= lo["lo_discount"] <= 6 and 26 <= lo["lo_quantity"] <= 35,
               lambda lo, d, c, s, p: (), _ext_disc),
    "q1.3": _q("d", lambda lo, d, c, s, p: d["d_weeknuminyear"] == 6 and d["d_year"] == 1994
               and 5 <= lo["lo_discount"] <= 7 and 26 <= lo["lo_quantity"] <= 35,
               lambda lo, d, c, s, p: (), _ext_disc),
    "q2.1": _q("dps", lambda lo, d, c, s, p: p["p_category"] == 1 and s["s_region"] == AMERICA,
               lambda lo, d, c, s, p: (d["d_year"], p["p_brand1"]), _rev),
    "q2.2": _q("dps", lambda lo, d, c, s, p: 260 <= p["p_brand1"] <= 267 and s["s_region"] == ASIA,
               lambda lo, d, c, s, p: (d["d_year"], p["p_brand1"]), _rev),
    "q2.3": _q("dps", lambda lo, d, c, s, p: p["p_brand1"] == 278 and s["s_region"] == EUROPE,
               lambda lo, d, c, s, p: (d["d_year"], p["p_brand1"]), _rev),
    "q3.1": _q("dcs", lambda lo, d, c, s, p: c["c_region"] == ASIA and s["s_region"] == ASIA
               and 1992 <= d["d_year"] <= 1997,
               lambda lo, d, c, s, p: (c["c_nation"], s["s_nation"], d["d_year"]), _rev),
    "q3.2": _q("dcs", lambda lo, d, c, s, p: c["c_nation"] == US and s["s_nation"] == US
               and 1992 <= d["d_year"] <= 1997,
               lambda lo, d, c, s, p: (c["c_city"], s["s_city"], d["d_year"]), _rev),
    "q3.3": _q("dcs", lambda lo, d, c, s, p: c["c_city"] in (KI1, KI5) and s["s_city"] in (KI1, KI5)
               and 1992 <= d["d_year"] <= 1997,
               lambda lo, d, c, s, p: (c["c_city"], s["s_city"], d["d_year"]), _rev),
    "q3.4": _q("dcs", lambda lo, d, c, s, p: c["c_city"] in (KI1, KI5) and s["s_city"] in (KI1, KI5)
               and d["d_yearmonthnum"] == 199712,
               lambda lo, d, c, s, p: (c["c_city"], s["s_city"], d["d_year"]), _rev),
    "q4.1": _q("dcsp", lambda lo, d, c, s, p: c["c_region"] == AMERICA and s["s_region"] == AMERICA
               and p["p_mfgr"] in (0, 1),
               lambda lo, d, c, s, p: (d["d_year"], c["c_nation"]), _profit),
    "q4.2": _q("dcsp", lambda lo, d, c, s, p: c["c_region"] == AMERICA and s["s_region"] == AMERICA
               and d["d_year"] in (1997, 1998) and p["p_mfgr"] in (0, 1),
               lambda lo, d, c, s, p: (d["d_year"], s["s_nation"], p["p_category"]), _profit),
    "q4.3": _q("dcsp", lambda lo, d, c, s, p: c["c_region"] == AMERICA and s["s_nation"] == US
               and d["d_year"] in (1997, 1998) and p["p_category"] == 3,
               lambda lo, d, c, s, p: (d["d_year"], s["s_city"], p["p_brand1"]), _profit),
}

_DIM = {"d": ("date", "d_datekey", "lo_orderdate"), "c": ("customer", "c_custkey", "lo_custkey"),
        "s": ("supplier", "s_suppkey", "lo_suppkey"), "p": ("part", "p_partkey", "lo_partkey")}


def run(q, db, row_begin=0, row_end=None):
    """{group codes: (sum, count)} by nested loops: each lineorder row is compared with
    every row of each joined dimension (vectorised over the dimension rows only)."""
    spec = QUERIES[q]
    lo_t = db["lineorder"]
    n = len(lo_t["lo_orderdate"]) if row_end is None else row_end
    dims = {}
    for k in spec["dims"]:
        table, pk, fk = _DIM[k]
        dims[k] = (db[table], pk, fk)
    out = {}
    for i in range(row_begin, n):
        lo = {c: int(v[i]) for c, v in lo_t.items()}
        matches = []
        for k in spec["dims"]:
            t, pk, fk = dims[k]
            idx = np.nonzero(t[pk] == lo[fk])[0]  # every dimension row whose PK equals the FK
            matches.append([{c: int(v[j]) for c, v in t.items()} for j in idx])
        for combo in itertools.product(*matches):
            bound = dict(zip(spec["dims"], combo))
            args = (lo, bound.get("d"), bound.get("c"), bound.get("s"), bound.get("p"))
            if spec["where"](*args):
                key = spec["key"](*args)
                s0, c0 = out.get(key, (0, 0))
                out[key] = (s0 + spec["measure"](lo), c0 + 1)
    return out

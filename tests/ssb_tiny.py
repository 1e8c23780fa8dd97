"""Tiny, skewed SSB databases for brute-force pins (test-side input generation only).

ssbgen's uniform distributions leave most SSB queries empty at a few thousand rows, so
here the dimension attributes are drawn from small value sets that contain the query
literals (SURVEY.md §8(c) encodings), order dates concentrate on the boundary days the
queries test, some foreign keys miss, and (optionally) some dimension keys are duplicated
so the join's multiplicity is exercised. Seeded numpy RNG; no query arithmetic.
"""
import numpy as np

import ssbgen

NATION_REGION = [ssbgen.region(ssbgen.NATION_REGION[n]) for n in ssbgen.NATIONS]
# 1993-01-15, 1994-01-05, 1994-02-03..1994-02-11, 1997-11-30, 1997-12-01, 1997-12-31,
# 1998-01-05, 1992-03-01, 1998-12-31
HOT_DATES = [19930115, 19940105, 19940203, 19940204, 19940205, 19940209, 19940210, 19940211,
             19971130, 19971201, 19971231, 19980105, 19920301, 19981231]


def tiny_db(seed, n_lo=3000, n_cust=40, n_supp=20, n_part=60, dup_keys=False, miss_frac=0.02):
    rng = np.random.default_rng(seed)
    sz = {"n_lineorder": n_lo, "n_customer": n_cust, "n_supplier": n_supp, "n_part": n_part,
          "n_date": ssbgen.N_DATE}
    db = {"date": {c: ssbgen.column(seed, sz, c) for c in ssbgen.TABLE_COLS["date"]}}

    def people(prefix, n):
        nations = rng.choice([2, 3, 4, 9, 13, 22, 23], size=n)
        digits = rng.choice([0, 1, 5, 9], size=n)
        return {f"{prefix}_city": (nations * 10 + digits).astype(np.int32),
                f"{prefix}_nation": nations.astype(np.int32),
                f"{prefix}_region": np.asarray([NATION_REGION[x] for x in nations], np.int32)}

    cust = {"c_custkey": np.arange(1, n_cust + 1, dtype=np.int32), **people("c", n_cust)}
    supp = {"s_suppkey": np.arange(1, n_supp + 1, dtype=np.int32), **people("s", n_supp)}
    cats = rng.choice([1, 3, 5, 6, 10], size=n_part)
    part = {"p_partkey": np.arange(1, n_part + 1, dtype=np.int32),
            "p_mfgr": (cats // 5).astype(np.int32), "p_category": cats.astype(np.int32),
            "p_brand1": (cats * 40 + rng.choice([0, 5, 20, 27, 28, 38], size=n_part)).astype(np.int32)}
    if dup_keys:
        # duplicate a few primary keys with different attributes (join multiplicity)
        for t in (cust, supp, part):
            k = list(t)[0]
            n = len(t[k])
            pick = rng.choice(n, size=max(1, n // 10), replace=False)
            for c in t:
                if c == k:
                    t[c] = np.concatenate([t[c], t[c][pick]])
                else:
                    t[c] = np.concatenate([t[c], rng.permutation(t[c])[: len(pick)]])
    db.update(customer=cust, supplier=supp, part=part)

    lo_gen = {c: ssbgen.column(seed, sz, c) for c in ssbgen.TABLE_COLS["lineorder"]}
    hot = rng.random(n_lo) < 0.6
    lo_gen["lo_orderdate"] = np.where(hot, rng.choice(HOT_DATES, size=n_lo),
                                      lo_gen["lo_orderdate"]).astype(np.int32)
    for fk, n in (("lo_custkey", n_cust), ("lo_suppkey", n_supp), ("lo_partkey", n_part)):
        miss = rng.random(n_lo) < miss_frac
        lo_gen[fk] = np.where(miss, n + 1 + rng.integers(0, 5, n_lo), lo_gen[fk]).astype(np.int32)
    miss = rng.random(n_lo) < miss_frac
    lo_gen["lo_orderdate"] = np.where(miss, 19930230, lo_gen["lo_orderdate"]).astype(np.int32)
    db["lineorder"] = lo_gen
    return db

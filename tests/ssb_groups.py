"""The grouping dimensions of the 13 SSB queries, from the query texts,
computed with numpy from the generated tables — independent of libhx. For query q, in
SELECT (GROUP BY) order: each grouping attribute's values and the mask of the dimension rows
passing that dimension's filter. The union router's group array is dense over the RANKS of
these attributes (the distinct passing codes, ascending; R17)."""
import numpy as np

AMERICA, ASIA, US, KI = 1, 2, 23, (221, 225)


def group_dims(db, q):
    d, c, s, p = db["date"], db["customer"], db["supplier"], db["part"]
    year = d["d_year"]
    y9297 = (year >= 1992) & (year <= 1997)
    y9798 = (year == 1997) | (year == 1998)
    brand, cat = p["p_brand1"], p["p_category"]
    every = np.ones(len(year), dtype=bool)
    return {
        "q1.1": [], "q1.2": [], "q1.3": [],
        "q2.1": [(year, every), (brand, cat == 1)],
        "q2.2": [(year, every), (brand, (brand >= 260) & (brand <= 267))],
        "q2.3": [(year, every), (brand, brand == 278)],
        "q3.1": [(c["c_nation"], c["c_region"] == ASIA), (s["s_nation"], s["s_region"] == ASIA),
                 (year, y9297)],
        "q3.2": [(c["c_city"], c["c_nation"] == US), (s["s_city"], s["s_nation"] == US),
                 (year, y9297)],
        "q3.3": [(c["c_city"], np.isin(c["c_city"], KI)), (s["s_city"], np.isin(s["s_city"], KI)),
                 (year, y9297)],
        "q3.4": [(c["c_city"], np.isin(c["c_city"], KI)), (s["s_city"], np.isin(s["s_city"], KI)),
                 (year, d["d_yearmonthnum"] == 199712)],
        "q4.1": [(year, every), (c["c_nation"], c["c_region"] == AMERICA)],
        "q4.2": [(year, y9798), (s["s_nation"], s["s_region"] == AMERICA),
                 (cat, np.isin(p["p_mfgr"], (0, 1)))],
        "q4.3": [(year, y9798), (s["s_city"], s["s_nation"] == US), (brand, cat == 3)],
    }[q]


def rank_maps(db, q):
    """rank -> code of each grouping dimension (an empty dimension keeps one empty rank)."""
    out = []
    for col, mask in group_dims(db, q):
        codes = np.unique(col[mask])
        out.append(codes if len(codes) else np.zeros(1, dtype=np.int32))
    return out


def n_groups(db, q):
    n = 1
    for m in rank_maps(db, q):
        n *= len(m)
    return n

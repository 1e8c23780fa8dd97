"""The 13 Star Schema Benchmark queries as HetExchange GPU plans over libhx.

PAPER.md:1160-1163 §6.1: "the optimizer of Proteus opts for broadcast-hash-join-based
plans" — every SSB query is one fused GPU pipeline over lineorder that probes one hash table
per joined dimension (Q1.x one join with date, Q2.x and Q3.x three,
Q4.x four), each table built from the FILTERED dimension. The query texts are the SSB
spec's [SSB-spec] (PAPER.md:1124-1125 cites SSB [26]; DESIGN.md restates them); string
literals are encoded with the input generator's order-preserving dictionary (ssbgen).

Plan choices that cannot change the result (R15): dimension predicates are pushed
into the hash-table build; joins are probed in ascending pass fraction (a miss drops the row
early); lineorder-only predicates (Q1.x) are evaluated before any probe.
"""
from __future__ import annotations

from dataclasses import dataclass, field
from typing import Dict, List, Optional, Sequence, Tuple

import numpy as np

import ssbgen

from . import _hx
from . import hx
from ._hx import pred

C = ssbgen.COLS


@dataclass
class DimBuild:
    table: str
    key: str
    preds: List[Tuple] = field(default_factory=list)   # (col, lo, hi) or (col, [values])
    group: Optional[Tuple[str, int, int]] = None       # (col, code_lo, code_hi)


@dataclass
class Plan:
    name: str
    joins: List[Tuple[str, DimBuild]]                  # (fact FK column, build), probe order
    agg: Tuple[int, str, str]                          # (HX_AGG_*, a, b)
    gdims: List[int] = field(default_factory=list)     # join indices, SELECT order of keys
    fact_preds: List[Tuple] = field(default_factory=list)
    order_q3: bool = False                             # ORDER BY d_year asc, revenue desc


YEAR = ("d_year", 1992, 1998)
NATION_C, NATION_S = ("c_nation", 0, 24), ("s_nation", 0, 24)
CITY_C, CITY_S = ("c_city", 0, 249), ("s_city", 0, 249)
BRAND = ("p_brand1", 0, 999)
CATEGORY = ("p_category", 0, 24)


def _date(preds=(), group=True):
    return DimBuild("date", "d_datekey", list(preds), YEAR if group else None)


def _plans() -> Dict[str, Plan]:
    R, N, CI = ssbgen.region, ssbgen.nation, ssbgen.city
    mf, cat, br = ssbgen.mfgr, ssbgen.category, ssbgen.brand1
    q1 = (_hx.HX_AGG_SUM_MUL, "lo_extendedprice", "lo_discount")
    rev = (_hx.HX_AGG_SUM, "lo_revenue", "lo_revenue")
    profit = (_hx.HX_AGG_SUM_SUB, "lo_revenue", "lo_supplycost")
    ki = [CI("UNITED KI1"), CI("UNITED KI5")]
    p = {}
    # Q1.x: select sum(lo_extendedprice*lo_discount) from lineorder, date where ...
    p["q1.1"] = Plan("q1.1", [("lo_orderdate", _date([("d_year", 1993, 1993)], group=False))], q1,
                     fact_preds=[("lo_discount", 1, 3), ("lo_quantity", None, 24)])
    p["q1.2"] = Plan("q1.2", [("lo_orderdate", _date([("d_yearmonthnum", 199401, 199401)], group=False))],
                     q1, fact_preds=[("lo_discount", 4, 6), ("lo_quantity", 26, 35)])
    p["q1.3"] = Plan("q1.3", [("lo_orderdate", _date([("d_weeknuminyear", 6, 6), ("d_year", 1994, 1994)],
                                                     group=False))],
                     q1, fact_preds=[("lo_discount", 5, 7), ("lo_quantity", 26, 35)])
    # Q2.x: sum(lo_revenue), d_year, p_brand1 ... group by d_year, p_brand1
    for q, ppred, reg in (("q2.1", ("p_category", cat("MFGR#12"), cat("MFGR#12")), "AMERICA"),
                          ("q2.2", ("p_brand1", br("MFGR#2221"), br("MFGR#2228")), "ASIA"),
                          ("q2.3", ("p_brand1", br("MFGR#2239"), br("MFGR#2239")), "EUROPE")):
        p[q] = Plan(q, [("lo_partkey", DimBuild("part", "p_partkey", [ppred], BRAND)),
                        ("lo_suppkey", DimBuild("supplier", "s_suppkey", [("s_region", R(reg), R(reg))])),
                        ("lo_orderdate", _date())], rev, gdims=[2, 0])
    # Q3.x: c attr, s attr, d_year, sum(lo_revenue) ... order by d_year asc, revenue desc
    y9297 = ("d_year", 1992, 1997)
    p["q3.1"] = Plan("q3.1", [
        ("lo_suppkey", DimBuild("supplier", "s_suppkey", [("s_region", R("ASIA"), R("ASIA"))], NATION_S)),
        ("lo_custkey", DimBuild("customer", "c_custkey", [("c_region", R("ASIA"), R("ASIA"))], NATION_C)),
        ("lo_orderdate", _date([y9297]))], rev, gdims=[1, 0, 2], order_q3=True)
    us = N("UNITED STATES")
    p["q3.2"] = Plan("q3.2", [
        ("lo_suppkey", DimBuild("supplier", "s_suppkey", [("s_nation", us, us)], CITY_S)),
        ("lo_custkey", DimBuild("customer", "c_custkey", [("c_nation", us, us)], CITY_C)),
        ("lo_orderdate", _date([y9297]))], rev, gdims=[1, 0, 2], order_q3=True)
    p["q3.3"] = Plan("q3.3", [
        ("lo_suppkey", DimBuild("supplier", "s_suppkey", [("s_city", ki)], CITY_S)),
        ("lo_custkey", DimBuild("customer", "c_custkey", [("c_city", ki)], CITY_C)),
        ("lo_orderdate", _date([y9297]))], rev, gdims=[1, 0, 2], order_q3=True)
    p["q3.4"] = Plan("q3.4", [
        ("lo_suppkey", DimBuild("supplier", "s_suppkey", [("s_city", ki)], CITY_S)),
        ("lo_custkey", DimBuild("customer", "c_custkey", [("c_city", ki)], CITY_C)),
        ("lo_orderdate", _date([("d_yearmonthnum", 199712, 199712)]))], rev, gdims=[1, 0, 2],
        order_q3=True)
    # Q4.x: d_year, ..., sum(lo_revenue - lo_supplycost) as profit
    am = R("AMERICA")
    m12 = [mf("MFGR#1"), mf("MFGR#2")]
    p["q4.1"] = Plan("q4.1", [
        ("lo_suppkey", DimBuild("supplier", "s_suppkey", [("s_region", am, am)])),
        ("lo_custkey", DimBuild("customer", "c_custkey", [("c_region", am, am)], NATION_C)),
        ("lo_partkey", DimBuild("part", "p_partkey", [("p_mfgr", m12)])),
        ("lo_orderdate", _date())], profit, gdims=[3, 1])
    p["q4.2"] = Plan("q4.2", [
        ("lo_suppkey", DimBuild("supplier", "s_suppkey", [("s_region", am, am)], NATION_S)),
        ("lo_custkey", DimBuild("customer", "c_custkey", [("c_region", am, am)])),
        ("lo_orderdate", _date([("d_year", [1997, 1998])])),
        ("lo_partkey", DimBuild("part", "p_partkey", [("p_mfgr", m12)], CATEGORY))],
        profit, gdims=[2, 0, 3])
    p["q4.3"] = Plan("q4.3", [
        ("lo_suppkey", DimBuild("supplier", "s_suppkey", [("s_nation", us, us)], CITY_S)),
        ("lo_partkey", DimBuild("part", "p_partkey", [("p_category", cat("MFGR#14"), cat("MFGR#14"))], BRAND)),
        ("lo_custkey", DimBuild("customer", "c_custkey", [("c_region", am, am)])),
        ("lo_orderdate", _date([("d_year", [1997, 1998])]))], profit, gdims=[3, 0, 1])
    return p


PLANS = _plans()
QUERIES = list(PLANS)
# lineorder columns each query's K1 scans (the referenced-column bytes of SURVEY.md §8(d))
FACT_COLS = {q: sorted({C[fk] for fk, _ in pl.joins} | {C[c[0]] for c in pl.fact_preds}
                       | {C[pl.agg[1]], C[pl.agg[2]]}) for q, pl in PLANS.items()}


def _hx_pred(t):
    if len(t) == 2:
        return pred(C[t[0]], isin=list(t[1]))
    return pred(C[t[0]], lo=t[1], hi=t[2])


@dataclass
class Pending:
    plan: Plan
    hts: list
    agg: hx.Agg


class SsbEngine:
    """Runs SSB plans on one GPU: dims are replicated device tables, `fact` this GPU's
    lineorder rows (its router blocks)."""

    def __init__(self, ctx: hx.Context, dims: Dict[str, hx.Table], fact: hx.Table):
        self.ctx, self.dims, self.fact = ctx, dims, fact

    def build(self, b: DimBuild) -> hx.HashTable:
        g = b.group
        return hx.build_dim_ht(self.ctx, self.dims[b.table], C[b.key],
                               [_hx_pred(t) for t in b.preds],
                               C[g[0]] if g else -1, g[1] if g else 0, g[2] if g else 0)

    def shape(self, plan: Plan):
        return hx.query_shape(
            preds=[_hx_pred(t) for t in plan.fact_preds],
            joins=[(C[fk], i) for i, (fk, _) in enumerate(plan.joins)],
            agg_op=plan.agg[0], agg_a=C[plan.agg[1]], agg_b=C[plan.agg[2]],
            gdims=plan.gdims)

    def start(self, q: str, fact: Optional[hx.Table] = None) -> Pending:
        """Enqueue the builds and the fused pipeline (asynchronous)."""
        plan = PLANS[q]
        hts = [self.build(b) for _, b in plan.joins]
        agg = hx.pipeline_probe_agg(self.ctx, fact or self.fact, self.shape(plan), hts)
        return Pending(plan, hts, agg)

    def finish(self, pend: Pending, root: int = -1) -> List[Tuple]:
        """Merge (union router; NCCL when the ctx has a communicator) and finalize."""
        keys, sums, cnts = hx.merge_aggregates(self.ctx, pend.agg, root)
        rows = [tuple(int(x) for x in keys[i]) + (int(sums[i]), int(cnts[i]))
                for i in range(len(sums))]
        for t in pend.hts:
            t.close()
        pend.agg.close()
        return order_by(pend.plan, rows)

    def run(self, q: str) -> List[Tuple]:
        return self.finish(self.start(q))

    # ---- hash-partitioned join of one dimension -------------------
    def _partitioned_build(self, b: DimBuild, dim_rows: hx.Table) -> hx.HashTable:
        g = b.group
        return hx.build_dim_ht(self.ctx, dim_rows, C[b.key], [_hx_pred(t) for t in b.preds],
                               C[g[0]] if g else -1, g[1] if g else 0, g[2] if g else 0,
                               flags=_hx.HX_BUILD_IDENTITY_RANKS)

    def _join_of(self, plan: Plan, dim: str) -> int:
        js = [i for i, (_, b) in enumerate(plan.joins) if b.table == dim]
        if len(js) != 1:
            raise ValueError(f"{plan.name} does not join {dim} once")
        return js[0]

    def run_hash_partitioned(self, q: str, dim: str, n_parts: int) -> List[Tuple]:
        """Hash-partitioned join on ONE GPU: lineorder and dimension `dim` are hash-packed on
        the join key into n_parts parts (K3, hx_hash_partition); part p of lineorder meets only
        part p of the dimension — the rows rank p would hold after the hash-routing exchange
         — while the other dimensions stay broadcast. The
        partitioned dimension's table of each part is built with identity ranks, so every
        part's partial aggregate has one group layout; the parts accumulate into one
        aggregate (the union router) and merge."""
        plan = PLANS[q]
        j = self._join_of(plan, dim)
        fk, b = plan.joins[j]
        fparts, foffs = hx.hash_partition(self.ctx, self.fact, C[fk], n_parts)
        dparts, doffs = hx.hash_partition(self.ctx, self.dims[dim], C[b.key], n_parts)
        hts = [self.build(bb) if i != j else None for i, (_, bb) in enumerate(plan.joins)]
        shape = self.shape(plan)
        agg, keep = None, []
        for p in range(n_parts):
            fp = fparts.slice(foffs[p], foffs[p + 1])
            dp = dparts.slice(doffs[p], doffs[p + 1])
            htp = self._partitioned_build(b, dp)
            hts_p = list(hts)
            hts_p[j] = htp
            if agg is None:
                agg = hx.pipeline_probe_agg(self.ctx, fp, shape, hts_p)
            else:
                hx.pipeline_probe_agg_into(self.ctx, fp, shape, hts_p, agg)
            keep += [fp, dp, htp]
        hts[j] = keep[2]
        rows = self.finish(Pending(plan, [t for t in hts if t is not None], agg))
        for o in keep:
            o.close()
        fparts.close()
        dparts.close()
        return rows

    def run_routed(self, q: str, router: hx.SharedRouter, block_rows: int,
                   root: int = -1) -> Tuple[List[Tuple], int]:
        """Host-resident lineorder (self.fact: HX_PLACE_HOST_PINNED over the WHOLE table)
        streamed in the blocks a shared router hands out — every process of the node draws
        from the same counter, so each GPU takes blocks as fast as it consumes them
         — then the union-router merge. -> (rows, blocks this rank ran)."""
        plan = PLANS[q]
        hts = [self.build(b) for _, b in plan.joins]
        agg, nb = hx.pipeline_probe_agg_routed(self.ctx, self.fact, self.shape(plan), hts, router,
                                               block_rows)
        return self.finish(Pending(plan, hts, agg), root), nb

    def run_hash_routed(self, q: str, dim: str, root: int = -1,
                        dim_local: Optional[hx.Table] = None) -> List[Tuple]:
        """The multi-GPU form: every rank hash-packs its lineorder rows into nranks parts and
        the hash-routing exchange (hx_exchange_partitions, NCCL send/recv over NVLink) gives
        rank r part r of everyone's rows; rank r joins them with part r of the dimension
        (identity ranks; the other dimensions broadcast), and the union router merges the
        partials (allreduce). With one rank: a copy of itself.
        The dimension is replicated (self.dims[dim]: part r is taken locally) unless
        `dim_local` gives this rank's share of a PARTITIONED dimension (each row on exactly
        one rank): then it is hash-packed and exchanged too, both inputs of the join going
        through the hash-routing router (Fig. 1d/e)."""
        plan = PLANS[q]
        j = self._join_of(plan, dim)
        fk, b = plan.joins[j]
        rank, nr = self.ctx.comm_info()
        fparts, foffs = hx.hash_partition(self.ctx, self.fact, C[fk], nr)
        f_in = hx.exchange_partitions(self.ctx, fparts, foffs)
        fparts.close()
        if dim_local is None:
            # a replicated dimension (§8(a) a1): rank r's part is already local — hash-pack
            # it and keep part r (exchanging it would deliver nranks copies of every key)
            dparts, doffs = hx.hash_partition(self.ctx, self.dims[dim], C[b.key], nr)
            d_in = dparts.slice(doffs[rank], doffs[rank + 1])
        else:
            # a partitioned dimension: its rows hashed to part p go to rank p
            dparts, doffs = hx.hash_partition(self.ctx, dim_local, C[b.key], nr)
            d_in = hx.exchange_partitions(self.ctx, dparts, doffs)
        hts = [self.build(bb) if i != j else self._partitioned_build(bb, d_in)
               for i, (_, bb) in enumerate(plan.joins)]
        agg = hx.pipeline_probe_agg(self.ctx, f_in, self.shape(plan), hts)
        rows = self.finish(Pending(plan, hts, agg), root)
        f_in.close()
        d_in.close()
        dparts.close()
        return rows

    # ---- prepared plans (allocation- and sync-free executions, graph capturable) ----------
    DIM_ORDER = ("date", "customer", "supplier", "part")

    def plan(self, q: str, fact: Optional[hx.Table] = None) -> "QueryPlan":
        plan = PLANS[q]
        dims = [self.dims[t] for t in self.DIM_ORDER]
        builds = []
        for _, b in plan.joins:
            g = b.group
            builds.append(hx.build_spec(self.DIM_ORDER.index(b.table), C[b.key],
                                        [_hx_pred(t) for t in b.preds],
                                        C[g[0]] if g else -1, g[1] if g else 0, g[2] if g else 0))
        return QueryPlan(plan, hx.Plan(self.ctx, fact or self.fact, dims, builds, self.shape(plan)))


class QueryPlan:
    """A prepared SSB query: enqueue() runs builds -> K1 -> merge -> finalize on the device;
    rows() waits and returns the result in ORDER BY order."""

    def __init__(self, plan: Plan, hp: hx.Plan):
        self.plan, self.hp = plan, hp

    def enqueue(self) -> None:
        self.hp.enqueue()

    def rows(self) -> List[Tuple]:
        keys, sums, cnts = self.hp.result()
        # the device finalize emits groups in group-index order = the group codes ascending in
        # SELECT order (dense ranks preserve code order), which already is the ORDER BY of
        # Q2.x / Q4.x; Q3.x re-sorts by (d_year asc, revenue desc, codes asc)
        if self.plan.order_q3 and len(sums) > 1:
            idx = np.lexsort(tuple(keys[:, c] for c in range(keys.shape[1] - 1, -1, -1))
                             + (-sums, keys[:, 2]))
            keys, sums, cnts = keys[idx], sums[idx], cnts[idx]
        return [tuple(k) + (s, c) for k, s, c in zip(keys.tolist(), sums.tolist(), cnts.tolist())]

    def close(self) -> None:
        self.hp.close()


def order_by(plan: Plan, rows: List[Tuple]) -> List[Tuple]:
    """SSB ORDER BY: the group keys ascending (Q2, Q4), or d_year asc, revenue desc (Q3;
    ties by the group codes ascending, R8)."""
    if plan.order_q3:
        return sorted(rows, key=lambda r: (r[2], -r[-2], r[:-2]))
    return sorted(rows, key=lambda r: r[:-2])


# ---- loading an SSB database onto one GPU --------------------------------------------------
def load_db_numpy(ctx: hx.Context, db: Dict[str, Dict[str, np.ndarray]],
                  part: Optional[hx.Partition] = None, part_index: int = 0):
    """Host numpy tables -> device tables (mem-move H2D). Lineorder is restricted to the
    router blocks of `part_index` when a partition is given; dimensions are replicated."""
    dims = {t: hx.load_numpy(ctx, {C[c]: v for c, v in db[t].items()})
            for t in ("date", "customer", "supplier", "part")}
    fact = hx.load_numpy(ctx, {C[c]: v for c, v in db["lineorder"].items()}, part, part_index)
    return dims, fact


def load_db_host_resident(ctx: hx.Context, db: Dict[str, Dict[str, np.ndarray]], pin,
                          placement: int = _hx.HX_PLACE_HOST_PINNED):
    """Dimensions to the device; lineorder stays in page-locked host memory.
    HX_PLACE_HOST_PINNED: K1 streams it block by block over PCIe (mem-move, §8(a) a8);
    HX_PLACE_HOST_MAPPED: K1 reads it in place through UVA (zero-copy, §8(f) NEXT-3).
    `pin(n)` returns a page-locked (and, for MAPPED, device-mapped) int32 buffer of n values
    with .ctypes / data_ptr access (e.g. lambda n: torch.empty(n, dtype=torch.int32,
    pin_memory=True): the CUDA caching host allocator maps its pages)."""
    dims = {t: hx.load_numpy(ctx, {C[c]: v for c, v in db[t].items()})
            for t in ("date", "customer", "supplier", "part")}
    keep, spec = [], []
    for c, v in db["lineorder"].items():
        buf = pin(max(1, len(v)))
        arr = buf.numpy() if hasattr(buf, "numpy") else buf
        arr[: len(v)] = v
        keep.append(buf)
        spec.append((C[c], arr.ctypes.data, len(v)))
    fact = hx.load_columns(ctx, spec, placement=placement, keep=keep)
    return dims, fact

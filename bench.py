#!/usr/bin/env python
"""Benchmark of the HetExchange SSB hot path on B200 (BASELINE.json metric).

One STEP = all 13 SSB queries, each one pass of the whole hot path over this GPU's
lineorder partition: filter + hash-table build of every joined dimension (K2), the fused
scan -> filter -> probe x k -> aggregate pipeline (K1), and the union-router merge of the
partial aggregates (NCCL allreduce when N > 1) with the result copied to the host.

Workload (config.workload): SSB SF100 per GPU, HBM-resident — BASELINE.json configs[2], the
largest configuration that fits one GPU (N=1); weak scaling: N GPUs run SF 100*N with
lineorder range-partitioned in 2^22-row router blocks and the dimensions replicated.
Synthetic dbgen-shaped data from ssbgen (seed 42), generated directly in HBM outside the
timed region. Each query scans 9.6-14.4 GB per GPU, far larger than the 126 MB L2, so no L2
flush is needed between queries (--l2-flush flushes between steps for the SF1 C1 case).

    python bench.py [--gpus N] [--steps K] [--warmup W] [--sf SF_PER_GPU] [--impl reference]
    python -m torch.distributed.run --nproc-per-node N ... bench.py --gpus N ...

`--gpus N > 1` without a torch.distributed launcher re-executes itself under
`python -m torch.distributed.run --nproc-per-node N` (one process per GPU); under a launcher,
WORLD_SIZE must equal N (a mismatch is an error, never a silent 1-GPU run).
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys
import tempfile
import time

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

import numpy as np  # noqa: E402

import ssbgen  # noqa: E402

with open(os.path.join(ROOT, "BASELINE.json")) as _f:
    METRIC = json.load(_f)["metric"]
UNIT = "lineorder rows/s"
SEED = 42
BLOCK_ROWS = 1 << 22
SCALING = ["weak"]  # "strong" with --sf-total


def parse(argv=None):
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=50)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--sf", type=float, default=100.0, help="SSB scale factor per GPU (weak scaling)")
    ap.add_argument("--sf-total", type=float, default=0.0,
                    help="strong scaling: this total scale factor split over the GPUs (e.g. "
                         "configs[3]: --sf-total 1000 --gpus 2|4|8); overrides --sf")
    ap.add_argument("--impl", default="hx", choices=["hx", "reference"])
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--no-e2e", action="store_true")
    ap.add_argument("--queries", default="all")
    ap.add_argument("--no-graph", action="store_true", help="enqueue plans without a CUDA graph")
    ap.add_argument("--no-pipeline", action="store_true",
                    help="one plan set: the host reads a step's results before the next starts")
    ap.add_argument("--variant", default="hbm", choices=["hbm", "host", "uva"],
                    help="host: lineorder in pinned host memory streamed over PCIe (config 5, "
                         "mem-move DMA); uva: the same memory read in place by K1 (zero-copy)")
    ap.add_argument("--workload", default="ssb", choices=["ssb", "sum", "join"],
                    help="sum / join: the paper's §6.4 micro-benchmarks (SUM over one 23 GB "
                         "column; COUNT of a 1:N join with a 7.7 MB build side)")
    ap.add_argument("--force-collectives", action="store_true",
                    help="N=1: a 1-rank NCCL communicator with HX_FORCE_COLLECTIVES=1, so the "
                         "step includes the union-router allreduce a multi-GPU step issues")
    ap.add_argument("--micro-rows", type=int, default=0,
                    help="fact rows per GPU of the micro-benchmarks (default: the paper's 23 GB)")
    ap.add_argument("--router", default="static", choices=["static", "shared"],
                    help="--variant host: static = each rank streams its own router blocks (plans, "
                         "CUDA graph); shared = ONE pinned copy of lineorder in shared memory, blocks "
                         "drawn from a shared counter by whichever GPU is free (dynamic load "
                         "balancing, PAPER.md:469-473)")
    ap.add_argument("--sizeup", action="store_true",
                    help="with --workload sum|join: the §6.4 size-up sweep (0.125-16 GB per "
                         "column), one JSON line per size")
    ap.add_argument("--no-ht-path", action="store_true",
                    help="skip the ht_path block (the same plans on open-addressing hash tables)")
    ap.add_argument("--l2-flush", action="store_true",
                    help="flush L2 (write 2x its size) between timed steps, outside the per-step "
                         "events (small inputs, e.g. C1 = --sf 1 --queries q1.1)")
    return ap.parse_args(argv)


def dist_env():
    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    return world, rank, local


def free_port():
    import socket
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    port = s.getsockname()[1]
    s.close()
    return port


def launch_plan(gpus, env, argv):
    """How this invocation runs: ("run", None) in this process, ("relaunch", cmd) under
    torch.distributed.run with one process per GPU, or ("error", message).
    `--gpus N > 1` without WORLD_SIZE re-executes under the launcher; with WORLD_SIZE set it
    must equal N (the driver's torchrun launch), never a silent 1-GPU run."""
    if gpus < 1:
        return "error", f"bench.py: --gpus {gpus} < 1"
    ws = env.get("WORLD_SIZE")
    if ws is None:
        if gpus == 1:
            return "run", None
        cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1",
               f"--nproc-per-node={gpus}", "--master-addr=127.0.0.1",
               f"--master-port={free_port()}", os.path.abspath(__file__)] + list(argv)
        return "relaunch", cmd
    if int(ws) != gpus:
        return "error", f"bench.py: --gpus {gpus} but WORLD_SIZE={ws} (launch one process per GPU)"
    return "run", None


def peaks():
    try:
        with open(os.path.join(ROOT, "MEASURED_PEAKS.json")) as f:
            m = json.load(f)
        return float(m["hbm_gbs"]), "measured (MEASURED_PEAKS.json hbm_gbs)"
    except Exception:
        return 6650.0, "fallback (B200_PROFILING.md)"


def workload_name(sf, world, variant="hbm", queries=None):
    if variant in ("host", "uva"):
        how = ("streamed over PCIe (mem-move DMA into a device ring)" if variant == "host"
               else "read in place over PCIe by K1 through UVA (zero-copy)")
        return (f"SSB {'/'.join(q.upper() for q in queries)}, SF{sf:g} per GPU (SF{sf * world:g} "
                f"total), lineorder host-resident in pinned memory, {how}")
    which = ("all 13 queries" if queries is None or len(queries) == 13
             else "/".join(q.upper() for q in queries))
    return f"SSB {which}, SF{sf:g} per GPU (SF{sf * world:g} total), HBM-resident"


def config(args, world, n_rows_gpu, queries):
    return {"workload": workload_name(args.sf, world, getattr(args, "variant", "hbm"), queries),
            "sf_per_gpu": args.sf,
            "sf_total": args.sf * world, "queries": queries,
            "lineorder_rows_per_gpu": n_rows_gpu, "router_block_rows": BLOCK_ROWS,
            "parallelism": f"lineorder block-partitioned over {world} GPU(s); dims replicated; "
                           "partials merged by NCCL allreduce" if world > 1 else
                           ("1 GPU, 1-rank NCCL communicator issuing the merge allreduce"
                            if getattr(args, "force_collectives", False) else "1 GPU"),
            "l2": ("L2 flushed between steps (a 256 MB buffer written outside the per-step "
                   "events)" if getattr(args, "l2_flush", False) else
                   f"inputs larger than L2 (each query scans >= {0.096 * args.sf:.2f} GB/GPU vs "
                   f"126 MB L2); no flush")}


class Clocks:
    """nvidia-smi sampling DURING the timed region (B200_PROFILING.md clocks line)."""

    def __init__(self, index):
        self.index, self.proc, self.path = index, None, None

    def start(self):
        try:
            fd, self.path = tempfile.mkstemp(suffix=".csv")
            os.close(fd)
            self.proc = subprocess.Popen(
                ["nvidia-smi", "-i", str(self.index), "--query-gpu=clocks.sm,clocks.max.sm,"
                 "clocks_event_reasons.active,clocks_event_reasons.hw_slowdown,"
                 "clocks_event_reasons.hw_thermal_slowdown,clocks_event_reasons.sw_thermal_slowdown,"
                 "clocks_event_reasons.sw_power_cap", "--format=csv,noheader,nounits", "-lms", "20"],
                stdout=open(self.path, "w"), stderr=subprocess.DEVNULL)
        except Exception:
            self.proc = None

    def stop(self):
        if not self.proc:
            return None
        time.sleep(0.25)
        self.proc.terminate()
        self.proc.wait()
        sm, mx, reasons = [], 0, set()
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        with open(self.path) as f:
            for line in f:
                parts = [p.strip() for p in line.split(",")]
                if len(parts) < 7:
                    continue
                try:
                    sm.append(float(parts[0]))
                    mx = max(mx, float(parts[1]))
                except ValueError:
                    continue
                for n, v in zip(names, parts[3:7]):
                    if v.lower() == "active":
                        reasons.add(n)
        os.unlink(self.path)
        if not sm:
            return None
        return {"sm_mhz": statistics.median(sm), "sm_max_mhz": mx, "reasons": sorted(reasons),
                "samples": len(sm)}


def ncu_traffic():
    """DRAM bytes per K1 launch from the committed ncu --set full capture (or None)."""
    p = os.path.join(ROOT, "profiles", "k1_traffic.json")
    try:
        with open(p) as f:
            return json.load(f)
    except Exception:
        return None


# ---------------------------------------------------------------------------------------
def run_reference(args, world, rank):
    """--impl reference: the oracle (the paper's method as a plain CPU program) as it stands,
    on this box's host cores, over a bounded sample of the same workload per step."""
    import oracle
    if rank != 0:
        return
    sz = ssbgen.sizes(args.sf * world)
    threads = os.cpu_count() or 1
    sample = min(sz["n_lineorder"], 125_000 * threads)
    db = ssbgen.database(SEED, sz, 0, sample)
    queries = oracle.QUERIES if args.queries == "all" else args.queries.split(",")
    # the oracle's dimension maps are built once (oracle.DimIndex; a per-process setup like the
    # GPU side's plans), the timed steps evaluate the queries row by row over `threads` row
    # ranges, partials merged by summation (evaluation only is timed)
    import threading
    idx = oracle.DimIndex(db)
    bounds = np.linspace(0, sample, threads + 1).astype(np.int64)

    def step():
        for q in queries:
            parts = [None] * threads

            def work(i):
                parts[i] = idx.query(q, db["lineorder"], int(bounds[i]), int(bounds[i + 1]))

            ts = [threading.Thread(target=work, args=(i,)) for i in range(threads)]
            for t in ts:
                t.start()
            for t in ts:
                t.join()
            oracle.merge(parts)

    for _ in range(args.warmup):
        step()
    t0 = time.perf_counter()
    for _ in range(args.steps):
        step()
    dt = (time.perf_counter() - t0) / args.steps
    value = len(queries) * sample / dt
    idx.close()
    samp = (f"lineorder rows [0, {sample}) of SF{args.sf * world:g} (dims full, their maps built "
            f"once outside the clock), {len(queries)} queries, {threads} threads")
    line = {"impl": "reference", "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": world,
            "steps": args.steps, "warmup": args.warmup, "ms_per_step": dt * 1e3,
            "higher_is_better": True, "scaling": SCALING[0], "vs_baseline": None, "dtype": "int64",
            "data": f"synthetic (ssbgen dbgen-shaped SSB, seed {SEED})",
            "config": dict(config(args, world, sz["n_lineorder"] // world, queries),
                           executed_as=f"reference arm: the CPU oracle (oracle/ssb_oracle.cpp) "
                                       f"over lineorder rows [0, {sample}) in host memory, not "
                                       f"the HBM-resident GPU path", sample_rows=sample),
            "cpu_baseline": {"value": value, "unit": UNIT, "cores": threads, "kind": "oracle",
                             "sample": samp},
            "e2e": {"value": value, "unit": UNIT, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}}
    print(json.dumps(line), flush=True)


def cpu_baseline(args, world):
    """The oracle, single-threaded as it stands, on a bounded sample (rank 0, N=1)."""
    import oracle
    sz = ssbgen.sizes(args.sf * world)
    sample = min(sz["n_lineorder"], 12_000_000)  # ~10 s of single-threaded oracle work
    db = ssbgen.database(SEED, sz, 0, sample)
    idx = oracle.DimIndex(db)  # the dimension maps, built once (not timed: SURVEY.md 8(d))
    # pinned to one core for the timed evaluation (taskset to one core)
    aff = os.sched_getaffinity(0) if hasattr(os, "sched_getaffinity") else None
    core = min(aff) if aff else None
    if core is not None:
        os.sched_setaffinity(0, {core})
    try:
        t0 = time.perf_counter()
        for q in oracle.QUERIES:
            idx.query(q, db["lineorder"])
        dt = time.perf_counter() - t0
    finally:
        if aff:
            os.sched_setaffinity(0, aff)
    idx.close()
    return {"value": 13 * sample / dt, "unit": UNIT, "cores": 1, "kind": "oracle",
            "sample": f"13 queries over lineorder rows [0, {sample}) of SF{args.sf * world:g} "
                      f"(full dims, maps built once outside the clock), single-threaded, pinned "
                      f"to core {core}, {dt:.1f} s"}


def run_micro(args, world, rank, local, ctx, stream, torch, dist, hx):
    """--workload sum|join: §6.4 micro-benchmarks, one step = one
    execution of the prepared plan (join: K2 build of the 7.7 MB side + K1 probe; sum: K1
    scan) + merge + finalize + result to the host, in a CUDA graph."""
    from paper_journals_pvldb_chrysogeloskaa19_b200 import micro
    n_gpu = args.micro_rows or ssbgen.MICRO_PAPER_ROWS
    sz = ssbgen.micro_sizes(n_gpu * world, ssbgen.MICRO_PAPER_BUILD)
    r0 = rank * n_gpu
    keep = []
    C = ssbgen.COLS

    def dev_table(cols, row_begin, n):
        spec = []
        for c in cols:
            t = torch.empty(max(n, 1), dtype=torch.int32, device="cuda")
            ssbgen.column_device(SEED, sz, c, t.data_ptr(), row_begin, n, stream.cuda_stream)
            keep.append(t)
            spec.append((C[c], t.data_ptr(), n))
        return hx.load_columns(ctx, spec, placement=hx._hx.HX_PLACE_VIEW)

    cols = ["mb_value"] if args.workload == "sum" else ["mb_value", "mb_probekey"]
    fact = dev_table(cols, r0, n_gpu)
    build = dev_table(["mb_buildkey"], 0, sz["n_part"])
    torch.cuda.synchronize()
    eng = micro.MicroEngine(ctx, fact, build)
    plans = [eng.plan_sum() if args.workload == "sum" else eng.plan_join() for _ in range(2)]
    graphs = [hx.capture(ctx, lambda p=p: hx.plans_enqueue(ctx, [p])) for p in plans]
    k1 = [0.0, 0]

    def run(n, timed=False):
        for i in range(n):
            graphs[i % 2].launch()
            if i:
                eng.plan_value(plans[(i - 1) % 2], args.workload)
                if timed:
                    k1[0] += plans[(i - 1) % 2].k1_time()[0]
                    k1[1] += 1
        if n:
            eng.plan_value(plans[(n - 1) % 2], args.workload)
            if timed:
                k1[0] += plans[(n - 1) % 2].k1_time()[0]
                k1[1] += 1

    run(args.warmup)
    clocks = Clocks(local)
    if world > 1:
        dist.barrier()
    torch.cuda.synchronize()
    clocks.start()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record(stream)
    run(args.steps, timed=True)
    e1.record(stream)
    torch.cuda.synchronize()
    if world > 1:
        dist.barrier()
    clk = clocks.stop()
    ms = e0.elapsed_time(e1)
    launches, _, _ = ctx.stats(reset=True)
    if world > 1:
        t = torch.tensor([ms], device="cuda", dtype=torch.float64)
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
        ms = float(t[0])
    ms_step = ms / args.steps
    bpr = 4 * len(cols)
    peak, peak_src = peaks()
    k1_ms = k1[0] / max(k1[1], 1)
    achieved = n_gpu * bpr / (k1_ms / 1e3) / 1e9 if k1_ms > 0 else 0.0
    cpu = None
    if rank == 0 and world == 1 and not args.no_cpu_baseline:
        from oracle import micro as omicro
        sample = min(n_gpu, 200_000_000)
        v = ssbgen.column(SEED, sz, "mb_value", 0, sample)
        t0 = time.perf_counter()
        if args.workload == "sum":
            omicro.sum_column([v])
        else:
            pk = ssbgen.column(SEED, sz, "mb_probekey", 0, sample)
            bk = ssbgen.column(SEED, sz, "mb_buildkey")
            t0 = time.perf_counter()
            omicro.join_count(bk, [(pk, v)])
        dt = time.perf_counter() - t0
        cpu = {"value": sample / dt, "unit": "fact rows/s", "cores": 1, "kind": "oracle",
               "sample": f"oracle/micro.py (numpy) over fact rows [0, {sample}), {dt:.1f} s"}
    if rank == 0:
        name = ("§6.4 SUM over one int32 column" if args.workload == "sum" else
                "§6.4 COUNT (and SUM) of a non-partitioned 1:N join")
        line = {"metric": f"micro-benchmark fact rows/sec & HBM GB/s ({args.workload})",
                "value": n_gpu * world / (ms_step / 1e3), "unit": "fact rows/s",
                "n_gpus": world, "steps": args.steps, "warmup": args.warmup,
                "ms_per_step": ms_step, "higher_is_better": True, "scaling": SCALING[0],
                "vs_baseline": None, "dtype": "int32 columns, int64 accumulate",
                "data": f"synthetic (ssbgen mb_* columns, seed {SEED}), generated in HBM",
                "config": {"workload": f"{name}: {n_gpu * 4 / 1e9:.1f} GB per column per GPU, "
                                       f"build side {sz['n_part'] * 4 / 1e6:.1f} MB (PAPER.md:1364-1366)",
                           "fact_rows_per_gpu": n_gpu, "build_rows": sz["n_part"],
                           "l2": "inputs larger than L2; no flush"},
                "roofline": {"bound": "hbm", "achieved": achieved, "peak": peak, "unit": "GB/s",
                             "frac": achieved / peak, "peak_source": peak_src,
                             "kernel": "k1_probe_agg", "algorithmic_bytes_per_launch": n_gpu * bpr,
                             "k1_ms_per_launch": k1_ms, "traffic": None},
                "cpu_baseline": cpu, "e2e": None, "clocks": clk, "gpu_launches": launches}
        print(json.dumps(line), flush=True)
    for g in graphs:
        g.close()
    for p in plans:
        p.close()
    fact.close()
    build.close()


def run_host_routed(args, world, rank, local, ctx, stream, torch, dist, hx, ssb, queries):
    """--variant host --router shared: lineorder (the referenced columns of the whole table)
    lives ONCE in shared pinned host memory that every rank maps (cudaHostRegister); each
    query's blocks are drawn from a shared counter (hx_shared_router) as GPUs free a staging
    slot — the paper's router with dynamic load balancing over the consumers (PAPER.md:469-473,
    1214-1233) — then merged by the union router (NCCL allreduce). Not a CUDA graph (the host
    draws blocks). value = queries x rows / step time (max over ranks)."""
    from multiprocessing import shared_memory
    C = ssbgen.COLS
    sz = ssbgen.sizes(args.sf * world)
    n = sz["n_lineorder"]
    need = set().union(*(ssb.FACT_COLS[q] for q in queries))
    lo_cols = [c for c in ssbgen.TABLE_COLS["lineorder"] if C[c] in need]
    tag = os.environ.get("MASTER_PORT", str(os.getpid()))
    shm_name = f"hx_bench_lo_{tag}"
    if rank == 0:
        shm = shared_memory.SharedMemory(name=shm_name, create=True, size=4 * n * len(lo_cols))
    if world > 1:
        dist.barrier()
    if rank != 0:
        shm = shared_memory.SharedMemory(name=shm_name)
    buf = np.ndarray((len(lo_cols), n), dtype=np.int32, buffer=shm.buf)
    if rank == 0:  # fill from the seeded generator (in HBM, copied down in pieces)
        piece = 1 << 27
        tmp = torch.empty(piece, dtype=torch.int32, device="cuda")
        for i, c in enumerate(lo_cols):
            for b in range(0, n, piece):
                k = min(piece, n - b)
                ssbgen.column_device(SEED, sz, c, tmp.data_ptr(), b, k, stream.cuda_stream)
                torch.cuda.synchronize()
                buf[i, b:b + k] = tmp[:k].cpu().numpy()
        del tmp
    if world > 1:
        dist.barrier()
    ptr = buf.ctypes.data
    assert torch.cuda.cudart().cudaHostRegister(ptr, buf.nbytes, 1) == 0  # portable pinning
    keep = []

    def dev_table(cols, nrows):
        spec = []
        for c in cols:
            t = torch.empty(max(nrows, 1), dtype=torch.int32, device="cuda")
            ssbgen.column_device(SEED, sz, c, t.data_ptr(), 0, nrows, stream.cuda_stream)
            keep.append(t)
            spec.append((C[c], t.data_ptr(), nrows))
        return hx.load_columns(ctx, spec, placement=hx._hx.HX_PLACE_VIEW)

    dims = {t: dev_table(ssbgen.TABLE_COLS[t], ssbgen.table_rows(sz, ssbgen.TABLE_COLS[t][0]))
            for t in ("date", "customer", "supplier", "part")}
    fact = hx.load_columns(ctx, [(C[c], ptr + 4 * n * i, n) for i, c in enumerate(lo_cols)],
                           placement=hx._hx.HX_PLACE_HOST_PINNED)
    torch.cuda.synchronize()
    block = 1 << 21
    n_blocks = (n + block - 1) // block
    rname = f"/{shm_name}_r"
    router = hx.SharedRouter(rname, n_blocks, create=True) if rank == 0 else None
    if world > 1:
        dist.barrier()
    if rank != 0:
        router = hx.SharedRouter(rname, n_blocks, create=False)
    eng = ssb.SsbEngine(ctx, dims, fact)
    mine_blocks = [0]

    def step():
        for q in queries:
            if rank == 0:
                router.reset()
            if world > 1:
                dist.barrier()
            _, nb = eng.run_routed(q, router, block)
            mine_blocks[0] += nb

    for _ in range(args.warmup):
        step()
    ctx.stats(reset=True)
    mine_blocks[0] = 0
    clocks = Clocks(local)
    if world > 1:
        dist.barrier()
    torch.cuda.synchronize()
    clocks.start()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record(stream)
    for _ in range(args.steps):
        step()
    e1.record(stream)
    torch.cuda.synchronize()
    if world > 1:
        dist.barrier()
    clk = clocks.stop()
    ms = e0.elapsed_time(e1)
    launches, h2d, d2h = ctx.stats(reset=True)
    share = float(mine_blocks[0]) / max(1, args.steps * len(queries) * n_blocks)
    if world > 1:
        t = torch.tensor([ms, float(launches), share, share], device="cuda", dtype=torch.float64)
        dist.all_reduce(t[:1], op=dist.ReduceOp.MAX)
        dist.all_reduce(t[1:2], op=dist.ReduceOp.SUM)
        dist.all_reduce(t[2:3], op=dist.ReduceOp.MIN)
        dist.all_reduce(t[3:4], op=dist.ReduceOp.MAX)
        ms, launches, smin, smax = float(t[0]), int(t[1]), float(t[2]), float(t[3])
    else:
        smin = smax = share
    ms_step = ms / args.steps
    value = len(queries) * n / (ms_step / 1e3)
    # the host link's own ceiling, measured in this run (pinned H2D, 1 GiB, best of 3)
    hb = torch.empty(1 << 28, dtype=torch.int32, pin_memory=True)
    dbf = torch.empty(1 << 28, dtype=torch.int32, device="cuda")
    best = 0.0
    for _ in range(3):
        c0, c1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        c0.record(stream)
        dbf.copy_(hb, non_blocking=True)
        c1.record(stream)
        torch.cuda.synchronize()
        best = max(best, hb.numel() * 4 / (c0.elapsed_time(c1) / 1e3) / 1e9)
    del hb, dbf
    streamed = sum(4 * len(ssb.FACT_COLS[q]) * n for q in queries) / (ms_step / 1e3) / 1e9
    if rank == 0:
        print(json.dumps({
            "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": world, "steps": args.steps,
            "warmup": args.warmup, "ms_per_step": ms_step, "higher_is_better": True,
            "scaling": SCALING[0], "vs_baseline": None, "dtype": "int32 columns, int64 accumulate",
            "data": f"synthetic (ssbgen dbgen-shaped SSB, seed {SEED}), lineorder in shared pinned "
                    "host memory",
            "config": dict(config(args, world, n // world, queries), router="shared counter "
                           "(hx_shared_router): blocks of 2^21 rows to whichever GPU frees a "
                           "staging slot", block_rows=block, n_blocks=n_blocks),
            "roofline": {"bound": "pcie", "achieved": streamed, "peak": best * world,
                         "unit": "GB/s", "frac": streamed / (best * world),
                         "peak_source": "measured in this run: pinned H2D cudaMemcpyAsync, 1 GiB, "
                                        "best of 3, x GPUs",
                         "kernel": "mem-move H2D ring + k1_probe_agg per drawn block",
                         "traffic": None},
            "load_balance": {"min_share": smin, "max_share": smax,
                             "ideal_share": 1.0 / world},
            "e2e": {"value": value, "unit": UNIT, "h2d_bytes_per_step": h2d // args.steps,
                    "d2h_bytes_per_step": d2h // args.steps, "ms_per_step": ms_step,
                    "path": "builds + hx_pipeline_probe_agg_routed + hx_merge_aggregates per query"},
            "cpu_baseline": None, "clocks": clk, "gpu_launches": launches}), flush=True)
    fact.close()
    for t in dims.values():
        t.close()
    torch.cuda.cudart().cudaHostUnregister(ptr)
    router.close(unlink=(rank == 0))
    if world > 1:
        dist.barrier()
    del buf
    shm.close()
    if rank == 0:
        shm.unlink()


def run_sizeup(args, world, rank, local, ctx, stream, torch, dist, hx):
    """--workload sum|join --sizeup: the §6.4 size-up sweep (Fig. 8):
    the same prepared plan over the first 0.125 ... 16 GB of the column(s), one JSON line per
    size. Reported beside rows/s: the step's fixed part (step - K1: graph launch, builds,
    merge, finalize, D2H) and the overhead against the ideal scan at the read-stream ceiling
    (the paper: <= 10% above 512 MB, up to 50% at 64 MB for its GPU sum)."""
    from paper_journals_pvldb_chrysogeloskaa19_b200 import micro
    sizes_gb = [0.125, 0.25, 0.5, 1, 2, 4, 8, 16]
    n_max = int(sizes_gb[-1] * 1e9) // 4
    sz = ssbgen.micro_sizes(n_max * world, ssbgen.MICRO_PAPER_BUILD)
    C = ssbgen.COLS
    keep = []

    def gen(c, row_begin, n):
        t = torch.empty(max(n, 1), dtype=torch.int32, device="cuda")
        ssbgen.column_device(SEED, sz, c, t.data_ptr(), row_begin, n, stream.cuda_stream)
        keep.append(t)
        return t

    cols = ["mb_value"] if args.workload == "sum" else ["mb_value", "mb_probekey"]
    full = {c: gen(c, rank * n_max, n_max) for c in cols}
    bt = gen("mb_buildkey", 0, sz["n_part"])
    build = hx.load_columns(ctx, [(C["mb_buildkey"], bt.data_ptr(), sz["n_part"])],
                            placement=hx._hx.HX_PLACE_VIEW)
    torch.cuda.synchronize()
    peak, _ = peaks()
    read_ceiling = 7100.0  # GB/s, tools/stream_roofline.cu
    for gb in sizes_gb:
        n = (int(gb * 1e9) // 4) & ~3
        fact = hx.load_columns(ctx, [(C[c], full[c].data_ptr(), n) for c in cols],
                               placement=hx._hx.HX_PLACE_VIEW)
        eng = micro.MicroEngine(ctx, fact, build)
        plan = eng.plan_sum() if args.workload == "sum" else eng.plan_join()
        graph = hx.capture(ctx, lambda: hx.plans_enqueue(ctx, [plan]))
        for _ in range(max(3, args.warmup)):
            graph.launch()
            eng.plan_value(plan, args.workload)
        if world > 1:
            dist.barrier()
        torch.cuda.synchronize()
        evs = [torch.cuda.Event(enable_timing=True) for _ in range(args.steps + 1)]
        k1 = 0.0
        evs[0].record(stream)
        for i in range(args.steps):
            graph.launch()
            evs[i + 1].record(stream)
            eng.plan_value(plan, args.workload)
            k1 += plan.k1_time()[0]
        torch.cuda.synchronize()
        steps = sorted(a.elapsed_time(b) for a, b in zip(evs, evs[1:]))
        ms = steps[len(steps) // 2]
        if world > 1:
            t = torch.tensor([ms], device="cuda", dtype=torch.float64)
            dist.all_reduce(t, op=dist.ReduceOp.MAX)
            ms = float(t[0])
        k1_ms = k1 / args.steps
        bytes_ = n * 4 * len(cols)
        ideal_ms = bytes_ / (read_ceiling * 1e9) * 1e3
        if rank == 0:
            print(json.dumps({
                "metric": f"micro-benchmark size-up ({args.workload})", "size_gb_per_column": gb,
                "fact_rows_per_gpu": n, "n_gpus": world, "steps": args.steps,
                "ms_per_step_median": ms, "k1_ms": k1_ms, "fixed_ms": ms - k1_ms,
                "value": n * world / (ms / 1e3), "unit": "fact rows/s",
                "gbps_step": bytes_ / (ms / 1e3) / 1e9, "gbps_k1": bytes_ / (k1_ms / 1e3) / 1e9,
                "frac_of_peak_step": bytes_ / (ms / 1e3) / 1e9 / peak,
                "overhead_vs_ideal_scan": ms / ideal_ms - 1.0,
                "ideal_definition": f"bytes / {read_ceiling:.0f} GB/s read-stream ceiling",
                "step": "one CUDA graph launch of the prepared plan (builds + K1 + merge + "
                        "finalize + D2H) + the host read of the result"}), flush=True)
        graph.close()
        plan.close()
        fact.close()
    build.close()


def nccl_log_env(env):
    """NCCL's communicator log on (INFO, INIT subsystem: it shows nranks = N) and written to
    stderr, so that stdout carries only the one JSON line. The image sets NCCL_DEBUG=VERSION,
    which prints a bare version line on stdout: anything below INFO is raised to INFO."""
    if env.get("NCCL_DEBUG", "").upper() not in ("INFO", "TRACE"):
        env["NCCL_DEBUG"] = "INFO"
    env.setdefault("NCCL_DEBUG_SUBSYS", "INIT")
    env.setdefault("NCCL_DEBUG_FILE", "/dev/stderr")


def main():
    args = parse()
    how, what = launch_plan(args.gpus, os.environ, sys.argv[1:])
    if how == "error":
        print(what, file=sys.stderr, flush=True)
        sys.exit(2)
    if how == "relaunch":
        env = dict(os.environ)
        nccl_log_env(env)
        sys.exit(subprocess.run(what, env=env).returncode)
    world, rank, local = dist_env()
    if args.sf_total > 0:
        args.sf = args.sf_total / world
    SCALING[0] = "strong" if args.sf_total > 0 else "weak"
    if world > 1 or args.force_collectives:
        nccl_log_env(os.environ)
    if args.impl == "reference":
        run_reference(args, world, rank)
        return

    import torch
    import torch.distributed as dist
    from paper_journals_pvldb_chrysogeloskaa19_b200 import hx, ssb

    if torch.cuda.device_count() <= local:
        print(f"bench.py: rank {rank} needs GPU {local} but {torch.cuda.device_count()} are visible",
              file=sys.stderr, flush=True)
        sys.exit(2)
    torch.cuda.set_device(local)
    if world > 1:
        dist.init_process_group("nccl", device_id=torch.device("cuda", local))
    # one real (non-legacy) stream shared by torch and the library: the timing events below
    # are recorded on the very stream the kernels are launched on
    stream = torch.cuda.Stream(device=local)
    torch.cuda.set_stream(stream)
    ctx = hx.Context(local, stream.cuda_stream)
    assert ctx.stream == stream.cuda_stream
    if world > 1:
        uid = [hx.comm_unique_id() if rank == 0 else None]
        dist.broadcast_object_list(uid, src=0)
        ctx.comm_init(world, rank, uid[0])
    elif args.force_collectives:
        os.environ["HX_FORCE_COLLECTIVES"] = "1"
        ctx.comm_init(1, 0, hx.comm_unique_id())
    if args.workload != "ssb" and args.sizeup:
        run_sizeup(args, world, rank, local, ctx, stream, torch, dist, hx)
        ctx.close()
        if world > 1:
            dist.destroy_process_group()
        return
    if args.workload != "ssb":
        run_micro(args, world, rank, local, ctx, stream, torch, dist, hx)
        ctx.close()
        if world > 1:
            dist.destroy_process_group()
        return
    if args.queries == "all":
        queries = ["q2.1", "q3.1", "q4.1"] if args.variant in ("host", "uva") else ssb.QUERIES
    else:
        queries = args.queries.split(",")
    if args.variant == "host" and args.router == "shared":
        run_host_routed(args, world, rank, local, ctx, stream, torch, dist, hx, ssb, queries)
        ctx.close()
        if world > 1:
            dist.destroy_process_group()
        return
    C = ssbgen.COLS
    # only the lineorder columns the selected queries reference are placed (SF1000 on one
    # GPU: the 6 columns of Q2-Q4 = 144 GB or the 4 of Q1 = 96 GB fit HBM; all 9 do not)
    need = set().union(*(ssb.FACT_COLS[q] for q in queries))
    lo_cols = [c for c in ssbgen.TABLE_COLS["lineorder"] if C[c] in need]

    # ---- data in HBM: this rank's router blocks of lineorder, full replicated dims -------
    sz = ssbgen.sizes(args.sf * world)
    part = hx.router_partition(sz["n_lineorder"], world, BLOCK_ROWS)
    mine = [(b, e) for b, e, p in part.blocks() if p == rank]
    r0, r1 = (mine[0][0], mine[-1][1]) if mine else (0, 0)
    n_mine = r1 - r0
    keep = []

    def dev_table(cols, row_begin, n):
        spec = []
        for c in cols:
            t = torch.empty(max(n, 1), dtype=torch.int32, device="cuda")
            ssbgen.column_device(SEED, sz, c, t.data_ptr(), row_begin, n, stream.cuda_stream)
            keep.append(t)
            spec.append((C[c], t.data_ptr(), n))
        return hx.load_columns(ctx, spec, placement=hx._hx.HX_PLACE_VIEW)

    dims = {t: dev_table(ssbgen.TABLE_COLS[t], 0, ssbgen.table_rows(sz, ssbgen.TABLE_COLS[t][0]))
            for t in ("date", "customer", "supplier", "part")}
    if args.variant in ("host", "uva"):
        # §8(a) a8: lineorder stays in page-locked host memory; K1 streams it over PCIe
        # (host: DMA into a device staging ring; uva: K1's bulk copies read it in place)
        spec = []
        for c in lo_cols:
            buf = torch.empty(max(n_mine, 1), dtype=torch.int32, pin_memory=True)
            ssbgen.column(SEED, sz, c, r0, n_mine, out=buf.numpy())
            keep.append(buf)
            spec.append((C[c], buf.data_ptr(), n_mine))
        fact = hx.load_columns(ctx, spec, placement=hx._hx.HX_PLACE_HOST_PINNED if args.variant == "host"
                               else hx._hx.HX_PLACE_HOST_MAPPED)
    else:
        fact = dev_table(lo_cols, r0, n_mine)
    torch.cuda.synchronize()
    eng = ssb.SsbEngine(ctx, dims, fact)
    # one prepared plan per query (HT + group buffers allocated once, builds sized once);
    # the 13 executions are captured into ONE CUDA graph: a step is one graph launch plus
    # the 13 host reads of the finalized results. Two such plan sets alternate (steps i and
    # i+1 use different buffers), so the host reads step i's results while the device
    # already runs step i+1 — every step still builds, probes, merges and reads everything.
    big = n_mine * 4 * len(lo_cols) > (64 << 30)  # SF >= ~300 per GPU: one plan set fits
    n_sets = 1 if (args.no_graph or args.no_pipeline or big or args.l2_flush) else 2
    sets = []
    for _ in range(n_sets):
        pl_ = {q: eng.plan(q) for q in queries}
        od_ = [pl_[q].hp for q in queries]
        gr_ = None if args.no_graph else hx.capture(ctx, lambda od_=od_: hx.plans_enqueue(ctx, od_))
        sets.append((pl_, od_, gr_))
    plans, order, graph = sets[0]
    # SURVEY.md §8(d) algorithmic bytes per lineorder row: the referenced columns (16 B for
    # Q1-Q3, 24 B for Q4); the bytes K1 actually moves can be fewer (late materialisation)
    B = {q: 4 * len(ssb.FACT_COLS[q]) for q in queries}
    k1_acc = [0.0, 0, 0, 0.0, 0]  # ms, launches, moved bytes, span ms, algorithmic bytes

    def launch(st):
        if st[2] is not None:
            st[2].launch()
        else:
            hx.plans_enqueue(ctx, st[1])

    def collect(st, timed):
        out = [st[0][q].rows() for q in queries]
        if timed:
            k1_acc[3] += st[1][0].k1_span(st[1][-1])
            for q in queries:
                ms_, b_ = st[0][q].hp.k1_time()
                k1_acc[0] += ms_
                k1_acc[1] += 1
                k1_acc[2] += b_
                k1_acc[4] += n_mine * B[q]
        return out

    step_ev = []  # an event after each timed step's launch: per-step device times

    # --l2-flush: a 2 x L2 buffer is written between steps (outside the per-step events), so
    # every step starts with a cold L2 (inputs smaller than L2, e.g. C1 = SF1 Q1.1, 96 MB)
    flush_buf = torch.empty(64 << 20, dtype=torch.int32, device="cuda") if args.l2_flush else None
    flush_ev = []

    def run_steps(n, timed=False):
        prev = None
        for i in range(n):
            cur = sets[i % n_sets]
            if flush_buf is not None:
                flush_buf.fill_(i)
                if timed:
                    ev = torch.cuda.Event(enable_timing=True)
                    ev.record(stream)
                    flush_ev.append(ev)
            launch(cur)
            if timed:
                ev = torch.cuda.Event(enable_timing=True)
                ev.record(stream)
                step_ev.append(ev)
            if n_sets == 1:
                collect(cur, timed)
                continue
            if prev is not None:
                collect(prev, timed)
            prev = cur
        if prev is not None:
            collect(prev, timed)

    # ---- warm-up, then exactly K timed steps ---------------------------------------------
    run_steps(args.warmup)
    ctx.stats(reset=True)
    clocks = Clocks(local)
    if world > 1:
        dist.barrier()
    torch.cuda.synchronize()
    clocks.start()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record(stream)
    run_steps(args.steps, timed=True)
    e1.record(stream)
    torch.cuda.synchronize()
    if world > 1:
        dist.barrier()
    clk = clocks.stop()
    ms = e0.elapsed_time(e1)
    if flush_buf is not None:  # the steps only: each from its flush's end to its own end
        ms = sum(a.elapsed_time(b) for a, b in zip(flush_ev, step_ev))
    k1_ms, k1_n, k1_moved, k1_span, k1_bytes = k1_acc
    launches, step_h2d, step_d2h = ctx.stats(reset=True)
    if world > 1:
        t = torch.tensor([ms, float(launches)], device="cuda", dtype=torch.float64)
        dist.all_reduce(t[:1], op=dist.ReduceOp.MAX)
        dist.all_reduce(t[1:], op=dist.ReduceOp.SUM)
        ms, launches = float(t[0]), int(t[1])
    ms_step = ms / args.steps
    per_step = ([a.elapsed_time(b) for a, b in zip(flush_ev, step_ev)] if flush_buf is not None else
                [e0.elapsed_time(step_ev[0])] + [a.elapsed_time(b) for a, b in zip(step_ev, step_ev[1:])])
    total_rows = sz["n_lineorder"]
    value = len(queries) * total_rows / (ms_step / 1e3)

    peak, peak_src = peaks()
    achieved = (k1_bytes / (k1_ms / 1e3)) / 1e9 if k1_ms > 0 else 0.0
    moved = (k1_moved / (k1_ms / 1e3)) / 1e9 if k1_ms > 0 else 0.0
    tr = ncu_traffic()
    roofline = {"bound": "hbm", "achieved": achieved, "peak": peak, "unit": "GB/s",
                "frac": achieved / peak, "peak_source": peak_src,
                "kernel": f"k1_probe_agg (fused scan->filter->probe->aggregate), {len(queries)} queries",
                "algorithmic_bytes_per_launch": k1_bytes / max(k1_n, 1),
                "algorithmic_bytes_definition": "SURVEY.md 8(d): 4 B x referenced lineorder columns "
                                                "(16 B/row Q1-Q3, 24 B/row Q4) x rows",
                "moved_bytes_per_launch": k1_moved / max(k1_n, 1),
                "moved_bytes_definition": "streamed columns (4 B/row) + one 32-B sector per "
                                          "gathered measure value of a row that passed every join",
                "achieved_moved": moved, "frac_moved": moved / peak,
                "peak_nominal": 8000.0, "frac_nominal": achieved / 8000.0,
                "peak_read_stream": 7100.0,
                "peak_read_stream_source": "tools/stream_roofline.cu: the same bulk-copy ring with "
                                           "trivial consumers, 7.0-7.2 TB/s on this B200 (DESIGN.md 7)",
                "k1_ms_per_launch": k1_ms / max(k1_n, 1),
                "k1_busy_frac_of_step": k1_ms / ms if ms > 0 else None,
                "k1_span_ms_per_step": k1_span / args.steps,
                "traffic": tr["dram_bytes_per_launch"] if tr else None,
                "traffic_source": tr["source"] if tr else None}
    if args.variant in ("host", "uva"):
        # the streamed pipeline (H2D copies overlapped with K1) is bound by the host link:
        # peak = this run's own pinned H2D copy bandwidth (1 GiB, best of 3)
        hb = torch.empty(1 << 28, dtype=torch.int32, pin_memory=True)
        db_ = torch.empty(1 << 28, dtype=torch.int32, device="cuda")
        best = 0.0
        for _ in range(3):
            c0, c1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            c0.record(stream)
            db_.copy_(hb, non_blocking=True)
            c1.record(stream)
            torch.cuda.synchronize()
            best = max(best, hb.numel() * 4 / (c0.elapsed_time(c1) / 1e3) / 1e9)
        del hb, db_
        roofline.update({"bound": "pcie", "peak": best, "frac": achieved / best,
                         "peak_source": "measured in this run: pinned H2D cudaMemcpyAsync, 1 GiB, best of 3",
                         "kernel": ("mem-move H2D ring + k1_probe_agg per block (achieved = streamed "
                                    "referenced-column bytes / span of the query's K1 launches)")
                         if args.variant == "host" else
                         "k1_probe_agg reading mapped host memory through UVA (achieved = "
                         "referenced-column bytes / K1 time)",
                         "traffic": None, "traffic_source": None})

    # ---- per query (after the timed region): K1-only and whole-query time ---------------
    per_query = {}
    for q in queries:
        reps = 5
        qe0, qe1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        kms, kmoved = 0.0, 0
        qe0.record(stream)
        for _ in range(reps):
            plans[q].enqueue()
            plans[q].rows()
            ms_, b_ = plans[q].hp.k1_time()
            kms += ms_
            kmoved += b_
        qe1.record(stream)
        torch.cuda.synchronize()
        qms = qe0.elapsed_time(qe1) / reps
        kms /= reps
        per_query[q] = {"query_ms": round(qms, 4), "k1_ms": round(kms, 4),
                        "rows_per_s": n_mine / (qms / 1e3),
                        "k1_hbm_gbps": n_mine * B[q] / (kms / 1e3) / 1e9 if kms else None,
                        "k1_frac_of_peak": (n_mine * B[q] / (kms / 1e3) / 1e9) / peak if kms else None,
                        "bytes_per_row": B[q],
                        "k1_moved_gbps": kmoved / reps / (kms / 1e3) / 1e9 if kms else None,
                        "k1_frac_moved": kmoved / reps / (kms / 1e3) / 1e9 / peak if kms else None,
                        "moved_bytes_per_row": kmoved / reps / max(n_mine, 1)}

    # ---- ht_path: the same step on open-addressing hash tables (north_star's layout) -------
    # Plans created under HX_OPT_JOIN_LAYOUT = HX_JOIN_HASH probe the hash tables of the
    # dimension builds instead of direct maps (R20); same
    # results, timed the same way (one graph per step, K steps), per query K1 as above.
    ht_path = None
    if args.variant == "hbm" and not args.no_ht_path and not big:
        ctx.set_option(hx._hx.HX_OPT_JOIN_LAYOUT, hx._hx.HX_JOIN_HASH)
        hpl = {q: eng.plan(q) for q in queries}
        ctx.set_option(hx._hx.HX_OPT_JOIN_LAYOUT, hx._hx.HX_JOIN_AUTO)
        hod = [hpl[q].hp for q in queries]
        hgr = hx.capture(ctx, lambda: hx.plans_enqueue(ctx, hod))
        same = True
        for _ in range(max(1, args.warmup)):
            hgr.launch()
            same = same and all(hpl[q].rows() == plans[q].rows() for q in queries)
        if world > 1:
            dist.barrier()
        torch.cuda.synchronize()
        he0, he1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        hk = {q: [0.0, 0] for q in queries}
        he0.record(stream)
        for _ in range(args.steps):
            hgr.launch()
            for q in queries:
                hpl[q].rows()
                ms_, b_ = hpl[q].hp.k1_time()
                hk[q][0] += ms_
                hk[q][1] += b_
        he1.record(stream)
        torch.cuda.synchronize()
        hms = he0.elapsed_time(he1)
        if world > 1:
            t = torch.tensor([hms], device="cuda", dtype=torch.float64)
            dist.all_reduce(t, op=dist.ReduceOp.MAX)
            hms = float(t[0])
        hms_step = hms / args.steps
        hq = {}
        for q in queries:
            kms = hk[q][0] / args.steps
            hq[q] = {"k1_ms": round(kms, 4),
                     "k1_frac_of_peak": n_mine * B[q] / (kms / 1e3) / 1e9 / peak if kms else None,
                     "k1_frac_moved": hk[q][1] / args.steps / (kms / 1e3) / 1e9 / peak if kms else None,
                     "k1_vs_direct_map": kms / per_query[q]["k1_ms"] if per_query[q]["k1_ms"] else None}
        hvalue = len(queries) * total_rows / (hms_step / 1e3)
        ht_path = {"value": hvalue, "unit": UNIT, "ms_per_step": hms_step,
                   "vs_direct_map": hvalue / value, "results_identical": same,
                   "layout": "open addressing, 16-byte buckets of two {key, rank} slots, load "
                             "<= 1/4, Bloom filters in shared memory (hx_build_dim_ht)",
                   "per_query": hq}
        hgr.close()
        for pl in hpl.values():
            pl.close()

    # ---- e2e through the C-ABI with HOST buffers (H2D + queries + D2H inside the clock) ---
    e2e = None
    if args.variant in ("host", "uva"):
        # the timed step already moves every input from pinned host memory (H2D ring) and
        # reads the results back: it IS the end-to-end measurement
        e2e = {"value": value, "unit": UNIT, "h2d_bytes_per_step": step_h2d // args.steps,
               "d2h_bytes_per_step": step_d2h // args.steps, "ms_per_step": ms_step,
               "path": ("plans over a HX_PLACE_HOST_PINNED fact table: H2D staging ring + K1 "
                        "per block + merge + finalize + D2H, one CUDA graph per step")
                       if args.variant == "host" else
                       ("plans over a HX_PLACE_HOST_MAPPED fact table: K1 reads pinned host "
                        "memory in place over PCIe + merge + finalize + D2H, one CUDA graph per step")}
    elif not args.no_e2e and (n_mine * 4 * len(lo_cols) > (32 << 30)
                              or world * n_mine * 4 * len(lo_cols) > (256 << 30)):
        e2e = {"value": None, "unit": UNIT, "skipped": "lineorder partitions larger than the "
               "pinned host memory the e2e leg allocates (32 GB per rank, 256 GB per node)"}
    elif not args.no_e2e:
        # the host copies of this rank's inputs, in page-locked memory (filled from the same
        # seeded generator: generated in HBM and copied down, outside the clock)
        host = {}
        for t in ("lineorder", "date", "customer", "supplier", "part"):
            host[t] = {}
            for c in (lo_cols if t == "lineorder" else ssbgen.TABLE_COLS[t]):
                n = n_mine if t == "lineorder" else ssbgen.table_rows(sz, c)
                buf = torch.empty(max(n, 1), dtype=torch.int32, pin_memory=True)
                tmp = torch.empty(max(n, 1), dtype=torch.int32, device="cuda")
                ssbgen.column_device(SEED, sz, c, tmp.data_ptr(), r0 if t == "lineorder" else 0, n,
                                     stream.cuda_stream)
                buf.copy_(tmp)
                del tmp
                host[t][c] = (buf, n)
        torch.cuda.synchronize()

        def timed(step, n, flush=None, ctxs=(ctx,)):
            step()
            if flush:
                flush()
            for c_ in ctxs:
                c_.stats(reset=True)
            if world > 1:
                dist.barrier()
            torch.cuda.synchronize()
            t0 = time.perf_counter()
            for _ in range(n):
                step()
            if flush:
                flush()
            torch.cuda.synchronize()
            dt_ = (time.perf_counter() - t0) / n
            h2d_ = d2h_ = 0
            for c_ in ctxs:
                _, a_, b_ = c_.stats(reset=True)
                h2d_, d2h_ = h2d_ + a_, d2h_ + b_
            if world > 1:
                t = torch.tensor([dt_], device="cuda", dtype=torch.float64)
                dist.all_reduce(t, op=dist.ReduceOp.MAX)
                dt_ = float(t[0])
            return dt_, h2d_ // n, d2h_ // n

        # (1) the serving pattern: device tables and prepared plans created once (outside the
        # clock), in two sets; every step copies ALL its inputs host -> HBM into one set
        # (hx_table_write, issued by a context on a copy stream), runs the 13 plans on that set
        # (one graph launch on the compute stream) and reads the 13 results back. Step i's
        # copy overlaps step i-1's pipelines (the copy waits only for the last use of its set);
        # the host reads step i-1's results after launching step i.
        cstream = torch.cuda.Stream(device=local)
        cctx = hx.Context(local, cstream.cuda_stream)
        esets = []
        for _ in range(2):
            tabs = {t: hx.load_columns(cctx, [(C[c], b_.data_ptr(), n_) for c, (b_, n_) in host[t].items()])
                    for t in host}
            torch.cuda.synchronize()
            eng_ = ssb.SsbEngine(ctx, {t: tabs[t] for t in ("date", "customer", "supplier", "part")},
                                 tabs["lineorder"])
            pl_ = {q: eng_.plan(q) for q in queries}
            od_ = [pl_[q].hp for q in queries]
            esets.append({"tabs": tabs, "plans": pl_,
                          "graph": hx.capture(ctx, lambda od_=od_: hx.plans_enqueue(ctx, od_)),
                          "done": torch.cuda.Event(), "copied": torch.cuda.Event()})
        ek, epending, eout = [0], [None], []

        def e2e_step():
            st = esets[ek[0] % 2]
            ek[0] += 1
            cstream.wait_event(st["done"])  # the previous step on this set has finished
            for t, cols_ in host.items():
                for c, (b_, n_) in cols_.items():
                    st["tabs"][t].write(C[c], b_.data_ptr(), n_)
            st["copied"].record(cstream)
            stream.wait_event(st["copied"])
            st["graph"].launch()
            st["done"].record(stream)
            e2e_flush()
            epending[0] = st

        def e2e_flush():
            if epending[0] is not None:
                eout.append([epending[0]["plans"][q].rows() for q in queries])
                epending[0] = None

        # (2) one-shot: fresh device tables every step and the unprepared calls
        def e2e_fresh_step():
            def load(t):
                return hx.load_columns(ctx, [(C[c], b_.data_ptr(), n_) for c, (b_, n_) in host[t].items()])
            d = {t: load(t) for t in ("date", "customer", "supplier", "part")}
            f = load("lineorder")
            e = ssb.SsbEngine(ctx, d, f)
            pend = [e.start(q) for q in queries]
            out = [e.finish(p_) for p_ in pend]
            for tb in list(d.values()) + [f]:
                tb.close()
            return out

        e2e_step()
        e2e_flush()
        assert eout[-1] == e2e_fresh_step()  # both paths give the same 13 results
        dt, h2d, d2h = timed(e2e_step, args.steps, flush=e2e_flush, ctxs=(ctx, cctx))
        dtf, h2df, d2hf = timed(e2e_fresh_step, max(3, args.steps // 5))
        e2e = {"value": len(queries) * total_rows / dt, "unit": UNIT,
               "h2d_bytes_per_step": h2d, "d2h_bytes_per_step": d2h, "ms_per_step": dt * 1e3,
               "path": "hx_table_write of every lineorder and dimension column (pinned host -> "
                       "HBM, on a copy stream, into one of two table sets the prepared plans "
                       "were created on) + one graph launch of the 13 plans (builds, K1, merge, "
                       "finalize, D2H) + 13 host result reads; step i's copy overlaps step "
                       "i-1's pipelines",
               "fresh": {"value": len(queries) * total_rows / dtf, "ms_per_step": dtf * 1e3,
                         "h2d_bytes_per_step": h2df, "d2h_bytes_per_step": d2hf,
                         "path": "hx_load_columns(pinned host -> new HBM tables) + 13 x "
                                 "(hx_build_dim_ht.. + hx_pipeline_probe_agg + "
                                 "hx_merge_aggregates -> host)"}}
        torch.cuda.synchronize()
        for st in esets:
            st["graph"].close()
            for pl in st["plans"].values():
                pl.close()
            for tb in st["tabs"].values():
                tb.close()
        cctx.close()

    cpu = None
    if rank == 0 and world == 1 and not args.no_cpu_baseline:
        cpu = cpu_baseline(args, world)

    if rank == 0:
        n_sms, ctas = ctx.info()
        line = {"metric": METRIC, "value": value, "unit": UNIT, "n_gpus": world,
                "steps": args.steps, "warmup": args.warmup, "ms_per_step": ms_step,
                "ms_per_step_median": statistics.median(per_step), "ms_per_step_min": min(per_step),
                "higher_is_better": True, "scaling": SCALING[0], "vs_baseline": None,
                "dtype": "int32 columns, int64 accumulate",
                "data": f"synthetic (ssbgen dbgen-shaped SSB distributions, seed {SEED}), "
                        "generated in HBM",
                "config": dict(config(args, world, n_mine, queries), plan_sets=n_sets,
                               step_overlap="host reads step i's results while the device runs "
                                            "step i+1" if n_sets == 2 else "none"),
                "hbm_gbps_per_gpu": sum(n_mine * B[q] for q in queries) / (ms_step / 1e3) / 1e9,
                "roofline": roofline, "cpu_baseline": cpu, "e2e": e2e, "clocks": clk,
                "gpu_launches": launches, "per_query": per_query, "ht_path": ht_path,
                "k1_ctas_per_sm": ctas, "n_sms": n_sms}
        print(json.dumps(line), flush=True)
    # release library objects before their context
    for pl_, _, gr_ in sets:
        if gr_ is not None:
            gr_.close()
        for pl in pl_.values():
            pl.close()
    for t in list(dims.values()) + [fact]:
        t.close()
    ctx.close()
    if world > 1:
        dist.destroy_process_group()


if __name__ == "__main__":
    main()

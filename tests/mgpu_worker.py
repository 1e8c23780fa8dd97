"""One rank of the 2-GPU NCCL test (tests/test_multigpu_gpu.py): launched by
torch.distributed.run, one process per GPU. Every rank holds its router blocks of lineorder
(range policy, ragged 4,097-row blocks) and the replicated dimensions, and the libhx
communicator carries every data-path collective (gloo only ships the NCCL unique id):
  * hx_merge_aggregates allreduce (every rank) and reduce (root 0) of the 13 queries;
  * prepared plans with their per-plan allreduce, plain and replayed from a CUDA graph;
  * hx_ht_broadcast from rank 0 into tables the other ranks built with a different filter;
  * the hash-routing exchange (NCCL send/recv) of the hash-partitioned join, with the
    dimension replicated and with it partitioned across the ranks (both inputs exchanged);
  * host-resident lineorder in one shared pinned buffer, blocks drawn from a shared router
    (dynamic load balancing across the ranks).
Results are compared bit-exactly with the oracle over the WHOLE table."""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import torch  # noqa: E402
import torch.distributed as dist  # noqa: E402

import oracle  # noqa: E402
import ssbgen  # noqa: E402
from paper_journals_pvldb_chrysogeloskaa19_b200 import hx, ssb  # noqa: E402


def main():
    rank, world = int(os.environ["RANK"]), int(os.environ["WORLD_SIZE"])
    torch.cuda.set_device(rank)
    dist.init_process_group("gloo")
    uid = [hx.comm_unique_id() if rank == 0 else None]
    dist.broadcast_object_list(uid, src=0)
    ctx = hx.Context(rank)
    ctx.comm_init(world, rank, uid[0])
    assert ctx.comm_info() == (rank, world)
    db = ssbgen.database(7, ssbgen.sizes(0.02))
    want = {q: oracle.run_query(q, db) for q in ssb.QUERIES}
    part = hx.router_partition(len(db["lineorder"]["lo_orderdate"]), world, 4097)
    dims, fact = ssb.load_db_numpy(ctx, db, part, rank)
    eng = ssb.SsbEngine(ctx, dims, fact)
    assert fact.n_rows == part.rows(rank)
    fails = []

    def check(tag, got, q):
        if got != want[q]:
            fails.append(f"rank {rank} {tag} {q}: {got[:2]} vs {want[q][:2]}")

    for q in ssb.QUERIES:  # union router: allreduce on every rank
        check("allreduce", eng.run(q), q)
    for q in ssb.QUERIES:  # reduce to root 0
        rows = eng.finish(eng.start(q), 0)
        if rank == 0:
            check("reduce", rows, q)
    plans = {q: eng.plan(q) for q in ssb.QUERIES}
    order = [plans[q].hp for q in ssb.QUERIES]
    ctx.comm_trace(reset=True)
    hx.plans_enqueue(ctx, order)
    for q in ssb.QUERIES:
        check("plans", plans[q].rows(), q)
    counts = torch.tensor([r["count"] for r in ctx.comm_trace(reset=True)], dtype=torch.int64)
    other = counts.clone()
    dist.broadcast(other, src=0)
    if not torch.equal(counts, other):
        fails.append(f"rank {rank}: per-plan allreduce counts differ from rank 0's")
    graph = hx.capture(ctx, lambda: hx.plans_enqueue(ctx, order))
    for _ in range(2):
        graph.launch()
        for q in ssb.QUERIES:
            check("graph", plans[q].rows(), q)
    graph.close()
    for pl in plans.values():
        pl.close()
    for q in ("q2.1", "q3.2", "q4.3"):  # HT broadcast from rank 0
        plan = ssb.PLANS[q]
        hts = []
        for _, b in plan.joins:
            if rank != 0 and b.preds:  # a different filter: broadcast must overwrite it
                b = ssb.DimBuild(b.table, b.key, [], b.group)
            hts.append(eng.build(b))
        for t in hts:
            t.broadcast(0)
        agg = hx.pipeline_probe_agg(ctx, fact, eng.shape(plan), hts)
        check("ht_broadcast", eng.finish(ssb.Pending(plan, hts, agg)), q)
    for q, dim in (("q2.1", "part"), ("q3.1", "customer"), ("q4.3", "supplier")):
        check(f"hash_routed[{dim}]", eng.run_hash_routed(q, dim), q)
        # the dimension partitioned too (rows r, r + world, ... on rank r): both inputs are
        # hash-packed and exchanged
        mine = {c: v[rank::world] for c, v in db[dim].items()}
        local = hx.load_numpy(ctx, {ssbgen.COLS[c]: v for c, v in mine.items()})
        check(f"hash_routed_partitioned[{dim}]", eng.run_hash_routed(q, dim, dim_local=local), q)
        local.close()
    # host-resident lineorder in ONE shared pinned buffer (every rank maps it), blocks handed
    # out by the shared router: each block runs on exactly one GPU, whichever drew it
    from multiprocessing import shared_memory

    import numpy as np
    lo = db["lineorder"]
    n = len(lo["lo_orderdate"])
    names = list(lo)
    shm_name = f"hx_mgpu_lo_{os.environ.get('MASTER_PORT', '0')}"
    if rank == 0:
        shm = shared_memory.SharedMemory(name=shm_name, create=True, size=4 * n * len(names))
        buf = np.ndarray((len(names), n), dtype=np.int32, buffer=shm.buf)
        for i, c in enumerate(names):
            buf[i] = lo[c]
        router = hx.SharedRouter(f"/{shm_name}_r", (n + 8191) // 8192, create=True)
    dist.barrier()
    if rank != 0:
        shm = shared_memory.SharedMemory(name=shm_name)
        buf = np.ndarray((len(names), n), dtype=np.int32, buffer=shm.buf)
        router = hx.SharedRouter(f"/{shm_name}_r", (n + 8191) // 8192, create=False)
    ptr = buf.ctypes.data
    assert torch.cuda.cudart().cudaHostRegister(ptr, buf.nbytes, 1) == 0  # portable
    hfact = hx.load_columns(ctx, [(ssbgen.COLS[c], ptr + 4 * n * i, n) for i, c in enumerate(names)],
                            placement=hx._hx.HX_PLACE_HOST_PINNED)
    heng = ssb.SsbEngine(ctx, dims, hfact)
    for q in ("q1.1", "q2.1", "q3.1", "q4.1"):
        if rank == 0:
            router.reset()
        dist.barrier()
        rows, nb = heng.run_routed(q, router, 8192)
        check("shared_router", rows, q)
        tot = torch.tensor([nb], dtype=torch.int64)
        dist.all_reduce(tot)
        if int(tot[0]) != (n + 8191) // 8192:
            fails.append(f"rank {rank} shared_router {q}: {int(tot[0])} blocks ran")
        dist.barrier()
    hfact.close()
    torch.cuda.cudart().cudaHostUnregister(ptr)
    router.close(unlink=(rank == 0))
    dist.barrier()
    del buf
    shm.close()
    if rank == 0:
        shm.unlink()
    for t in list(dims.values()) + [fact]:
        t.close()
    ctx.close()
    flag = torch.tensor([len(fails)], dtype=torch.int64)
    dist.all_reduce(flag)
    for f in fails:
        print(f, flush=True)
    dist.destroy_process_group()
    if int(flag[0]):
        sys.exit(1)
    print(f"rank {rank}: OK", flush=True)


if __name__ == "__main__":
    main()

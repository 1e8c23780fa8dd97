// hx_plan.cu — prepared query plans and CUDA-graph capture (the native runtime around K1/K2).
//
// PAPER.md:769-790 §4.1: a query is split into pipelines that are compiled once and then
// executed; §4.2: parallelism and affinity are fixed when the pipeline
// instances are created; §4.3: memory is pre-allocated at initialisation
// so that query execution does not allocate. A plan is that for one SSB query on one GPU:
// creation validates the shape, allocates every buffer (hash tables, group arrays, result
// buffer in pinned host memory) and runs the builds once to size the group arrays exactly;
// execution (hx_plan_enqueue) is then one asynchronous, allocation-free, sync-free sequence
//   K2 builds -> K1 prepare -> K1 -> [NCCL allreduce of the partials] -> finalize -> D2H
// that a CUDA graph can capture, so a whole SSB step replays with one launch.
#include <cub/block/block_scan.cuh>

#include <algorithm>
#include <cstdlib>
#include <cstring>

#include "hx_internal.cuh"

namespace hx {
namespace {

constexpr int kOutInline = 4096;  // result rows copied to the host by every execution
constexpr int64_t kDirectMaxBytes = int64_t(16) << 20;  // direct maps up to 16 MB (L2: 126 MB)

struct OutHeader {
  long long n_rows;
  long long n_groups;
  int32_t error;
  int32_t n_gdims;
  long long n_pass;  // rows that passed every join (sum of the group counts)
  int32_t pad[8];
};
static_assert(sizeof(OutHeader) == 64, "OutHeader is 64 bytes");

struct OutRow {
  long long sum;
  long long cnt;
  int32_t key[HX_MAX_GDIMS];
  int32_t pad;
};
static_assert(sizeof(OutRow) == 32, "OutRow is 32 bytes");

struct FinalizeArgs {
  const AggMeta* meta;
  const unsigned long long* sums;
  const unsigned long long* cnts;
  int32_t n_gdims;
  const int32_t* r2c[HX_MAX_GDIMS];       // nullptr: membership-only dimension (code 0)
  const HtHeader* deps[HX_MAX_JOINS];
  int32_t n_deps;
  long long expect_groups;                 // the plan's group count (-1: any)
  OutHeader* hdr;
  OutRow* rows;
  long long out_cap;
};

// a7 Finalize on the device: ordered compaction of the non-empty groups (a query without
// GROUP BY keeps its one row) and decoding of each group index into dictionary codes.
__global__ void k1_finalize(FinalizeArgs a) {
  using Scan = cub::BlockScan<int, 1024>;
  __shared__ typename Scan::TempStorage tmp;
  __shared__ long long running;
  __shared__ unsigned long long n_pass;
  const long long n = a.meta->n_groups;
  int err = a.meta->error;
  for (int d = 0; d < a.n_deps && !err; ++d) err = a.deps[d]->error;
  if (!err && a.expect_groups >= 0 && n != a.expect_groups) err = HX_ECAPACITY;
  if (threadIdx.x == 0) {
    running = 0;
    n_pass = 0;
  }
  __syncthreads();
  if (!err) {
    for (long long base = 0; base < n; base += 1024) {
      const long long g = base + threadIdx.x;
      if (g < n && a.cnts[g]) atomicAdd(&n_pass, a.cnts[g]);
      const int flag = g < n && (a.n_gdims == 0 || a.cnts[g] > 0);
      int excl, total;
      Scan(tmp).ExclusiveSum(flag, excl, total);
      const long long pos = running + excl;
      if (flag && pos < a.out_cap) {
        OutRow r{};
        r.sum = (long long)a.sums[g];
        r.cnt = (long long)a.cnts[g];
        long long rem = g;
        for (int d = a.n_gdims - 1; d >= 0; --d) {
          const long long nr = a.meta->n_ranks[d] > 0 ? a.meta->n_ranks[d] : 1;
          const int rank = (int)(rem % nr);
          rem /= nr;
          r.key[d] = a.r2c[d] ? a.r2c[d][rank] : 0;
        }
        a.rows[pos] = r;
      }
      __syncthreads();
      if (threadIdx.x == 0) running += total;
      __syncthreads();
    }
  }
  if (threadIdx.x == 0) {
    OutHeader h{};
    h.n_rows = err ? 0 : running;
    h.n_groups = n;
    h.error = err;
    h.n_gdims = a.n_gdims;
    h.n_pass = err ? 0 : (long long)n_pass;
    *a.hdr = h;
  }
}

}  // namespace
}  // namespace hx

using namespace hx;

struct hx_plan {
  hx_ctx* ctx = nullptr;
  std::vector<hx_ht*> hts;
  hx_agg agg;
  K1Prepared* k1 = nullptr;
  long long n_groups = 1;
  FinalizeArgs fin{};
  void* d_out = nullptr;
  void* h_out = nullptr;       // pinned
  size_t out_bytes = 0, inline_bytes = 0;
  cudaEvent_t done = nullptr, k1_e0 = nullptr, k1_e1 = nullptr;
  cudaEvent_t probed = nullptr;  // K1 (+ merge) complete: the finalize branch forks here
  cudaEvent_t built_ev[hx_ctx::kAux] = {nullptr, nullptr, nullptr, nullptr};
  StageRing* ring = nullptr;   // host-resident fact table: the mem-move staging ring
  bool enqueued = false;
};

struct hx_graph {
  hx_ctx* ctx = nullptr;
  cudaGraph_t graph = nullptr;
  cudaGraphExec_t exec = nullptr;
  int64_t launches = 0;
  int64_t d2h = 0, h2d = 0;
};

static int plan_enqueue_builds(hx_ctx* ctx, hx_plan* pl);
static int plan_enqueue_probe(hx_ctx* ctx, hx_plan* pl, bool merge = true);
static int plan_enqueue_finish(hx_ctx* ctx, hx_plan* pl, bool on_fin = false);
static int join_fin(hx_ctx* ctx);

static void plan_destroy(hx_plan* pl) {
  if (!pl) return;
  cudaSetDevice(pl->ctx->device);
  cudaStreamSynchronize(pl->ctx->stream);
  for (hx_ht* t : pl->hts) ht_destroy(t);
  if (pl->agg.base) cudaFreeAsync(pl->agg.base, pl->ctx->stream);
  if (pl->k1) k1_free(pl->k1);
  ring_destroy(pl->ctx, pl->ring);
  if (pl->d_out) cudaFreeAsync(pl->d_out, pl->ctx->stream);
  if (pl->h_out) cudaFreeHost(pl->h_out);
  for (cudaEvent_t e : {pl->done, pl->k1_e0, pl->k1_e1, pl->probed})
    if (e) cudaEventDestroy(e);
  for (cudaEvent_t e : pl->built_ev)
    if (e) cudaEventDestroy(e);
  delete pl;
}

extern "C" {

int hx_plan_create(hx_ctx* ctx, const hx_table* fact, hx_table* const* dims, int n_dims,
                   const hx_build_spec* builds, int n_builds, const hx_query_shape* shape,
                   hx_plan** out) {
  HX_REQUIRE(ctx && fact && shape && out && (n_builds == 0 || (builds && dims)), HX_EINVAL,
             "hx_plan_create: null argument");
  HX_REQUIRE(n_builds >= 0 && n_builds <= HX_MAX_JOINS, HX_EINVAL, "hx_plan_create: bad n_builds");
  HX_CK(cudaSetDevice(ctx->device));
  hx_plan* pl = new hx_plan();
  pl->ctx = ctx;
  pl->agg.ctx = ctx;
  auto bail = [&](int rc) {
    plan_destroy(pl);
    return rc;
  };
  // 1) hash tables: allocate, build once
  for (int b = 0; b < n_builds; ++b) {
    const hx_build_spec& s = builds[b];
    if (s.dim < 0 || s.dim >= n_dims || !dims[s.dim] || s.n_preds < 0 || s.n_preds > HX_MAX_PREDS)
      return bail(fail(HX_EINVAL, "hx_plan_create: bad build spec"));
    hx_ht* ht = nullptr;
    int rc = ht_create(ctx, dims[s.dim], s.key_col, s.preds, s.n_preds, s.group_col, s.group_lo,
                       s.group_hi, &ht);
    if (rc != HX_OK) return bail(rc);
    pl->hts.push_back(ht);
    rc = ht_enqueue_build(ctx, ht);
    if (rc != HX_OK) return bail(rc);
  }
  // 2) exact group count from the built tables (the plan's one synchronisation)
  const long long bound = k1_group_bound(shape, pl->hts.data(), n_builds);
  if (bound < 1 || shape->n_joins > HX_MAX_JOINS || shape->n_gdims > HX_MAX_GDIMS)
    return bail(fail(HX_EINVAL, "hx_plan_create: bad gdim_join / join_ht"));
  std::vector<HtHeader> hh(n_builds);
  for (int b = 0; b < n_builds; ++b) {
    cudaError_t e = cudaMemcpyAsync(&hh[b], pl->hts[b]->hdr, sizeof(HtHeader),
                                    cudaMemcpyDeviceToHost, ctx->stream);
    if (e != cudaSuccess) return bail(cuda_fail(e, "cudaMemcpyAsync", __FILE__, __LINE__));
  }
  {
    cudaError_t e = cudaStreamSynchronize(ctx->stream);
    if (e != cudaSuccess) return bail(cuda_fail(e, "cudaStreamSynchronize", __FILE__, __LINE__));
  }
  for (int b = 0; b < n_builds; ++b) {
    if (hh[b].error == HX_EDUPKEY) return bail(fail(HX_EDUPKEY, "dimension build: duplicate primary key"));
    if (hh[b].error) return bail(fail(HX_EINVAL, "dimension build: bad key or group code"));
    pl->hts[b]->known_keys = hh[b].n_keys;  // lets K1 reserve shared memory for its filter
  }
  // dense keys (R20): the plan's builds produce direct maps over the passing-key
  // range instead of hash tables when the map is no larger than kDirectMaxBytes (or than
  // twice the hash table); HX_NO_DM=1 keeps hash tables (A/B measurements, tests)
  // (all builds or none: one K1 instance probes either kind)
  bool use_dm = std::getenv("HX_NO_DM") == nullptr && ctx->join_layout == HX_JOIN_AUTO;
  int32_t dm_kmin[HX_MAX_JOINS] = {0, 0, 0, 0};
  int64_t dm_span[HX_MAX_JOINS] = {0, 0, 0, 0};
  int dm_lw[HX_MAX_JOINS] = {0, 0, 0, 0};
  for (int b = 0; b < n_builds && use_dm; ++b) {
    hx_ht* ht = pl->hts[b];
    const HtHeader& h = hh[b];
    int64_t kmin = 0, span = 0;
    if (h.n_keys > 0) {
      kmin = key_dec(~h.kmin_inv);
      span = (int64_t)key_dec(h.kmax_enc) - kmin + 1;
    }
    const int64_t values = ht->has_group ? std::max(1, h.n_ranks) : 1;
    int lw = 0;
    while (lw < 5 && (int64_t)dm_vmask(lw) < values) ++lw;
    const int64_t dm_bytes = dm_words_for(span, lw) * 4;
    const int64_t ht_bytes = (int64_t(1) << h.log2cap) * 8;
    if (span >= (int64_t(1) << 27) || dm_bytes > std::max<int64_t>(kDirectMaxBytes, 2 * ht_bytes))
      use_dm = false;
    dm_kmin[b] = (int32_t)kmin;
    dm_span[b] = span;
    dm_lw[b] = lw;
  }
  for (int b = 0; b < n_builds && use_dm; ++b) {
    int rc = ht_enable_direct(ctx, pl->hts[b], dm_kmin[b], (uint32_t)dm_span[b], dm_lw[b]);
    if (rc != HX_OK) return bail(rc);
  }
  long long ng = 1;
  for (int g = 0; g < shape->n_gdims; ++g) ng *= std::max(1, hh[shape->join_ht[shape->gdim_join[g]]].n_ranks);
  if (ng > HX_MAX_GROUPS) return bail(fail(HX_ECAPACITY, "hx_plan_create: too many groups"));
  pl->n_groups = ng;
  int rc = agg_alloc(ctx, &pl->agg, ng, shape, pl->hts.data());
  if (rc != HX_OK) return bail(rc);
  for (int j = 0; j < shape->n_joins; ++j) pl->agg.deps.push_back(pl->hts[shape->join_ht[j]]);
  // 3) the K1 launch
  rc = k1_setup(ctx, fact, shape, pl->hts.data(), n_builds, &pl->agg, &pl->k1);
  if (rc != HX_OK) return bail(rc);
  if (k1_is_host(pl->k1) && fact->n_rows > 0) {
    rc = ring_create(ctx, pl->k1, kHostBlockRows, &pl->ring);
    if (rc != HX_OK) return bail(rc);
  }
  // 4) result buffers
  pl->out_bytes = sizeof(OutHeader) + (size_t)ng * sizeof(OutRow);
  pl->inline_bytes = sizeof(OutHeader) + (size_t)std::min<long long>(ng, kOutInline) * sizeof(OutRow);
  HX_CK(cudaMallocAsync(&pl->d_out, pl->out_bytes, ctx->stream));
  {
    cudaError_t e = cudaMallocHost(&pl->h_out, pl->inline_bytes);
    if (e != cudaSuccess) return bail(cuda_fail(e, "cudaMallocHost", __FILE__, __LINE__));
  }
  FinalizeArgs& f = pl->fin;
  f.meta = pl->agg.meta;
  f.sums = pl->agg.sums;
  f.cnts = pl->agg.cnts;
  f.n_gdims = shape->n_gdims;
  for (int g = 0; g < shape->n_gdims; ++g) {
    const hx_ht* ht = pl->agg.gdim_ht[g];
    f.r2c[g] = ht->has_group ? ht->rank_to_code : nullptr;
  }
  f.n_deps = (int)pl->agg.deps.size();
  for (int d = 0; d < f.n_deps; ++d) f.deps[d] = pl->agg.deps[d]->hdr;
  f.expect_groups = ng;
  f.hdr = static_cast<OutHeader*>(pl->d_out);
  f.rows = reinterpret_cast<OutRow*>(f.hdr + 1);
  f.out_cap = ng;
  for (cudaEvent_t* e : {&pl->done, &pl->k1_e0, &pl->k1_e1}) {
    cudaError_t err = cudaEventCreate(e);
    if (err != cudaSuccess) return bail(cuda_fail(err, "cudaEventCreate", __FILE__, __LINE__));
  }
  for (cudaEvent_t& e : pl->built_ev) {
    cudaError_t err = cudaEventCreateWithFlags(&e, cudaEventDisableTiming);
    if (err != cudaSuccess) return bail(cuda_fail(err, "cudaEventCreate", __FILE__, __LINE__));
  }
  {
    cudaError_t err = cudaEventCreateWithFlags(&pl->probed, cudaEventDisableTiming);
    if (err != cudaSuccess) return bail(cuda_fail(err, "cudaEventCreate", __FILE__, __LINE__));
  }
  *out = pl;
  return HX_OK;
}

int hx_plan_enqueue(hx_ctx* ctx, hx_plan* pl) {
  HX_REQUIRE(ctx && pl && pl->ctx == ctx, HX_EINVAL, "hx_plan_enqueue: bad argument");
  HX_CK(cudaSetDevice(ctx->device));
  HX_CK(cudaEventRecord(ctx->fork_ev, ctx->stream));
  for (int a = 0; a < hx_ctx::kAux; ++a) HX_CK(cudaStreamWaitEvent(ctx->aux[a], ctx->fork_ev, 0));
  int rc = plan_enqueue_builds(ctx, pl);
  if (rc != HX_OK) return rc;
  rc = plan_enqueue_probe(ctx, pl);
  if (rc != HX_OK) return rc;
  return join_fin(ctx);
}

int hx_plans_enqueue(hx_ctx* ctx, hx_plan* const* plans, int n) {
  HX_REQUIRE(ctx && (n == 0 || plans) && n >= 0, HX_EINVAL, "hx_plans_enqueue: bad argument");
  for (int i = 0; i < n; ++i)
    HX_REQUIRE(plans[i] && plans[i]->ctx == ctx, HX_EINVAL, "hx_plans_enqueue: bad plan");
  HX_CK(cudaSetDevice(ctx->device));
  // every build of every plan first (forked from one point: they overlap the pipelines of
  // the earlier plans), then the pipelines in order, each waiting only for its own builds
  HX_CK(cudaEventRecord(ctx->fork_ev, ctx->stream));
  for (int a = 0; a < hx_ctx::kAux; ++a) HX_CK(cudaStreamWaitEvent(ctx->aux[a], ctx->fork_ev, 0));
  for (int i = 0; i < n; ++i) {
    int rc = plan_enqueue_builds(ctx, plans[i]);
    if (rc != HX_OK) return rc;
  }
  if (std::getenv("HX_SERIAL_BUILDS")) {  // A/B: every build done before the first pipeline
    for (int i = 0; i < n; ++i) HX_CK(cudaStreamWaitEvent(ctx->stream, plans[i]->built_ev[0], 0));
  }
  // > 1 rank: each plan's union-router allreduce runs on the finalize stream, overlapping
  // the next pipelines (HX_GROUPED_MERGE: one grouped NCCL launch after the last pipeline
  // instead — measured 2.87 vs 2.64 ms per SF10 step with a 1-rank communicator: the
  // finalizes then no longer overlap the pipelines)
  static const bool grouped_env = std::getenv("HX_GROUPED_MERGE") != nullptr;  // A/B
  const bool grouped = grouped_env && use_collectives(ctx) && n > 1;
  for (int i = 0; i < n; ++i) {
    int rc = plan_enqueue_probe(ctx, plans[i], /*merge=*/!grouped);
    if (rc != HX_OK) return rc;
  }
  if (grouped) {
    HX_REQUIRE(ncclGroupStart() == ncclSuccess, HX_ENCCL, "ncclGroupStart");
    for (int i = 0; i < n; ++i) {
      coll_log(ctx, HX_COLL_ALLREDUCE, plans[i]->agg.sums, 2 * (int64_t)plans[i]->n_groups, 8);
      ncclResult_t r = ncclAllReduce(plans[i]->agg.sums, plans[i]->agg.sums,
                                     2 * (size_t)plans[i]->n_groups, ncclUint64, ncclSum,
                                     ctx->comm, ctx->stream);
      if (r != ncclSuccess) {
        ncclGroupEnd();
        return fail(HX_ENCCL, std::string("ncclAllReduce: ") + ncclGetErrorString(r));
      }
    }
    ncclResult_t r = ncclGroupEnd();
    HX_REQUIRE(r == ncclSuccess, HX_ENCCL, std::string("ncclGroupEnd: ") + ncclGetErrorString(r));
    for (int i = 0; i < n; ++i) {
      int rc = plan_enqueue_finish(ctx, plans[i]);
      if (rc != HX_OK) return rc;
    }
  }
  return n > 0 ? join_fin(ctx) : HX_OK;
}

}  // extern "C"

// builds of one plan on the auxiliary streams (which must already follow the main stream's
// fork point), then K1's prepare on aux[0] once all of them are done: built_ev[0] marks the
// plan ready for its K1, and none of this sits on the main stream between two K1 launches
static int plan_enqueue_builds(hx_ctx* ctx, hx_plan* pl) {
  const int nb = (int)pl->hts.size();
  for (int b = 0; b < nb; ++b) {
    int rc = ht_enqueue_build(ctx, pl->hts[b], ctx->aux[b % hx_ctx::kAux]);
    if (rc != HX_OK) return rc;
  }
  for (int a = 1; a < std::min(nb, (int)hx_ctx::kAux); ++a) {
    HX_CK(cudaEventRecord(pl->built_ev[a], ctx->aux[a]));
    HX_CK(cudaStreamWaitEvent(ctx->aux[0], pl->built_ev[a], 0));
  }
  int rc = k1_enqueue_prepare(ctx, pl->k1, true, ctx->aux[0]);
  if (rc != HX_OK) return rc;
  HX_CK(cudaEventRecord(pl->built_ev[0], ctx->aux[0]));
  return HX_OK;
}

// K1 (after the plan's builds) -> merge on the main stream; finalize -> D2H on the finalize
// stream, so the next plan's K1 starts as soon as this one's merge is done
static int plan_enqueue_probe(hx_ctx* ctx, hx_plan* pl, bool merge) {
  HX_CK(cudaStreamWaitEvent(ctx->stream, pl->built_ev[0], 0));
  int rc = k1_enqueue(ctx, pl->k1, true, pl->k1_e0, pl->k1_e1, pl->ring, /*prepare=*/false);
  if (rc != HX_OK) return rc;
  if (!merge) return HX_OK;  // the caller merges (grouped) and finishes
  if (use_collectives(ctx)) {
    // union router: partial {sum,cnt} arrays are adjacent, one allreduce over NVLink — on the
    // finalize stream, so the next plan's K1 does not wait for the collective
    HX_CK(cudaEventRecord(pl->probed, ctx->stream));
    HX_CK(cudaStreamWaitEvent(ctx->fin_stream, pl->probed, 0));
    coll_log(ctx, HX_COLL_ALLREDUCE, pl->agg.sums, 2 * (int64_t)pl->n_groups, 8);
    ncclResult_t r = ncclAllReduce(pl->agg.sums, pl->agg.sums, 2 * (size_t)pl->n_groups,
                                   ncclUint64, ncclSum, ctx->comm, ctx->fin_stream);
    HX_REQUIRE(r == ncclSuccess, HX_ENCCL, std::string("ncclAllReduce: ") + ncclGetErrorString(r));
    return plan_enqueue_finish(ctx, pl, /*on_fin=*/true);
  }
  return plan_enqueue_finish(ctx, pl);
}

// after the (merged) group arrays are final on the main stream: finalize -> D2H on the
// finalize stream
static int plan_enqueue_finish(hx_ctx* ctx, hx_plan* pl, bool on_fin) {
  if (!on_fin) {  // the group arrays are final on the main stream
    HX_CK(cudaEventRecord(pl->probed, ctx->stream));
    HX_CK(cudaStreamWaitEvent(ctx->fin_stream, pl->probed, 0));
  }
  k1_finalize<<<1, 1024, 0, ctx->fin_stream>>>(pl->fin);
  HX_CK_LAUNCH("k1_finalize");
  ctx->launches += 1;
  HX_CK(cudaMemcpyAsync(pl->h_out, pl->d_out, pl->inline_bytes, cudaMemcpyDeviceToHost,
                        ctx->fin_stream));
  ctx->d2h_bytes += (int64_t)pl->inline_bytes;
  HX_CK(record_event(pl->done, ctx->fin_stream));
  pl->enqueued = true;
  return HX_OK;
}

// the main stream waits for every finalize enqueued so far (a later execution of the same
// plan must not overwrite its group arrays before they are read; graph capture needs the join)
static int join_fin(hx_ctx* ctx) {
  HX_CK(cudaEventRecord(ctx->fin_join_ev, ctx->fin_stream));
  HX_CK(cudaStreamWaitEvent(ctx->stream, ctx->fin_join_ev, 0));
  return HX_OK;
}

extern "C" {

int hx_plan_result(hx_plan* pl, int64_t* sums, int64_t* counts, int32_t* keys, int64_t cap,
                   int64_t* n_rows) {
  HX_REQUIRE(pl && n_rows && cap >= 0 && (cap == 0 || (sums && counts)), HX_EINVAL,
             "hx_plan_result: bad argument");
  HX_REQUIRE(pl->enqueued, HX_EINVAL, "hx_plan_result: plan never executed");
  HX_CK(cudaSetDevice(pl->ctx->device));
  HX_CK(cudaEventSynchronize(pl->done));
  const OutHeader* h = static_cast<const OutHeader*>(pl->h_out);
  *n_rows = 0;
  if (h->error == HX_EDUPKEY) return fail(HX_EDUPKEY, "dimension build: duplicate primary key");
  if (h->error == HX_ECAPACITY)
    return fail(HX_ECAPACITY, "hx_plan: group count changed since the plan was created");
  if (h->error) return fail(HX_EINVAL, "dimension build: bad key or group code");
  const int64_t n = h->n_rows;
  *n_rows = n;
  if (n > cap) return fail(HX_ECAPACITY, "hx_plan_result: output buffer too small");
  const OutRow* rows = reinterpret_cast<const OutRow*>(h + 1);
  std::vector<OutRow> rest;
  if (n > kOutInline) {  // large results: the rows beyond the inline block
    rest.resize(n - kOutInline);
    HX_CK(cudaMemcpy(rest.data(), pl->fin.rows + kOutInline, rest.size() * sizeof(OutRow),
                     cudaMemcpyDeviceToHost));
  }
  const int nd = pl->fin.n_gdims;
  for (int64_t i = 0; i < n; ++i) {
    const OutRow& r = i < kOutInline ? rows[i] : rest[i - kOutInline];
    sums[i] = r.sum;
    counts[i] = r.cnt;
    for (int d = 0; d < nd; ++d) keys[i * nd + d] = r.key[d];
  }
  return HX_OK;
}

int hx_plan_k1_time(hx_plan* pl, float* ms, int64_t* bytes) {
  HX_REQUIRE(pl && pl->enqueued, HX_EINVAL, "hx_plan_k1_time: plan never executed");
  HX_CK(cudaEventSynchronize(pl->done));
  if (ms) {
    *ms = 0.f;
    if (pl->k1_e0 && k1_bytes(pl->k1) > 0) HX_CK(cudaEventElapsedTime(ms, pl->k1_e0, pl->k1_e1));
  }
  if (bytes) {  // streamed columns + one 32-byte sector per gathered value
    const OutHeader* h = static_cast<const OutHeader*>(pl->h_out);
    *bytes = k1_bytes(pl->k1) + h->n_pass * 32 * k1_gathered_cols(pl->k1);
  }
  return HX_OK;
}

int hx_plan_k1_span(hx_plan* first, hx_plan* last, float* ms) {
  HX_REQUIRE(first && last && ms && first->enqueued && last->enqueued && first->ctx == last->ctx,
             HX_EINVAL, "hx_plan_k1_span: bad argument");
  HX_REQUIRE(k1_bytes(first->k1) > 0 && k1_bytes(last->k1) > 0, HX_EINVAL,
             "hx_plan_k1_span: a plan without K1 launch");
  HX_CK(cudaEventSynchronize(last->done));
  HX_CK(cudaEventElapsedTime(ms, first->k1_e0, last->k1_e1));
  return HX_OK;
}

int hx_plan_info(hx_plan* pl, int64_t* n_groups, int* n_gdims) {
  HX_REQUIRE(pl, HX_EINVAL, "hx_plan_info: null plan");
  if (n_groups) *n_groups = pl->n_groups;
  if (n_gdims) *n_gdims = pl->fin.n_gdims;
  return HX_OK;
}

int hx_plan_free(hx_plan* pl) {
  HX_REQUIRE(pl, HX_EINVAL, "hx_plan_free: null plan");
  plan_destroy(pl);
  return HX_OK;
}

// ---- CUDA graphs ---------------------------------------------------------------------------
int hx_graph_begin(hx_ctx* ctx) {
  HX_REQUIRE(ctx, HX_EINVAL, "hx_graph_begin: null ctx");
  HX_CK(cudaSetDevice(ctx->device));
  ctx->capture_launches = ctx->launches;
  ctx->capture_d2h = ctx->d2h_bytes;
  ctx->capture_h2d = ctx->h2d_bytes;
  HX_CK(cudaStreamBeginCapture(ctx->stream, cudaStreamCaptureModeThreadLocal));
  return HX_OK;
}

int hx_graph_end(hx_ctx* ctx, hx_graph** out) {
  HX_REQUIRE(ctx && out, HX_EINVAL, "hx_graph_end: null argument");
  HX_CK(cudaSetDevice(ctx->device));
  hx_graph* g = new hx_graph();
  g->ctx = ctx;
  cudaError_t e = cudaStreamEndCapture(ctx->stream, &g->graph);
  // node priorities (K1's launch priority) are honoured only with this flag
  if (e == cudaSuccess)
    e = cudaGraphInstantiateWithFlags(&g->exec, g->graph, cudaGraphInstantiateFlagUseNodePriority);
  g->launches = ctx->launches - ctx->capture_launches;
  ctx->launches = ctx->capture_launches;  // captured, not executed
  g->d2h = ctx->d2h_bytes - ctx->capture_d2h;
  ctx->d2h_bytes = ctx->capture_d2h;
  g->h2d = ctx->h2d_bytes - ctx->capture_h2d;
  ctx->h2d_bytes = ctx->capture_h2d;
  if (e != cudaSuccess) {
    if (g->graph) cudaGraphDestroy(g->graph);
    delete g;
    return cuda_fail(e, "cudaStreamEndCapture/cudaGraphInstantiate", __FILE__, __LINE__);
  }
  *out = g;
  return HX_OK;
}

int hx_graph_launch(hx_ctx* ctx, hx_graph* g) {
  HX_REQUIRE(ctx && g && g->ctx == ctx, HX_EINVAL, "hx_graph_launch: bad argument");
  HX_CK(cudaSetDevice(ctx->device));
  HX_CK(cudaGraphLaunch(g->exec, ctx->stream));
  ctx->launches += g->launches;
  ctx->d2h_bytes += g->d2h;
  ctx->h2d_bytes += g->h2d;
  return HX_OK;
}

int hx_graph_free(hx_graph* g) {
  HX_REQUIRE(g, HX_EINVAL, "hx_graph_free: null graph");
  cudaSetDevice(g->ctx->device);
  if (g->exec) cudaGraphExecDestroy(g->exec);
  if (g->graph) cudaGraphDestroy(g->graph);
  delete g;
  return HX_OK;
}

}  // extern "C"

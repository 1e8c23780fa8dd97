// hx_api.cu — the C-ABI entry points of libhx (include/hx.h): context, communicator,
// router, mem-move (column placement), hash-table objects, pipeline launch, union-router
// merge and measurement. The kernels live in hx_build.cu (K2) and hx_probe.cu (K1).
#include <algorithm>
#include <cstdlib>
#include <cstring>
#include <string>

#include "hx_internal.cuh"

namespace hx {

static thread_local std::string g_last_error;

void set_error(const std::string& msg) { g_last_error = msg; }

int fail(int code, const std::string& msg) {
  g_last_error = msg;
  return code;
}

int cuda_fail(cudaError_t e, const char* what, const char* file, int line) {
  g_last_error = std::string(what) + ": " + cudaGetErrorString(e) + " (" + file + ":" +
                 std::to_string(line) + ")";
  return e == cudaErrorMemoryAllocation ? HX_ENOMEM : HX_ECUDA;
}

static int nccl_fail(ncclResult_t r, const char* what) {
  g_last_error = std::string(what) + ": " + ncclGetErrorString(r);
  return HX_ENCCL;
}

#define HX_NCCL(call)                                   \
  do {                                                  \
    ncclResult_t _r = (call);                           \
    if (_r != ncclSuccess) return ::hx::nccl_fail(_r, #call); \
  } while (0)

const int32_t* table_col(const hx_table* t, int32_t col_id) {
  for (int i = 0; i < t->n_cols; ++i)
    if (t->col_id[i] == col_id) return t->dev[i];
  return nullptr;
}

bool table_has_col(const hx_table* t, int32_t col_id) {
  for (int i = 0; i < t->n_cols; ++i)
    if (t->col_id[i] == col_id) return true;
  return false;
}

cudaEvent_t pooled_event(hx_ctx* ctx) {
  if (!ctx->event_pool.empty()) {
    cudaEvent_t e = ctx->event_pool.back();
    ctx->event_pool.pop_back();
    return e;
  }
  cudaEvent_t e = nullptr;
  cudaEventCreate(&e);
  return e;
}

}  // namespace hx

using namespace hx;

extern "C" {

const char* hx_last_error(void) { return g_last_error.c_str(); }

// ---- context ------------------------------------------------------------------------------
int hx_init(int device, void* stream, hx_ctx** out) {
  HX_REQUIRE(out, HX_EINVAL, "hx_init: null out");
  int n = 0;
  HX_CK(cudaGetDeviceCount(&n));
  HX_REQUIRE(device >= 0 && device < n, HX_EINVAL, "hx_init: no such CUDA device");
  HX_CK(cudaSetDevice(device));
  int major = 0;
  HX_CK(cudaDeviceGetAttribute(&major, cudaDevAttrComputeCapabilityMajor, device));
  HX_REQUIRE(major >= 10, HX_EUNSUPPORTED, "hx_init: libhx is built for sm_100a (B200)");
  hx_ctx* ctx = new hx_ctx();
  ctx->device = device;
  if (stream) {
    ctx->stream = static_cast<cudaStream_t>(stream);
  } else {
    cudaError_t e = cudaStreamCreateWithFlags(&ctx->stream, cudaStreamNonBlocking);
    if (e != cudaSuccess) {
      delete ctx;
      return cuda_fail(e, "cudaStreamCreate", __FILE__, __LINE__);
    }
    ctx->own_stream = true;
  }
  cudaDeviceGetAttribute(&ctx->n_sms, cudaDevAttrMultiProcessorCount, device);
  // keep freed stream-ordered allocations in the pool (no re-mapping per query)
  cudaMemPool_t pool;
  if (cudaDeviceGetDefaultMemPool(&pool, device) == cudaSuccess) {
    uint64_t thr = UINT64_MAX;
    cudaMemPoolSetAttribute(pool, cudaMemPoolAttrReleaseThreshold, &thr);
  }
  ctx->k1_ctas_per_sm = std::max(1, k1_occupancy(ctx));
  // (the persisting L2 set-aside is reserved only when HX_OPT_L2_PERSIST is enabled: reserving
  // it, even with no access-policy window in use, measured 2-5% slower K1 and a 2x slower K3;
  // HX_L2_PERSIST=1 enables it at init, for A/B measurements)
  if (const char* e = std::getenv("HX_L2_PERSIST")) {
    if (std::atoi(e) != 0 && hx_ctx_set_option(ctx, HX_OPT_L2_PERSIST, 1) != HX_OK) {
      ctx->l2_persist = 0;  // (an A/B switch: without it the context still works, unpinned)
      cudaGetLastError();
    }
  }
  {
    int least = 0, greatest = 0;
    if (cudaDeviceGetStreamPriorityRange(&least, &greatest) == cudaSuccess &&
        std::getenv("HX_NO_K1_PRIORITY") == nullptr)
      ctx->k1_priority = greatest;
    cudaGetLastError();
  }
  for (int a = 0; a < hx_ctx::kAux; ++a) {
    HX_CK(cudaStreamCreateWithFlags(&ctx->aux[a], cudaStreamNonBlocking));
    HX_CK(cudaEventCreateWithFlags(&ctx->join_ev[a], cudaEventDisableTiming));
  }
  HX_CK(cudaEventCreateWithFlags(&ctx->fork_ev, cudaEventDisableTiming));
  HX_CK(cudaStreamCreateWithFlags(&ctx->copy_stream, cudaStreamNonBlocking));
  HX_CK(cudaStreamCreateWithFlags(&ctx->fin_stream, cudaStreamNonBlocking));
  HX_CK(cudaEventCreateWithFlags(&ctx->fin_join_ev, cudaEventDisableTiming));
  *out = ctx;
  return HX_OK;
}

int hx_finalize(hx_ctx* ctx) {
  HX_REQUIRE(ctx, HX_EINVAL, "hx_finalize: null ctx");
  cudaSetDevice(ctx->device);
  cudaStreamSynchronize(ctx->stream);
  for (auto& pr : ctx->prof_events) {
    cudaEventDestroy(pr.first);
    cudaEventDestroy(pr.second);
  }
  for (auto e : ctx->event_pool) cudaEventDestroy(e);
  for (int a = 0; a < hx_ctx::kAux; ++a) {
    if (ctx->aux[a]) {
      cudaStreamSynchronize(ctx->aux[a]);
      cudaStreamDestroy(ctx->aux[a]);
    }
    if (ctx->join_ev[a]) cudaEventDestroy(ctx->join_ev[a]);
  }
  if (ctx->fork_ev) cudaEventDestroy(ctx->fork_ev);
  if (ctx->copy_stream) {
    cudaStreamSynchronize(ctx->copy_stream);
    cudaStreamDestroy(ctx->copy_stream);
  }
  if (ctx->fin_stream) {
    cudaStreamSynchronize(ctx->fin_stream);
    cudaStreamDestroy(ctx->fin_stream);
  }
  if (ctx->fin_join_ev) cudaEventDestroy(ctx->fin_join_ev);
  if (ctx->comm) ncclCommDestroy(ctx->comm);
  if (ctx->own_stream) cudaStreamDestroy(ctx->stream);
  delete ctx;
  return HX_OK;
}

int hx_ctx_stream(hx_ctx* ctx, void** stream) {
  HX_REQUIRE(ctx && stream, HX_EINVAL, "hx_ctx_stream: null argument");
  *stream = ctx->stream;
  return HX_OK;
}

int hx_ctx_info(hx_ctx* ctx, int* n_sms, int* k1_ctas_per_sm) {
  HX_REQUIRE(ctx, HX_EINVAL, "hx_ctx_info: null ctx");
  if (n_sms) *n_sms = ctx->n_sms;
  if (k1_ctas_per_sm) *k1_ctas_per_sm = ctx->k1_ctas_per_sm;
  return HX_OK;
}

// ---- communicator -------------------------------------------------------------------------
int hx_comm_unique_id(void* id128) {
  HX_REQUIRE(id128, HX_EINVAL, "hx_comm_unique_id: null buffer");
  static_assert(sizeof(ncclUniqueId) == 128, "ncclUniqueId is 128 bytes");
  ncclUniqueId id;
  HX_NCCL(ncclGetUniqueId(&id));
  std::memcpy(id128, &id, sizeof(id));
  return HX_OK;
}

int hx_comm_init(hx_ctx* ctx, int nranks, int rank, const void* id128) {
  HX_REQUIRE(ctx && id128 && nranks >= 1 && rank >= 0 && rank < nranks, HX_EINVAL,
             "hx_comm_init: bad argument");
  HX_REQUIRE(!ctx->comm, HX_EINVAL, "hx_comm_init: communicator already initialised");
  ncclUniqueId id;
  std::memcpy(&id, id128, sizeof(id));
  HX_CK(cudaSetDevice(ctx->device));
  HX_NCCL(ncclCommInitRank(&ctx->comm, nranks, id, rank));
  ctx->force_coll = std::getenv("HX_FORCE_COLLECTIVES") != nullptr;
  ctx->rank = rank;
  ctx->nranks = nranks;
  return HX_OK;
}

int hx_comm_info(hx_ctx* ctx, int* rank, int* nranks) {
  HX_REQUIRE(ctx, HX_EINVAL, "hx_comm_info: null ctx");
  if (rank) *rank = ctx->rank;
  if (nranks) *nranks = ctx->nranks;
  return HX_OK;
}

// ---- router ------------------------------------------------------------------------------
int hx_router_partition(int64_t n_rows, int n_parts, int64_t block_rows, int policy,
                        hx_partition** out) {
  HX_REQUIRE(out && n_rows >= 0 && n_parts >= 1 && block_rows >= 1 &&
                 (policy == HX_POLICY_RANGE || policy == HX_POLICY_ROUND_ROBIN),
             HX_EINVAL, "hx_router_partition: bad argument");
  hx_partition* p = new hx_partition();
  p->n_rows = n_rows;
  p->n_parts = n_parts;
  p->block_rows = block_rows;
  p->policy = policy;
  const int64_t nb = (n_rows + block_rows - 1) / block_rows;
  p->blocks.resize(nb);
  for (int64_t b = 0; b < nb; ++b) {
    hx_block& h = p->blocks[b];
    h.row_begin = b * block_rows;
    h.row_end = std::min(n_rows, (b + 1) * block_rows);
    h.part = (int32_t)(b % n_parts);  // round-robin; RANGE is assigned below
    h.reserved = 0;
  }
  if (policy == HX_POLICY_RANGE) {
    // part i owns blocks [floor(i*nb/P), floor((i+1)*nb/P)): contiguous, balanced to one block
    for (int i = 0; i < n_parts; ++i) {
      const int64_t b0 = (int64_t)i * nb / n_parts, b1 = (int64_t)(i + 1) * nb / n_parts;
      for (int64_t b = b0; b < b1; ++b) p->blocks[b].part = i;
    }
  }
  *out = p;
  return HX_OK;
}

int hx_partition_info(const hx_partition* p, int64_t* n_blocks, const hx_block** blocks) {
  HX_REQUIRE(p, HX_EINVAL, "hx_partition_info: null partition");
  if (n_blocks) *n_blocks = (int64_t)p->blocks.size();
  if (blocks) *blocks = p->blocks.data();
  return HX_OK;
}

int hx_partition_rows(const hx_partition* p, int part, int64_t* n_rows) {
  HX_REQUIRE(p && n_rows && part >= 0 && part < p->n_parts, HX_EINVAL,
             "hx_partition_rows: bad argument");
  int64_t n = 0;
  for (const hx_block& b : p->blocks)
    if (b.part == part) n += b.row_end - b.row_begin;
  *n_rows = n;
  return HX_OK;
}

int hx_partition_free(hx_partition* p) {
  delete p;
  return HX_OK;
}

// ---- columns (mem-move into HBM) ----------------------------------------------------------
int hx_load_columns(hx_ctx* ctx, const hx_col* cols, int n_cols, const hx_partition* part,
                    int part_index, int placement, hx_table** out) {
  HX_REQUIRE(ctx && out && n_cols >= 1 && cols, HX_EINVAL, "hx_load_columns: bad argument");
  HX_REQUIRE(n_cols <= HX_MAX_COLS, HX_ECAPACITY, "hx_load_columns: too many columns");
  HX_REQUIRE(placement >= HX_PLACE_COPY && placement <= HX_PLACE_HOST_MAPPED, HX_EINVAL,
             "hx_load_columns: bad placement");
  const int64_t n_src = cols[0].n_rows;
  for (int c = 0; c < n_cols; ++c) {
    HX_REQUIRE(cols[c].n_rows == n_src && (cols[c].data || n_src == 0), HX_EINVAL,
               "hx_load_columns: columns differ in length or are null");
    for (int d = 0; d < c; ++d)
      HX_REQUIRE(cols[d].col_id != cols[c].col_id, HX_EINVAL, "hx_load_columns: repeated col_id");
  }
  // rows of this part, as ranges of the source
  std::vector<std::pair<int64_t, int64_t>> ranges;
  if (part) {
    HX_REQUIRE(part->n_rows == n_src && part_index >= 0 && part_index < part->n_parts, HX_EINVAL,
               "hx_load_columns: partition does not match the columns");
    for (const hx_block& b : part->blocks) {
      if (b.part != part_index) continue;
      if (!ranges.empty() && ranges.back().second == b.row_begin)
        ranges.back().second = b.row_end;
      else
        ranges.push_back({b.row_begin, b.row_end});
    }
  } else if (n_src > 0) {
    ranges.push_back({0, n_src});
  }
  int64_t n = 0;
  for (auto& r : ranges) n += r.second - r.first;
  HX_CK(cudaSetDevice(ctx->device));
  hx_table* t = new hx_table();
  t->ctx = ctx;
  t->n_cols = n_cols;
  t->n_rows = n;
  t->placement = placement;
  for (int c = 0; c < n_cols; ++c) t->col_id[c] = cols[c].col_id;
  if (placement == HX_PLACE_COPY) {
    t->owned = true;
    for (int c = 0; c < n_cols; ++c) {
      t->dev[c] = nullptr;
      cudaPointerAttributes pa{};
      bool src_host = true;
      if (n > 0 && cudaPointerGetAttributes(&pa, cols[c].data) == cudaSuccess)
        src_host = pa.type != cudaMemoryTypeDevice && pa.type != cudaMemoryTypeManaged;
      cudaGetLastError();
      if (n == 0) continue;
      cudaError_t e = cudaMallocAsync(&t->dev[c], ((size_t)n * 4 + 255) & ~size_t(255), ctx->stream);
      if (e != cudaSuccess) {
        for (int d = 0; d < c; ++d) cudaFreeAsync(t->dev[d], ctx->stream);
        delete t;
        return cuda_fail(e, "cudaMallocAsync(column)", __FILE__, __LINE__);
      }
      int64_t off = 0;
      for (auto& r : ranges) {
        HX_CK(cudaMemcpyAsync(t->dev[c] + off, cols[c].data + r.first,
                              (size_t)(r.second - r.first) * 4, cudaMemcpyDefault, ctx->stream));
        if (src_host) ctx->h2d_bytes += (r.second - r.first) * 4;
        off += r.second - r.first;
      }
    }
  } else {
    if (ranges.size() > 1) {
      delete t;
      return fail(HX_EINVAL, "hx_load_columns: a view needs one contiguous row range");
    }
    const int64_t first = ranges.empty() ? 0 : ranges[0].first;
    for (int c = 0; c < n_cols; ++c) {
      cudaPointerAttributes a{};
      const int32_t* base = cols[c].data;
      if (n_src > 0 && cudaPointerGetAttributes(&a, cols[c].data) == cudaSuccess) {
        const bool ok = placement == HX_PLACE_VIEW ? a.type == cudaMemoryTypeDevice ||
                                                         a.type == cudaMemoryTypeManaged
                        : placement == HX_PLACE_HOST_MAPPED
                            ? a.type == cudaMemoryTypeHost && a.devicePointer != nullptr
                            : a.type == cudaMemoryTypeHost;
        if (!ok) {
          delete t;
          return fail(HX_EINVAL, placement == HX_PLACE_VIEW
                                     ? "hx_load_columns: HX_PLACE_VIEW needs device memory"
                                 : placement == HX_PLACE_HOST_MAPPED
                                     ? "hx_load_columns: HX_PLACE_HOST_MAPPED needs mapped pinned memory"
                                     : "hx_load_columns: HX_PLACE_HOST_PINNED needs pinned memory");
        }
        // zero-copy: the device's address of the mapped pages (equal to the host address
        // under UVA)
        if (placement == HX_PLACE_HOST_MAPPED) base = static_cast<const int32_t*>(a.devicePointer);
      } else {
        cudaGetLastError();
        if (placement == HX_PLACE_HOST_MAPPED && n_src > 0) {
          delete t;
          return fail(HX_EINVAL, "hx_load_columns: HX_PLACE_HOST_MAPPED needs mapped pinned memory");
        }
      }
      t->dev[c] = const_cast<int32_t*>(base) + first;
    }
  }
  *out = t;
  return HX_OK;
}

int hx_table_info(const hx_table* t, int64_t* n_rows, int* n_cols) {
  HX_REQUIRE(t, HX_EINVAL, "hx_table_info: null table");
  if (n_rows) *n_rows = t->n_rows;
  if (n_cols) *n_cols = t->n_cols;
  return HX_OK;
}

int hx_table_slice(const hx_table* t, int64_t row_begin, int64_t row_end, hx_table** out) {
  HX_REQUIRE(t && out && row_begin >= 0 && row_end >= row_begin && row_end <= t->n_rows,
             HX_EINVAL, "hx_table_slice: bad range");
  hx_table* s = new hx_table(*t);
  s->owned = false;
  s->parent = t;
  s->n_rows = row_end - row_begin;
  for (int c = 0; c < t->n_cols; ++c) s->dev[c] = t->dev[c] ? t->dev[c] + row_begin : nullptr;
  *out = s;
  return HX_OK;
}

int hx_table_read(const hx_table* t, int32_t col_id, int64_t row_begin, int64_t n, int32_t* dst) {
  HX_REQUIRE(t && (dst || n == 0) && row_begin >= 0 && n >= 0 && row_begin + n <= t->n_rows,
             HX_EINVAL, "hx_table_read: bad argument");
  HX_REQUIRE(table_has_col(t, col_id), HX_EINVAL, "hx_table_read: column not in table");
  if (n == 0) return HX_OK;
  HX_CK(cudaSetDevice(t->ctx->device));
  HX_CK(cudaMemcpyAsync(dst, table_col(t, col_id) + row_begin, (size_t)n * 4, cudaMemcpyDefault,
                        t->ctx->stream));
  HX_CK(cudaStreamSynchronize(t->ctx->stream));
  t->ctx->d2h_bytes += n * 4;
  return HX_OK;
}

int hx_table_write(hx_table* t, int32_t col_id, int64_t row_begin, int64_t n, const int32_t* src) {
  HX_REQUIRE(t && (src || n == 0) && row_begin >= 0 && n >= 0 && row_begin + n <= t->n_rows,
             HX_EINVAL, "hx_table_write: bad argument");
  HX_REQUIRE(t->placement == HX_PLACE_COPY || t->placement == HX_PLACE_VIEW, HX_EUNSUPPORTED,
             "hx_table_write: the table must be device resident");
  HX_REQUIRE(table_has_col(t, col_id), HX_EINVAL, "hx_table_write: column not in table");
  if (n == 0) return HX_OK;
  HX_CK(cudaSetDevice(t->ctx->device));
  cudaPointerAttributes pa{};
  bool src_host = true;
  if (cudaPointerGetAttributes(&pa, src) == cudaSuccess)
    src_host = pa.type != cudaMemoryTypeDevice && pa.type != cudaMemoryTypeManaged;
  cudaGetLastError();
  HX_CK(cudaMemcpyAsync(const_cast<int32_t*>(table_col(t, col_id)) + row_begin, src, (size_t)n * 4,
                        cudaMemcpyDefault, t->ctx->stream));
  if (src_host) t->ctx->h2d_bytes += n * 4;
  return HX_OK;
}

int hx_table_free(hx_table* t) {
  HX_REQUIRE(t, HX_EINVAL, "hx_table_free: null table");
  if (t->owned) {
    cudaSetDevice(t->ctx->device);
    for (int c = 0; c < t->n_cols; ++c)
      if (t->dev[c]) cudaFreeAsync(t->dev[c], t->ctx->stream);
  }
  delete t;
  return HX_OK;
}

// ---- hash tables ---------------------------------------------------------------------------
int hx_build_dim_ht(hx_ctx* ctx, const hx_table* dim, int32_t key_col, const hx_pred* preds,
                    int n_preds, int32_t group_col, int32_t group_lo, int32_t group_hi,
                    hx_ht** out) {
  if (ctx) HX_CK(cudaSetDevice(ctx->device));
  return build_dim_ht(ctx, dim, key_col, preds, n_preds, group_col, group_lo, group_hi, out);
}

int hx_build_dim_ht_ex(hx_ctx* ctx, const hx_table* dim, int32_t key_col, const hx_pred* preds,
                       int n_preds, int32_t group_col, int32_t group_lo, int32_t group_hi,
                       int flags, hx_ht** out) {
  if (ctx) HX_CK(cudaSetDevice(ctx->device));
  return build_dim_ht(ctx, dim, key_col, preds, n_preds, group_col, group_lo, group_hi, out,
                      flags);
}

int hx_ht_info(hx_ht* ht, int64_t* n_keys, int64_t* n_slots, int32_t* n_ranks,
               int32_t* rank_to_code) {
  HX_REQUIRE(ht, HX_EINVAL, "hx_ht_info: null table");
  HX_CK(cudaSetDevice(ht->ctx->device));
  HtHeader h{};
  HX_CK(cudaMemcpyAsync(&h, ht->hdr, sizeof(h), cudaMemcpyDeviceToHost, ht->ctx->stream));
  HX_CK(cudaStreamSynchronize(ht->ctx->stream));
  if (n_keys) *n_keys = h.n_keys;
  if (n_slots) *n_slots = int64_t(1) << h.log2cap;
  if (n_ranks) *n_ranks = h.n_ranks;
  if (rank_to_code && ht->has_group && h.n_ranks > 0) {
    HX_CK(cudaMemcpy(rank_to_code, ht->rank_to_code, sizeof(int32_t) * h.n_ranks,
                     cudaMemcpyDeviceToHost));
  } else if (rank_to_code && !ht->has_group) {
    rank_to_code[0] = 0;
  }
  if (h.error == HX_EDUPKEY) return fail(HX_EDUPKEY, "hx_build_dim_ht: duplicate primary key");
  if (h.error) return fail(h.error, "hx_build_dim_ht: group code outside [group_lo, group_hi]");
  return HX_OK;
}

int hx_ctx_set_option(hx_ctx* ctx, int option, int value) {
  HX_REQUIRE(ctx, HX_EINVAL, "hx_ctx_set_option: null ctx");
  if (option == HX_OPT_JOIN_LAYOUT) {
    HX_REQUIRE(value == HX_JOIN_AUTO || value == HX_JOIN_HASH, HX_EINVAL,
               "hx_ctx_set_option: bad join layout");
    ctx->join_layout = value;
  } else if (option == HX_OPT_L2_PERSIST) {
    // L2 set-aside for persisting accesses (the probe structures' access-policy windows): the
    // device maximum while enabled (HX_L2_PERSIST_MB lowers it), released when disabled
    HX_CK(cudaSetDevice(ctx->device));
    int pmax = 0, wmax = 0;
    cudaDeviceGetAttribute(&pmax, cudaDevAttrMaxPersistingL2CacheSize, ctx->device);
    cudaDeviceGetAttribute(&wmax, cudaDevAttrMaxAccessPolicyWindowSize, ctx->device);
    int64_t want = value ? pmax : 0;
    if (const char* e = std::getenv("HX_L2_PERSIST_MB")) want = std::min<int64_t>(want, std::atoll(e) << 20);
    HX_CK(cudaDeviceSetLimit(cudaLimitPersistingL2CacheSize, (size_t)want));
    size_t got = 0;
    cudaDeviceGetLimit(&got, cudaLimitPersistingL2CacheSize);
    ctx->l2_persist = value != 0 && got > 0 && wmax > 0;
    ctx->l2_persist_max = ctx->l2_persist ? (int64_t)got : 0;
    ctx->l2_window_max = wmax;
    if (!value) cudaCtxResetPersistingL2Cache();
  } else {
    return fail(HX_EINVAL, "hx_ctx_set_option: unknown option");
  }
  return HX_OK;
}

int hx_comm_trace(hx_ctx* ctx, hx_coll_rec* out, int cap, int* n, int reset) {
  HX_REQUIRE(ctx && n && cap >= 0 && (cap == 0 || out), HX_EINVAL, "hx_comm_trace: bad argument");
  *n = (int)ctx->coll_trace.size();
  for (int i = 0; i < std::min(cap, *n); ++i) out[i] = ctx->coll_trace[i];
  if (reset) ctx->coll_trace.clear();
  return HX_OK;
}

int hx_ht_broadcast(hx_ctx* ctx, hx_ht* ht, int root) {
  HX_REQUIRE(ctx && ht, HX_EINVAL, "hx_ht_broadcast: null argument");
  HX_REQUIRE(ctx->comm, HX_ENCCL, "hx_ht_broadcast: no communicator (hx_comm_init)");
  HX_REQUIRE(root >= 0 && root < ctx->nranks, HX_EINVAL, "hx_ht_broadcast: bad root");
  HX_CK(cudaSetDevice(ctx->device));
  // 1) header + rank maps (same layout on every rank: same dimension and group range)
  const size_t maps = (sizeof(HtHeader) + 2 * (size_t)ht->domain * sizeof(int32_t) + 255) & ~size_t(255);
  coll_log(ctx, HX_COLL_BROADCAST, ht->base, (int64_t)maps, 1, root);
  HX_NCCL(ncclBroadcast(ht->base, ht->base, maps, ncclUint8, root, ctx->comm, ctx->stream));
  // 2) the slots in use: every rank learns the capacity from the broadcast header
  HtHeader h{};
  HX_CK(cudaMemcpyAsync(&h, ht->hdr, sizeof(h), cudaMemcpyDeviceToHost, ctx->stream));
  HX_CK(cudaStreamSynchronize(ctx->stream));
  HX_REQUIRE(h.log2cap <= ht->max_log2cap, HX_EINVAL,
             "hx_ht_broadcast: tables differ in size across ranks");
  coll_log(ctx, HX_COLL_BROADCAST, ht->slots, (int64_t(1) << h.log2cap) * 8, 1, root);
  HX_NCCL(ncclBroadcast(ht->slots, ht->slots, (size_t(1) << h.log2cap) * 8, ncclUint8, root,
                        ctx->comm, ctx->stream));
  HX_REQUIRE(h.bloom_log2w <= ht->max_bloom_log2w, HX_EINVAL,
             "hx_ht_broadcast: tables differ in size across ranks");
  coll_log(ctx, HX_COLL_BROADCAST, ht->bloom, (int64_t(1) << h.bloom_log2w) * 4, 1, root);
  HX_NCCL(ncclBroadcast(ht->bloom, ht->bloom, (size_t(1) << h.bloom_log2w) * 4, ncclUint8, root,
                        ctx->comm, ctx->stream));
  return HX_OK;
}

int hx_ht_free(hx_ht* ht) {
  HX_REQUIRE(ht, HX_EINVAL, "hx_ht_free: null table");
  cudaSetDevice(ht->ctx->device);
  ht_destroy(ht);
  return HX_OK;
}

// ---- fused pipeline --------------------------------------------------------------------------
int hx_pipeline_probe_agg(hx_ctx* ctx, const hx_table* fact, const hx_query_shape* shape,
                          hx_ht* const* hts, int n_hts, hx_agg** out) {
  HX_REQUIRE(ctx && out, HX_EINVAL, "hx_pipeline_probe_agg: null argument");
  HX_CK(cudaSetDevice(ctx->device));
  hx_agg* agg = new hx_agg();
  agg->ctx = ctx;
  int rc = probe_agg(ctx, fact, shape, hts, n_hts, agg, true);
  if (rc != HX_OK) {
    if (agg->base) cudaFreeAsync(agg->base, ctx->stream);
    delete agg;
    return rc;
  }
  *out = agg;
  return HX_OK;
}

int hx_pipeline_probe_agg_into(hx_ctx* ctx, const hx_table* fact, const hx_query_shape* shape,
                               hx_ht* const* hts, int n_hts, hx_agg* agg) {
  HX_REQUIRE(ctx && agg && agg->base, HX_EINVAL, "hx_pipeline_probe_agg_into: null argument");
  HX_CK(cudaSetDevice(ctx->device));
  return probe_agg(ctx, fact, shape, hts, n_hts, agg, false);
}

int hx_pipeline_probe_agg_routed(hx_ctx* ctx, const hx_table* fact, const hx_query_shape* shape,
                                 hx_ht* const* hts, int n_hts, hx_shared_router* router,
                                 int64_t block_rows, hx_agg** out, int64_t* n_blocks) {
  HX_REQUIRE(ctx && out, HX_EINVAL, "hx_pipeline_probe_agg_routed: null argument");
  HX_CK(cudaSetDevice(ctx->device));
  hx_agg* agg = new hx_agg();
  agg->ctx = ctx;
  int rc = probe_agg_routed(ctx, fact, shape, hts, n_hts, agg, router, block_rows, n_blocks);
  if (rc != HX_OK) {
    if (agg->base) cudaFreeAsync(agg->base, ctx->stream);
    delete agg;
    return rc;
  }
  *out = agg;
  return HX_OK;
}

// ---- union-router merge + finalize ------------------------------------------------------------
int hx_merge_aggregates(hx_ctx* ctx, hx_agg* agg, int root, int64_t* sums, int64_t* counts,
                        int32_t* keys, int64_t cap, int64_t* n_rows) {
  HX_REQUIRE(ctx && agg && n_rows && cap >= 0 && (cap == 0 || (sums && counts)), HX_EINVAL,
             "hx_merge_aggregates: bad argument");
  HX_REQUIRE(!(agg->n_gdims > 0 && cap > 0 && !keys), HX_EINVAL,
             "hx_merge_aggregates: keys buffer required for grouped queries");
  HX_CK(cudaSetDevice(ctx->device));
  *n_rows = 0;
  AggMeta m{};
  HX_CK(cudaMemcpyAsync(&m, agg->meta, sizeof(m), cudaMemcpyDeviceToHost, ctx->stream));
  HX_CK(cudaStreamSynchronize(ctx->stream));
  // builds this pipeline depended on
  int err = 0;
  const char* msg = nullptr;
  for (const hx_ht* ht : agg->deps) {
    HtHeader h{};
    HX_CK(cudaMemcpy(&h, ht->hdr, sizeof(h), cudaMemcpyDeviceToHost));
    if (!err && h.error == HX_EDUPKEY) err = HX_EDUPKEY, msg = "dimension build: duplicate primary key";
    if (!err && h.error) err = HX_EINVAL, msg = "dimension build: group code outside its range";
  }
  if (!err && m.error) err = m.error, msg = "hx_pipeline_probe_agg: group capacity exceeded";
  if (!err && root >= ctx->nranks) err = HX_EINVAL, msg = "hx_merge_aggregates: bad root";
  const int64_t ng = m.n_groups;
  if (use_collectives(ctx)) {
    // every rank reaches this collective, also one that failed locally: agree on {any error,
    // max n_groups} first, so that an error is reported on every rank instead of leaving the
    // others blocked in the data collective below
    int64_t st[2] = {err ? 1 : 0, ng};
    int64_t* dst = nullptr;
    HX_CK(cudaMallocAsync(reinterpret_cast<void**>(&dst), sizeof(st), ctx->stream));
    HX_CK(cudaMemcpyAsync(dst, st, sizeof(st), cudaMemcpyHostToDevice, ctx->stream));
    coll_log(ctx, HX_COLL_ALLREDUCE, dst, 2, 8);
    const ncclResult_t nr = ncclAllReduce(dst, dst, 2, ncclInt64, ncclMax, ctx->comm, ctx->stream);
    cudaMemcpyAsync(st, dst, sizeof(st), cudaMemcpyDeviceToHost, ctx->stream);
    cudaFreeAsync(dst, ctx->stream);
    HX_CK(cudaStreamSynchronize(ctx->stream));
    if (nr != ncclSuccess) return fail(HX_ENCCL, ncclGetErrorString(nr));
    if (err) return fail(err, msg);
    if (st[0]) return fail(HX_EINVAL, "hx_merge_aggregates: the merge failed on another rank");
    if (st[1] != ng) return fail(HX_EINVAL, "hx_merge_aggregates: ranks disagree on n_groups");
  } else if (err) {
    return fail(err, msg);
  }
  if (use_collectives(ctx) && ng > 0) {
    // sums and cnts are adjacent regions of cap_groups each: reduce both with one call each
    if (root < 0) {
      coll_log(ctx, HX_COLL_ALLREDUCE, agg->sums, ng, 8);
      HX_NCCL(ncclAllReduce(agg->sums, agg->sums, ng, ncclUint64, ncclSum, ctx->comm, ctx->stream));
      coll_log(ctx, HX_COLL_ALLREDUCE, agg->cnts, ng, 8);
      HX_NCCL(ncclAllReduce(agg->cnts, agg->cnts, ng, ncclUint64, ncclSum, ctx->comm, ctx->stream));
    } else {
      coll_log(ctx, HX_COLL_REDUCE, agg->sums, ng, 8, root);
      HX_NCCL(ncclReduce(agg->sums, agg->sums, ng, ncclUint64, ncclSum, root, ctx->comm, ctx->stream));
      coll_log(ctx, HX_COLL_REDUCE, agg->cnts, ng, 8, root);
      HX_NCCL(ncclReduce(agg->cnts, agg->cnts, ng, ncclUint64, ncclSum, root, ctx->comm, ctx->stream));
      if (ctx->rank != root) {
        HX_CK(cudaStreamSynchronize(ctx->stream));
        return HX_OK;
      }
    }
  }
  std::vector<int64_t> hs(ng), hc(ng);
  if (ng) {
    HX_CK(cudaMemcpyAsync(hs.data(), agg->sums, ng * 8, cudaMemcpyDeviceToHost, ctx->stream));
    HX_CK(cudaMemcpyAsync(hc.data(), agg->cnts, ng * 8, cudaMemcpyDeviceToHost, ctx->stream));
  }
  std::vector<int32_t> r2c[HX_MAX_GDIMS];
  for (int g = 0; g < agg->n_gdims; ++g) {
    const hx_ht* ht = agg->gdim_ht[g];
    r2c[g].assign(std::max(1, m.n_ranks[g]), 0);
    if (ht->has_group && m.n_ranks[g] > 0)
      HX_CK(cudaMemcpyAsync(r2c[g].data(), ht->rank_to_code, sizeof(int32_t) * m.n_ranks[g],
                            cudaMemcpyDeviceToHost, ctx->stream));
  }
  HX_CK(cudaStreamSynchronize(ctx->stream));
  ctx->d2h_bytes += (int64_t)sizeof(m) + 16 * ng;
  for (int g = 0; g < agg->n_gdims; ++g) ctx->d2h_bytes += 4 * (int64_t)r2c[g].size();
  // finalize (a7): drop empty groups (an ungrouped query keeps its one row), decode codes
  int32_t nrk[HX_MAX_GDIMS];
  const int32_t* maps[HX_MAX_GDIMS];
  for (int g = 0; g < agg->n_gdims; ++g) {
    nrk[g] = std::max(1, m.n_ranks[g]);
    maps[g] = r2c[g].data();
  }
  int64_t rows = 0;
  if (agg->n_gdims == 0 && ng == 0) {  // unreachable (n_groups >= 1), kept for safety
    if (cap > 0) sums[0] = counts[0] = 0;
    rows = 1;
  } else {
    const int rc = hx_group_decode(agg->n_gdims, nrk, maps, hs.data(), hc.data(), ng, keys, sums,
                                   counts, cap, &rows);
    if (rc != HX_OK && rc != HX_ECAPACITY) return rc;
  }
  *n_rows = rows;
  if (rows > cap) return fail(HX_ECAPACITY, "hx_merge_aggregates: output buffer too small");
  return HX_OK;
}

int hx_group_layout(int n_gdims, const int32_t* n_ranks, int64_t* strides, int64_t* n_groups) {
  HX_REQUIRE(n_gdims >= 0 && n_gdims <= HX_MAX_GDIMS && n_groups && (n_gdims == 0 || (n_ranks && strides)),
             HX_EINVAL, "hx_group_layout: bad argument");
  int64_t stride = 1;
  for (int g = n_gdims - 1; g >= 0; --g) {
    HX_REQUIRE(n_ranks[g] >= 1, HX_EINVAL, "hx_group_layout: a dimension needs >= 1 rank");
    strides[g] = stride;
    stride *= n_ranks[g];
    HX_REQUIRE(stride <= HX_MAX_GROUPS, HX_ECAPACITY, "hx_group_layout: too many groups");
  }
  *n_groups = stride;
  return HX_OK;
}

int hx_group_decode(int n_gdims, const int32_t* n_ranks, const int32_t* const* rank_to_code,
                    const int64_t* sums, const int64_t* counts, int64_t n_groups, int32_t* keys,
                    int64_t* out_sums, int64_t* out_counts, int64_t cap, int64_t* n_rows) {
  HX_REQUIRE(n_rows && n_groups >= 0 && (n_groups == 0 || (sums && counts)) && cap >= 0 &&
                 (cap == 0 || (out_sums && out_counts && (n_gdims == 0 || keys))),
             HX_EINVAL, "hx_group_decode: bad argument");
  int64_t strides[HX_MAX_GDIMS], ng = 0;
  const int rc = hx_group_layout(n_gdims, n_ranks, strides, &ng);
  if (rc != HX_OK) return rc;
  HX_REQUIRE(ng == n_groups, HX_EINVAL, "hx_group_decode: n_groups differs from the layout");
  for (int g = 0; g < n_gdims; ++g)
    HX_REQUIRE(rank_to_code && rank_to_code[g], HX_EINVAL, "hx_group_decode: missing rank map");
  int64_t rows = 0;
  for (int64_t i = 0; i < n_groups; ++i) {
    if (n_gdims > 0 && counts[i] == 0) continue;
    if (rows < cap) {
      out_sums[rows] = sums[i];
      out_counts[rows] = counts[i];
      for (int g = 0; g < n_gdims; ++g)
        keys[rows * n_gdims + g] = rank_to_code[g][(i / strides[g]) % n_ranks[g]];
    }
    ++rows;
  }
  *n_rows = rows;
  if (rows > cap) return fail(HX_ECAPACITY, "hx_group_decode: output buffer too small");
  return HX_OK;
}

int hx_agg_free(hx_agg* agg) {
  HX_REQUIRE(agg, HX_EINVAL, "hx_agg_free: null agg");
  cudaSetDevice(agg->ctx->device);
  if (agg->base) cudaFreeAsync(agg->base, agg->ctx->stream);
  delete agg;
  return HX_OK;
}

// ---- measurement -----------------------------------------------------------------------------
int hx_profile_enable(hx_ctx* ctx, int on) {
  HX_REQUIRE(ctx, HX_EINVAL, "hx_profile_enable: null ctx");
  ctx->prof_on = on != 0;
  return HX_OK;
}

int hx_profile_read(hx_ctx* ctx, double* k1_ms, int64_t* k1_launches, int64_t* k1_bytes,
                    int reset) {
  HX_REQUIRE(ctx, HX_EINVAL, "hx_profile_read: null ctx");
  HX_CK(cudaSetDevice(ctx->device));
  HX_CK(cudaStreamSynchronize(ctx->stream));
  for (auto& pr : ctx->prof_events) {
    float ms = 0.f;
    HX_CK(cudaEventElapsedTime(&ms, pr.first, pr.second));
    ctx->prof_ms += ms;
    ctx->event_pool.push_back(pr.first);
    ctx->event_pool.push_back(pr.second);
  }
  ctx->prof_events.clear();
  if (k1_ms) *k1_ms = ctx->prof_ms;
  if (k1_launches) *k1_launches = ctx->prof_launches;
  if (k1_bytes) *k1_bytes = ctx->prof_bytes;
  if (reset) {
    ctx->prof_ms = 0;
    ctx->prof_launches = 0;
    ctx->prof_bytes = 0;
  }
  return HX_OK;
}

int hx_stats(hx_ctx* ctx, int64_t* launches, int64_t* h2d_bytes, int64_t* d2h_bytes, int reset) {
  HX_REQUIRE(ctx, HX_EINVAL, "hx_stats: null ctx");
  if (launches) *launches = ctx->launches;
  if (h2d_bytes) *h2d_bytes = ctx->h2d_bytes;
  if (d2h_bytes) *d2h_bytes = ctx->d2h_bytes;
  if (reset) ctx->launches = ctx->h2d_bytes = ctx->d2h_bytes = 0;
  return HX_OK;
}

}  // extern "C"

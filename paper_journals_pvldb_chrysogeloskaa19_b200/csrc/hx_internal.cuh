// hx_internal.cuh — shared definitions of libhx (the product path). Not part of the C-ABI.
#pragma once
#include <cuda_runtime.h>
#include <nccl.h>
#include <stdint.h>

#include <string>
#include <vector>

#include "hx.h"

namespace hx {

// ---- error plumbing (hx_last_error) ----------------------------------------------------
void set_error(const std::string& msg);
int fail(int code, const std::string& msg);
int cuda_fail(cudaError_t e, const char* what, const char* file, int line);

#define HX_CK(call)                                                   \
  do {                                                                \
    cudaError_t _e = (call);                                          \
    if (_e != cudaSuccess) return ::hx::cuda_fail(_e, #call, __FILE__, __LINE__); \
  } while (0)
#define HX_CK_LAUNCH(what) HX_CK(cudaGetLastError())
#define HX_REQUIRE(cond, code, msg) \
  do {                              \
    if (!(cond)) return ::hx::fail((code), (msg)); \
  } while (0)

// ---- hash table layout (one device allocation per table) ------------------------------
// [HtHeader | code_to_rank[domain] | rank_to_code[domain] | pad to 256 | slots[max_cap]]
constexpr uint64_t kEmptySlot = 0xFFFFFFFFFFFFFFFFull;
constexpr int kMinLog2Cap = 4;

struct HtHeader {
  int32_t log2cap;   // device-written by the rank kernel
  int32_t n_keys;    // passing dimension rows (atomic counter in the filter kernel)
  int32_t n_ranks;   // distinct group codes among passing rows (1 if no group column)
  int32_t error;     // 0 ok, HX_EDUPKEY, HX_EINVAL (group code out of range)
  int32_t max_log2cap;
  int32_t group_lo;
  int32_t domain;
  int32_t bloom_log2w;  // log2 of the Bloom filter's 32-bit words in use (device-written)
  // range of the passing keys, order-preserving encoded (key ^ 0x80000000): the filter kernel
  // keeps ~min and max with atomicMax so that a zeroed header is the neutral element
  uint32_t kmin_inv;
  uint32_t kmax_enc;
  uint32_t done;     // CTAs of the filter kernel finished (the last one ranks)
};
__host__ __device__ __forceinline__ uint32_t key_enc(int32_t k) { return (uint32_t)k ^ 0x80000000u; }
__host__ __device__ __forceinline__ int32_t key_dec(uint32_t e) { return (int32_t)(e ^ 0x80000000u); }

// Direct map of a dense-key dimension (R20): entry (key - kmin), 2^lw bits wide,
// holds rank + 1 of the passing row with that key (0: no passing row). With surrogate keys
// 1..N (SSB) this is the hash table with the identity hash: one load, no probe chain, exact.
__host__ __device__ __forceinline__ uint32_t dm_vmask(int lw) {
  return lw >= 5 ? 0xFFFFFFFFu : ((1u << (1u << lw)) - 1u);
}
__host__ __device__ __forceinline__ int64_t dm_words_for(int64_t span, int lw) {
  const int64_t w = ((((span << lw) + 31) >> 5) + 3) & ~int64_t(3);  // whole 16-byte units
  return w < 4 ? 4 : w;
}

// Blocked Bloom filter over the passing keys (one 32-bit word per key, two bits set), built
// with the table. K1 stages it in shared memory to drop most non-matching rows before any
// L2 probe (semi-join reduction). kBloomBitsPerKey bits per key: false positives ~1.5% (K1 folds it to 8..1).
constexpr int kBloomBitsPerKey = 16;
__host__ __device__ __forceinline__ int bloom_log2w_for(long long n_keys) {
  long long bits = n_keys * kBloomBitsPerKey;
  int l = 5;
  while ((1ll << l) < bits) ++l;
  return l - 5;
}
// One multiply: the word is the top log2w bits of h, the two bit positions are h[6..10] and
// h[11..15] (disjoint from the word bits while log2w <= 16, i.e. filters up to 256 KB).
__host__ __device__ __forceinline__ uint32_t bloom_hash(int32_t key) {
  return (uint32_t)key * 0x85EBCA6Bu;
}
__host__ __device__ __forceinline__ uint32_t bloom_word(int32_t key, int log2w) {
  return log2w == 0 ? 0u : bloom_hash(key) >> (32 - log2w);
}
__host__ __device__ __forceinline__ uint32_t bloom_mask(int32_t key) {
  const uint32_t h = bloom_hash(key);
  return (1u << ((h >> 6) & 31u)) | (1u << ((h >> 11) & 31u));
}

// Slots are grouped in 16-byte buckets of kBucketSlots = 2 (one 128-bit load per probe
// step). A key's home is the first slot of its bucket; linear probing proceeds slot by
// slot from there, so within a bucket slot 1 is filled only after slot 0 and "slot 1 of the
// bucket is empty" proves a miss. Load factor <= 1/kLoadInv.
constexpr int kBucketSlots = 2;
#ifndef HX_LOAD_INV
#define HX_LOAD_INV 4
#endif
constexpr int kLoadInv = HX_LOAD_INV;
constexpr long long kBigTableBytes = 8ll << 20;  // above: load factor <= 1/2 (hx_build.cu)
constexpr int32_t kEmptyKey = -1;  // keys must differ from -1 (checked by the build)

// Multiplicative (Fibonacci) hashing: the top log2(cap/2) bits of key * 2^32/phi.
__host__ __device__ __forceinline__ uint32_t ht_bucket(int32_t key, int log2cap) {
  return ((uint32_t)key * 2654435769u) >> (33 - log2cap);
}
__host__ __device__ __forceinline__ uint32_t ht_home(int32_t key, int log2cap) {
  return ht_bucket(key, log2cap) << 1;
}

// Device-side predicate (a copy of hx_pred with the column resolved to a pointer or a
// staged-column index).
struct DevPred {
  int32_t c;      // column index (table column or staged column)
  int32_t kind;
  int32_t lo, hi;
  int32_t n_in;
  int32_t in[4];
};

__device__ __forceinline__ bool pred_pass(const DevPred& p, int32_t v) {
  if (p.kind == HX_PRED_RANGE) return v >= p.lo && v <= p.hi;
  bool r = false;
#pragma unroll
  for (int i = 0; i < 4; ++i) r |= (i < p.n_in) && v == p.in[i];
  return r;
}

}  // namespace hx

// ---- library objects (opaque in hx.h) ----------------------------------------------------
struct hx_ctx {
  int device = 0;
  cudaStream_t stream = nullptr;
  bool own_stream = false;
  int n_sms = 0;
  int k1_ctas_per_sm = 0;
  int k1_priority = 0;  // launch priority of K1 (the device's greatest; builds keep the default)
  ncclComm_t comm = nullptr;
  int rank = 0, nranks = 1;
  // run the collectives even on a 1-rank communicator (HX_FORCE_COLLECTIVES=1 at
  // hx_comm_init): the multi-GPU call sequence, exercised on one GPU by the tests
  bool force_coll = false;
  // K1 profiling: event pairs around each launch
  bool prof_on = false;
  std::vector<std::pair<cudaEvent_t, cudaEvent_t>> prof_events;
  std::vector<cudaEvent_t> event_pool;
  int64_t prof_launches = 0, prof_bytes = 0;
  double prof_ms = 0.0;
  // hx_stats counters
  int64_t launches = 0, h2d_bytes = 0, d2h_bytes = 0;
  int64_t capture_launches = 0, capture_d2h = 0, capture_h2d = 0;  // at hx_graph_begin
  // fork/join of the independent dimension builds of a plan (parallel graph branches)
  static constexpr int kAux = 4;
  cudaStream_t aux[kAux] = {nullptr, nullptr, nullptr, nullptr};
  cudaEvent_t fork_ev = nullptr;
  cudaEvent_t join_ev[kAux] = {nullptr, nullptr, nullptr, nullptr};
  cudaStream_t copy_stream = nullptr;  // mem-move H2D copies of host-resident blocks
  // finalize + D2H of each plan run off the main stream so the next pipeline's K1 does not
  // wait for them; joined back into the main stream at the end of every enqueue call
  cudaStream_t fin_stream = nullptr;
  cudaEvent_t fin_join_ev = nullptr;
  // hx_ctx_set_option
  int join_layout = HX_JOIN_AUTO;
  int l2_persist = 0;           // measured: the persisting window costs ~2%
  int64_t l2_persist_max = 0;   // persisting L2 set-aside (bytes) set at hx_init
  int64_t l2_window_max = 0;    // cudaDevAttrMaxAccessPolicyWindowSize
  // hx_comm_trace: the NCCL data calls issued on this ctx (last kTraceCap kept)
  static constexpr size_t kTraceCap = 4096;
  std::vector<hx_coll_rec> coll_trace;
};
namespace hx {
// Record one NCCL data call (hx_comm_trace); call it right before issuing the collective.
inline void coll_log(hx_ctx* ctx, int op, const void* buf, int64_t count, int elem_bytes,
                     int root_or_peer = -1) {
  if (ctx->coll_trace.size() >= hx_ctx::kTraceCap)
    ctx->coll_trace.erase(ctx->coll_trace.begin(), ctx->coll_trace.begin() + hx_ctx::kTraceCap / 2);
  ctx->coll_trace.push_back(hx_coll_rec{op, root_or_peer, count, elem_bytes, 0,
                                        (uint64_t)reinterpret_cast<uintptr_t>(buf)});
}
}  // namespace hx

struct hx_partition {
  int64_t n_rows = 0, block_rows = 0;
  int n_parts = 0, policy = 0;
  std::vector<hx_block> blocks;
};

struct hx_table {
  hx_ctx* ctx = nullptr;
  int n_cols = 0;
  int32_t col_id[HX_MAX_COLS];
  int32_t* dev[HX_MAX_COLS];       // device (or pinned host) base of each column
  int64_t n_rows = 0;
  int placement = HX_PLACE_COPY;
  bool owned = false;              // columns allocated by the library
  const hx_table* parent = nullptr;
};

struct hx_ht {
  hx_ctx* ctx = nullptr;
  void* base = nullptr;            // the single device allocation
  size_t bytes = 0;
  hx::HtHeader* hdr = nullptr;
  int32_t* code_to_rank = nullptr;
  int32_t* rank_to_code = nullptr;
  unsigned long long* slots = nullptr;
  int32_t max_log2cap = 0;
  int32_t domain = 1;              // group code range size (1 when no group column)
  int32_t group_lo = 0;
  bool has_group = false;
  bool identity_ranks = false;     // HX_BUILD_IDENTITY_RANKS: n_ranks == domain
  int64_t dim_rows = 0;
  void* build = nullptr;           // hx::BuildParams (hx_build.cu): re-enqueueable build
  uint32_t* bloom = nullptr;       // Bloom filter words (after the slots)
  int32_t max_bloom_log2w = 0;
  int64_t known_keys = -1;         // passing keys, when a plan has observed them (else -1)
  // direct map (plans over dense keys; nullptr: hash-table build and probe)
  uint32_t* dm = nullptr;
  int64_t dm_words = 0;
  uint32_t* dm_bm = nullptr;       // membership bitmap (== dm for a 1-bit map)
  int64_t bm_words = 0;
  int32_t dm_kmin = 0;
  uint32_t dm_span = 0;
  int32_t dm_lw = 0;
};

struct hx_agg {
  hx_ctx* ctx = nullptr;
  void* base = nullptr;
  unsigned long long* sums = nullptr;   // [cap_groups]
  unsigned long long* cnts = nullptr;   // [cap_groups]
  struct AggMeta* meta = nullptr;       // device
  int64_t cap_groups = 1;               // host-known upper bound of n_groups
  int n_gdims = 0;
  const hx_ht* gdim_ht[HX_MAX_GDIMS] = {nullptr, nullptr, nullptr};
  std::vector<const hx_ht*> deps;       // every HT the pipeline probed (error check)
};

// Device-computed group layout of one pipeline (written by the prepare kernel).
struct AggMeta {
  long long n_groups;
  int32_t jstride[HX_MAX_JOINS];   // per join: stride of its rank in the group index (0 = none)
  int32_t n_ranks[HX_MAX_GDIMS];
  int32_t error;
  int32_t pad;
};

namespace hx {
// the union-router merge / exchange go through NCCL (a communicator of > 1 ranks, or forced)
inline bool use_collectives(const hx_ctx* ctx) {
  return ctx->comm && (ctx->nranks > 1 || ctx->force_coll);
}
// launchers implemented in hx_build.cu / hx_probe.cu
int build_dim_ht(hx_ctx* ctx, const hx_table* dim, int32_t key_col, const hx_pred* preds,
                 int n_preds, int32_t group_col, int32_t group_lo, int32_t group_hi,
                 hx_ht** out, int flags = 0);
int ht_create(hx_ctx* ctx, const hx_table* dim, int32_t key_col, const hx_pred* preds,
              int n_preds, int32_t group_col, int32_t group_lo, int32_t group_hi, hx_ht** out,
              int flags = 0);
int ht_enqueue_build(hx_ctx* ctx, hx_ht* ht, cudaStream_t stream = nullptr);
void ht_destroy(hx_ht* ht);
// switch a table's builds to a direct map over keys [kmin, kmin + span) with 2^lw-bit entries
int ht_enable_direct(hx_ctx* ctx, hx_ht* ht, int32_t kmin, uint32_t span, int lw);
int probe_agg(hx_ctx* ctx, const hx_table* fact, const hx_query_shape* shape,
              hx_ht* const* hts, int n_hts, hx_agg* agg, bool fresh);
int k1_occupancy(hx_ctx* ctx);
// host-resident K1 over the blocks a shared router hands out (hx_pipeline_probe_agg_routed)
int probe_agg_routed(hx_ctx* ctx, const hx_table* fact, const hx_query_shape* sh, hx_ht* const* hts,
                     int n_hts, hx_agg* agg, hx_shared_router* router, int64_t block_rows,
                     int64_t* n_blocks);
struct K1Prepared;  // a resolved K1 launch (hx_probe.cu)
long long k1_group_bound(const hx_query_shape* sh, hx_ht* const* hts, int n_hts);
int agg_alloc(hx_ctx* ctx, hx_agg* agg, long long cap_groups, const hx_query_shape* sh,
              hx_ht* const* hts);
int k1_setup(hx_ctx* ctx, const hx_table* fact, const hx_query_shape* sh, hx_ht* const* hts,
             int n_hts, const hx_agg* agg, K1Prepared** out);
struct StageRing;   // device staging ring for host-resident fact tables (hx_probe.cu)
constexpr int64_t kHostBlockRows = int64_t(1) << 21;  // mem-move block: 8 MB per int32 column
// k1_prepare (clears the group arrays, publishes the group-space shape) on stream s
int k1_enqueue_prepare(hx_ctx* ctx, const K1Prepared* k, bool fresh, cudaStream_t s);
// [prepare on the main stream if `prepare`] then K1 on the main stream
int k1_enqueue(hx_ctx* ctx, const K1Prepared* k, bool fresh, cudaEvent_t e0, cudaEvent_t e1,
               StageRing* ring = nullptr, bool prepare = true);
bool k1_is_host(const K1Prepared* k);
int ring_create(hx_ctx* ctx, const K1Prepared* k, int64_t block_rows, StageRing** out);
void ring_destroy(hx_ctx* ctx, StageRing* r);
void k1_free(K1Prepared* k);
int64_t k1_bytes(const K1Prepared* k);          // streamed bytes (rows x 4 x staged columns)
int k1_gathered_cols(const K1Prepared* k);      // measure columns gathered for passing rows
const int32_t* table_col(const hx_table* t, int32_t col_id);
bool table_has_col(const hx_table* t, int32_t col_id);
cudaEvent_t pooled_event(hx_ctx* ctx);

// Record `e` on `s`; under stream capture it becomes an external event-record node of the
// graph (so the host can wait on / time each replay), otherwise a plain record.
inline cudaError_t record_event(cudaEvent_t e, cudaStream_t s) {
  cudaStreamCaptureStatus st = cudaStreamCaptureStatusNone;
  cudaError_t r = cudaStreamIsCapturing(s, &st);
  if (r != cudaSuccess) return r;
  return st == cudaStreamCaptureStatusActive ? cudaEventRecordWithFlags(e, s, cudaEventRecordExternal)
                                             : cudaEventRecord(e, s);
}
}  // namespace hx

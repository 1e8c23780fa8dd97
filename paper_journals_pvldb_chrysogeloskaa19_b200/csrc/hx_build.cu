// hx_build.cu — K2: dimension filter + open-addressing hash-table build (§8(a) a3).
//
// PAPER.md:1160-1163 §6.1: Proteus runs SSB with broadcast-hash-join plans; the build side
// of each join is the filtered dimension. PAPER.md:1019-1022 §4.3: the hash table is
// operator state allocated by the device-local memory manager. PAPER.md:231-233: the build
// phase needs atomics. The paper does not describe its table layout (R15), so
// this is a B200-first design:
//   * one HBM allocation per table (header, dense-rank maps, slot array) so the fused
//     probe kernel sees one L2-friendly region;
//   * 8-byte slots {int32 key, int32 rank} written with one 64-bit CAS, linear probing from
//     the first slot of a 16-byte bucket (one 128-bit load per probe step), capacity = next
//     pow2 >= 4 * passing rows (load factor <= 0.25), Fibonacci hashing;
//   * sizing happens ON THE DEVICE (count kernel -> rank kernel writes log2cap), so a query
//     enqueues build -> probe -> merge with no host round trip (CUDA-graph capturable);
//   * inserts are warp-cooperative: the warp takes one pending key at a time and inspects
//     32 consecutive slots with one coalesced load + ballot, CAS-ing the first empty one.
#include <cub/block/block_scan.cuh>

#include "hx_internal.cuh"

namespace hx {

namespace {

constexpr unsigned kFull = 0xFFFFFFFFu;

struct BuildParams {
  const int32_t* key;
  const int32_t* group;                // nullptr: membership only
  const int32_t* pcol[HX_MAX_PREDS];
  DevPred preds[HX_MAX_PREDS];
  int32_t n_preds;
  int64_t n_rows;
  HtHeader* hdr;
  int32_t* c2r;
  int32_t* r2c;
  unsigned long long* slots;
  uint32_t* bloom;
  int32_t group_lo, domain, max_log2cap, max_bloom_log2w;
  // direct map (nullptr: hash table)
  uint32_t* dm;
  int64_t dm_words;
  uint32_t* dm_bm;  // membership bitmap over the same keys (nullptr when the map is 1-bit)
  int64_t bm_words;
  int32_t dm_kmin;
  uint32_t dm_span;
  int32_t dm_lw;
  int32_t identity_ranks;  // HX_BUILD_IDENTITY_RANKS: rank = code - group_lo for every code
};

__device__ __forceinline__ bool row_pass(const BuildParams& p, int64_t i) {
  bool ok = true;
#pragma unroll
  for (int k = 0; k < HX_MAX_PREDS; ++k)
    if (k < p.n_preds) ok = ok && pred_pass(p.preds[k], __ldg(p.pcol[k] + i));
  return ok;
}

// The dense ranks of the present group codes (exclusive scan of the flags), the rank->code
// map, and the table capacity / Bloom size from the passing count: run by ONE CTA of NT
// threads once every flag and counter is final.
template <int NT>
__device__ void rank_codes(const BuildParams& p) {
  using Scan = cub::BlockScan<int, NT>;
  __shared__ typename Scan::TempStorage tmp;
  __shared__ int running;
  if (threadIdx.x == 0) running = 0;
  __syncthreads();
  if (p.group) {
    for (int base = 0; base < p.domain; base += NT) {
      const int code = base + threadIdx.x;
      const int flag = code < p.domain ? (p.identity_ranks ? 1 : __ldcg(p.c2r + code)) : 0;
      int excl, total;
      Scan(tmp).ExclusiveSum(flag, excl, total);
      const int rank = running + excl;
      if (flag) {
        p.c2r[code] = rank;
        p.r2c[rank] = code + p.group_lo;
      }
      __syncthreads();
      if (threadIdx.x == 0) running += total;
      __syncthreads();
    }
  }
  if (threadIdx.x == 0) {
    const int n = __ldcg(&p.hdr->n_keys);
    // load factor <= 1/4, or <= 1/2 for a table that would exceed kBigTableBytes at 1/4 (a
    // large table's L2 footprint costs more than its slightly longer probe chains; measured
    // at SF100: customer 600 K keys, 32 -> 16 MB, HT-path Q4.1 -33%, Q3.1 -9%)
    const long long inv = (long long)n * kLoadInv * 8 > kBigTableBytes ? 2 : kLoadInv;
    int lg = kMinLog2Cap;
    while (lg < p.max_log2cap && (1ll << lg) < inv * n) ++lg;
    p.hdr->log2cap = lg;
    p.hdr->bloom_log2w = min(p.max_bloom_log2w, bloom_log2w_for(n));
    p.hdr->n_ranks = p.group ? running : 1;
    p.hdr->max_log2cap = p.max_log2cap;
    p.hdr->group_lo = p.group_lo;
    p.hdr->domain = p.domain;
  }
}

// Count passing rows and their key range; flag the group codes present among them; zero the
// Bloom filter (all of its words) and, for a direct-map build, the map and bitmap (the
// insert kernel runs after this one). The LAST CTA to finish (threadfence + counter) then
// ranks the codes and sizes the table, so the build needs no separate rank launch.
// The passing count, key range and code flags are reduced in shared memory first: one set of
// global atomics per CTA (same-address atomics from every warp serialise at one L2 slice).
constexpr int kFilterThreads = 256;
constexpr int kSmemCodeWords = 1024;  // code-presence bitmap in shared memory (32 K codes)
__global__ void __launch_bounds__(kFilterThreads) k2_filter_mark(BuildParams p) {
  __shared__ uint32_t s_codes[kSmemCodeWords];
  __shared__ int s_n;
  __shared__ uint32_t s_min, s_max;
  const bool smem_codes = p.group && p.domain <= kSmemCodeWords * 32;
  const int code_words = smem_codes ? (p.domain + 31) / 32 : 0;
  for (int w = threadIdx.x; w < code_words; w += blockDim.x) s_codes[w] = 0u;
  if (threadIdx.x == 0) {
    s_n = 0;
    s_min = 0xFFFFFFFFu;
    s_max = 0u;
  }
  __syncthreads();
  int local = 0;
  uint32_t emin = 0xFFFFFFFFu, emax = 0u;
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  const int64_t gtid = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
  const int64_t bloom_words = int64_t(1) << p.max_bloom_log2w;
  for (int64_t i = gtid; i < bloom_words; i += stride) p.bloom[i] = 0u;
  if (p.dm) {
    for (int64_t i = gtid; i < p.dm_words; i += stride) p.dm[i] = 0u;
    if (p.dm_bm)
      for (int64_t i = gtid; i < p.bm_words; i += stride) p.dm_bm[i] = 0u;
  }
  for (int64_t i = gtid; i < p.n_rows; i += stride) {
    if (!row_pass(p, i)) continue;
    ++local;
    const int32_t key = __ldg(p.key + i);
    if (key == kEmptyKey) atomicExch(&p.hdr->error, HX_EINVAL);  // reserved key
    emin = min(emin, key_enc(key));
    emax = max(emax, key_enc(key));
    if (p.group) {
      int32_t code = __ldg(p.group + i) - p.group_lo;
      if (code < 0 || code >= p.domain)
        atomicExch(&p.hdr->error, HX_EINVAL);
      else if (smem_codes)
        atomicOr(s_codes + (code >> 5), 1u << (code & 31));
      else
        p.c2r[code] = 1;  // benign race: every writer stores 1
    }
  }
#pragma unroll
  for (int o = 16; o > 0; o >>= 1) local += __shfl_xor_sync(kFull, local, o);
  emin = __reduce_min_sync(kFull, emin);
  emax = __reduce_max_sync(kFull, emax);
  if ((threadIdx.x & 31) == 0 && local) {
    atomicAdd(&s_n, local);
    atomicMin(&s_min, emin);
    atomicMax(&s_max, emax);
  }
  __syncthreads();
  if (threadIdx.x == 0 && s_n) {
    atomicAdd(&p.hdr->n_keys, s_n);
    atomicMax(&p.hdr->kmin_inv, ~s_min);
    atomicMax(&p.hdr->kmax_enc, s_max);
  }
  for (int w = threadIdx.x; w < code_words; w += blockDim.x)
    for (uint32_t bits = s_codes[w]; bits; bits &= bits - 1u)
      p.c2r[w * 32 + __ffs(bits) - 1] = 1;
  // last-CTA-done: publish this CTA's flags and counters, then count it in
  __shared__ bool last;
  __threadfence();
  __syncthreads();
  if (threadIdx.x == 0) last = atomicAdd(&p.hdr->done, 1u) == gridDim.x - 1;
  __syncthreads();
  if (!last) return;
  __threadfence();
  rank_codes<kFilterThreads>(p);
}

// Empty the slots in use (their count is only known on the device; the Bloom filter was
// zeroed by the filter kernel).
__global__ void k2_clear(BuildParams p) {
  const int64_t cap = 1ll << p.hdr->log2cap;
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < cap; i += stride)
    p.slots[i] = kEmptySlot;
}

// Warp-cooperative linear-probing insert of every passing row.
__global__ void k2_insert(BuildParams p) {
  const int lane = threadIdx.x & 31;
  const int log2cap = p.hdr->log2cap;
  const int blw = p.hdr->bloom_log2w;
  const uint32_t mask = (1u << log2cap) - 1u;
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  for (int64_t base = (int64_t)blockIdx.x * blockDim.x + (threadIdx.x & ~31); base < p.n_rows;
       base += stride) {
    const int64_t i = base + lane;
    bool has = i < p.n_rows && row_pass(p, i);
    int32_t key = 0, rank = 0;
    if (has) {
      key = __ldg(p.key + i);
      if (p.group) {
        int32_t code = __ldg(p.group + i) - p.group_lo;
        has = code >= 0 && code < p.domain;  // out-of-range codes were flagged by the filter
        if (has) rank = p.c2r[code];
      }
      if (has) atomicOr(p.bloom + bloom_word(key, blw), bloom_mask(key));
    }
    // optimistic pass: every lane CASes its key into its home slot at once (at load factor
    // <= 1/4 most succeed in one round trip); only keys whose home slot was taken enter the
    // warp-cooperative probe below
    if (has) {
      const unsigned long long packed =
          ((unsigned long long)(uint32_t)rank << 32) | (unsigned long long)(uint32_t)key;
      const unsigned long long old = atomicCAS(p.slots + ht_home(key, log2cap), kEmptySlot, packed);
      if (old == kEmptySlot) {
        has = false;
      } else if ((int32_t)(uint32_t)old == key) {
        atomicExch(&p.hdr->error, HX_EDUPKEY);
        has = false;
      }
    }
    unsigned pending = __ballot_sync(kFull, has);
    while (pending) {
      const int leader = __ffs(pending) - 1;
      pending &= pending - 1;
      const int32_t k = __shfl_sync(kFull, key, leader);
      const int32_t r = __shfl_sync(kFull, rank, leader);
      const unsigned long long packed =
          ((unsigned long long)(uint32_t)r << 32) | (unsigned long long)(uint32_t)k;
      const uint32_t home = ht_home(k, log2cap);
      bool done = false;
      for (uint32_t off = 0; !done && off <= mask; off += 32) {
        const uint32_t s = (home + off + lane) & mask;
        const unsigned long long v = __ldcg(p.slots + s);
        unsigned mk = __ballot_sync(kFull, v != kEmptySlot && (int32_t)(uint32_t)v == k);
        unsigned any = mk | __ballot_sync(kFull, v == kEmptySlot);
        while (any) {
          const int f = __ffs(any) - 1;
          if (mk & (1u << f)) {  // the key is already present: duplicate primary key
            if (lane == 0) atomicExch(&p.hdr->error, HX_EDUPKEY);
            done = true;
            break;
          }
          unsigned long long old = 0;
          if (lane == f) old = atomicCAS(p.slots + ((home + off + f) & mask), kEmptySlot, packed);
          old = __shfl_sync(kFull, old, f);
          if (old == kEmptySlot) {
            done = true;
            break;
          }
          if ((int32_t)(uint32_t)old == k) {  // a concurrent insert of the same key won
            if (lane == 0) atomicExch(&p.hdr->error, HX_EDUPKEY);
            done = true;
            break;
          }
          any &= ~(1u << f);  // taken by another key: try the next free slot of the window
        }
      }
    }
  }
}

// Direct-map build: entry (key - kmin) |= rank + 1 for every passing row, plus the key's
// bit in the membership bitmap and the Bloom filter (K1 stages whichever of the three fits
// its shared memory). A key outside the map (the dimension changed since the plan sized it)
// or a rank too wide for the entry sets HX_ECAPACITY; a key already present sets
// HX_EDUPKEY (the entries are non-zero).
__global__ void k2_dm_insert(BuildParams p) {
  const uint32_t vmask = dm_vmask(p.dm_lw);
  const int blw = p.hdr->bloom_log2w;
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < p.n_rows; i += stride) {
    if (!row_pass(p, i)) continue;
    const int32_t key = __ldg(p.key + i);
    uint32_t rank = 0;
    if (p.group) {
      const int32_t code = __ldg(p.group + i) - p.group_lo;
      if (code < 0 || code >= p.domain) continue;  // flagged by the filter kernel
      rank = (uint32_t)p.c2r[code];
    }
    const uint32_t u = (uint32_t)key - (uint32_t)p.dm_kmin;
    if (u >= p.dm_span || rank + 1u > vmask) {
      atomicExch(&p.hdr->error, HX_ECAPACITY);
      continue;
    }
    const uint64_t bit = (uint64_t)u << p.dm_lw;
    const uint32_t sh = (uint32_t)bit & 31u;
    const uint32_t old = atomicOr(p.dm + (bit >> 5), (rank + 1u) << sh);
    if ((old >> sh) & vmask) atomicExch(&p.hdr->error, HX_EDUPKEY);
    if (p.dm_bm) atomicOr(p.dm_bm + (u >> 5), 1u << (u & 31u));
    atomicOr(p.bloom + bloom_word(key, blw), bloom_mask(key));
  }
}

int ceil_log2(int64_t x) {
  int l = 0;
  while ((1ll << l) < x) ++l;
  return l;
}

}  // namespace

// Validate a build and allocate its table (no kernels launched).
int ht_create(hx_ctx* ctx, const hx_table* dim, int32_t key_col, const hx_pred* preds,
              int n_preds, int32_t group_col, int32_t group_lo, int32_t group_hi, hx_ht** out,
              int flags) {
  HX_REQUIRE(ctx && dim && out, HX_EINVAL, "hx_build_dim_ht: null argument");
  HX_REQUIRE(n_preds >= 0 && n_preds <= HX_MAX_PREDS && (n_preds == 0 || preds), HX_EINVAL,
             "hx_build_dim_ht: bad predicate list");
  HX_REQUIRE(dim->placement != HX_PLACE_HOST_PINNED && dim->placement != HX_PLACE_HOST_MAPPED,
             HX_EUNSUPPORTED,
             "hx_build_dim_ht: dimension tables must be device resident");
  HX_REQUIRE(dim->n_rows < (1ll << 30), HX_ECAPACITY, "hx_build_dim_ht: dimension too large");
  BuildParams p{};
  p.key = table_col(dim, key_col);
  HX_REQUIRE(table_has_col(dim, key_col), HX_EINVAL, "hx_build_dim_ht: key column not in table");
  p.n_preds = n_preds;
  for (int k = 0; k < n_preds; ++k) {
    p.pcol[k] = table_col(dim, preds[k].col_id);
    HX_REQUIRE(table_has_col(dim, preds[k].col_id), HX_EINVAL, "hx_build_dim_ht: predicate column not in table");
    HX_REQUIRE(preds[k].kind == HX_PRED_RANGE ||
                   (preds[k].kind == HX_PRED_IN && preds[k].n_in >= 1 && preds[k].n_in <= 4),
               HX_EINVAL, "hx_build_dim_ht: bad predicate");
    p.preds[k] = DevPred{k, preds[k].kind, preds[k].lo, preds[k].hi, preds[k].n_in,
                         {preds[k].in[0], preds[k].in[1], preds[k].in[2], preds[k].in[3]}};
  }
  int64_t domain = 1;
  if (group_col >= 0) {
    p.group = table_col(dim, group_col);
    HX_REQUIRE(table_has_col(dim, group_col), HX_EINVAL, "hx_build_dim_ht: group column not in table");
    HX_REQUIRE(group_hi >= group_lo && (int64_t)group_hi - group_lo < (1 << 24), HX_EINVAL,
               "hx_build_dim_ht: bad group code range");
    domain = (int64_t)group_hi - group_lo + 1;
  }
  HX_REQUIRE((flags & ~HX_BUILD_IDENTITY_RANKS) == 0, HX_EINVAL, "hx_build_dim_ht: bad flags");
  p.identity_ranks = (flags & HX_BUILD_IDENTITY_RANKS) && group_col >= 0 ? 1 : 0;
  p.n_rows = dim->n_rows;
  p.group_lo = group_lo;
  p.domain = (int32_t)domain;
  p.max_log2cap = std::max(kMinLog2Cap, ceil_log2(kLoadInv * std::max<int64_t>(dim->n_rows, 1)));

  hx_ht* ht = new hx_ht();
  ht->ctx = ctx;
  ht->domain = (int32_t)domain;
  ht->group_lo = group_lo;
  ht->has_group = group_col >= 0;
  ht->identity_ranks = p.identity_ranks != 0;
  ht->max_log2cap = p.max_log2cap;
  ht->dim_rows = dim->n_rows;
  p.max_bloom_log2w = bloom_log2w_for(std::max<int64_t>(dim->n_rows, 1));
  ht->max_bloom_log2w = p.max_bloom_log2w;
  const size_t maps = (sizeof(HtHeader) + 2 * domain * sizeof(int32_t) + 255) & ~size_t(255);
  const size_t slot_bytes = (size_t(1) << p.max_log2cap) * sizeof(unsigned long long);
  ht->bytes = maps + slot_bytes + (size_t(1) << p.max_bloom_log2w) * sizeof(uint32_t);
  cudaError_t e = cudaMallocAsync(&ht->base, ht->bytes, ctx->stream);
  if (e != cudaSuccess) {
    delete ht;
    return cuda_fail(e, "cudaMallocAsync(hash table)", __FILE__, __LINE__);
  }
  ht->hdr = reinterpret_cast<HtHeader*>(ht->base);
  ht->code_to_rank = reinterpret_cast<int32_t*>(ht->hdr + 1);
  ht->rank_to_code = ht->code_to_rank + domain;
  ht->slots = reinterpret_cast<unsigned long long*>(static_cast<char*>(ht->base) + maps);
  p.hdr = ht->hdr;
  p.c2r = ht->code_to_rank;
  p.r2c = ht->rank_to_code;
  p.slots = ht->slots;
  ht->bloom = reinterpret_cast<uint32_t*>(static_cast<char*>(ht->base) + maps + slot_bytes);
  p.bloom = ht->bloom;
  ht->build = new BuildParams(p);
  *out = ht;
  return HX_OK;
}

// Enqueue the build (a header memset + 2 kernels for a direct map, + 3 for a hash table;
// asynchronous; CUDA-graph capturable). Re-running a build
// on the same table rebuilds it from scratch.
int ht_enqueue_build(hx_ctx* ctx, hx_ht* ht, cudaStream_t stream) {
  const BuildParams& p = *static_cast<const BuildParams*>(ht->build);
  cudaStream_t s = stream ? stream : ctx->stream;
  HX_CK(cudaMemsetAsync(ht->base, 0, sizeof(HtHeader) + p.domain * sizeof(int32_t), s));
  const int64_t want = (p.n_rows + 255) / 256;
  const int grid = (int)std::max<int64_t>(1, std::min<int64_t>(want, (int64_t)ctx->n_sms * 8));
  // (at most 2 CTAs per SM for the filter: its per-CTA flush is the serial part)
  const int fgrid = (int)std::max<int64_t>(1, std::min<int64_t>(want, (int64_t)ctx->n_sms * 2));
  k2_filter_mark<<<fgrid, kFilterThreads, 0, s>>>(p);  // + zeroing, + rank (last CTA)
  HX_CK_LAUNCH("k2_filter_mark");
  if (p.dm) {  // direct map (+ bitmap, Bloom filter) instead of slots
    k2_dm_insert<<<grid, 256, 0, s>>>(p);
    HX_CK_LAUNCH("k2_dm_insert");
    ctx->launches += 2;
    return HX_OK;
  }
  const int64_t slots_max = int64_t(1) << p.max_log2cap;
  const int cgrid = (int)std::min<int64_t>((slots_max + 255) / 256, (int64_t)ctx->n_sms * 16);
  k2_clear<<<cgrid, 256, 0, s>>>(p);
  HX_CK_LAUNCH("k2_clear");
  k2_insert<<<grid, 256, 0, s>>>(p);
  HX_CK_LAUNCH("k2_insert");
  ctx->launches += 3;
  return HX_OK;
}

int ht_enable_direct(hx_ctx* ctx, hx_ht* ht, int32_t kmin, uint32_t span, int lw) {
  HX_REQUIRE(lw >= 0 && lw <= 5 && ((uint64_t)span << lw) < (uint64_t(1) << 32), HX_EINVAL,
             "direct map: bad width or span");
  BuildParams& p = *static_cast<BuildParams*>(ht->build);
  const int64_t words = dm_words_for(span, lw);
  const int64_t bm_words = lw > 0 ? dm_words_for(span, 0) : 0;
  if (ht->dm) cudaFreeAsync(ht->dm, ctx->stream);
  ht->dm = nullptr;
  HX_CK(cudaMallocAsync(&ht->dm, (size_t)(words + bm_words) * sizeof(uint32_t), ctx->stream));
  ht->dm_words = words;
  ht->dm_bm = lw > 0 ? ht->dm + words : ht->dm;
  ht->bm_words = lw > 0 ? bm_words : words;
  p.dm_bm = lw > 0 ? ht->dm + words : nullptr;
  p.bm_words = bm_words;
  ht->dm_kmin = kmin;
  ht->dm_span = span;
  ht->dm_lw = lw;
  p.dm = ht->dm;
  p.dm_words = words;
  p.dm_kmin = kmin;
  p.dm_span = span;
  p.dm_lw = lw;
  return HX_OK;
}

void ht_destroy(hx_ht* ht) {
  if (ht->dm) cudaFreeAsync(ht->dm, ht->ctx->stream);
  if (ht->base) cudaFreeAsync(ht->base, ht->ctx->stream);
  delete static_cast<BuildParams*>(ht->build);
  delete ht;
}

int build_dim_ht(hx_ctx* ctx, const hx_table* dim, int32_t key_col, const hx_pred* preds,
                 int n_preds, int32_t group_col, int32_t group_lo, int32_t group_hi,
                 hx_ht** out, int flags) {
  hx_ht* ht = nullptr;
  int rc = ht_create(ctx, dim, key_col, preds, n_preds, group_col, group_lo, group_hi, &ht, flags);
  if (rc != HX_OK) return rc;
  rc = ht_enqueue_build(ctx, ht);
  if (rc != HX_OK) {
    ht_destroy(ht);
    return rc;
  }
  *out = ht;
  return HX_OK;
}

}  // namespace hx

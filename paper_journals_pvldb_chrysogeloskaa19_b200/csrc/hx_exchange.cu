// hx_exchange.cu — the hash-partitioned join's data movement:
// hash-pack (kernel K3: group a table's rows by the part of their key) and the hash-routing
// exchange (part p -> rank p over NCCL). PAPER.md:405-428 §3.1 (hash-based routing; the
// hash-pack operator), PAPER.md:557-561, 582-587 (Fig. 1d/e hash-partitioned joins).
//
// K3 is a three-pass radix scatter over whole rows, bound by HBM (each row is read twice and
// written once: 12 B per 4-byte column):
//   k3_count    each CTA counts the rows of its contiguous chunk per part (shared-memory
//               counters), writes counts[part][cta];
//   k3_scan     one CTA: exclusive scan over (part, cta) -> each CTA's write cursor per part,
//               and the part offsets;
//   k3_scatter  each CTA re-reads its chunk tile by tile, regroups each tile (every column at
//               once: more bytes in flight) by part in shared memory and writes one
//               contiguous run per part (coalesced).
#include <cub/block/block_scan.cuh>

#include <algorithm>
#include <cstdlib>
#include <vector>

#include "hx_internal.cuh"

namespace hx {
namespace {

constexpr int kK3Threads = 512;


// (murmur3's fmix32 finaliser, then multiply-shift range reduction. NOT the hash tables'
// Fibonacci hash: a part function correlated with the bucket function would crowd each part's
// keys into 1/n_parts of its table's buckets — measured 15 s instead of 10 ms for Q3.1 with
// 8 parts when both were Fibonacci hashes.)
__host__ __device__ __forceinline__ int part_of(int32_t key, int n_parts) {
  uint32_t h = (uint32_t)key;
  h ^= h >> 16;
  h *= 0x85EBCA6Bu;
  h ^= h >> 13;
  h *= 0xC2B2AE35u;
  h ^= h >> 16;
  return (int)(((unsigned long long)h * (unsigned)n_parts) >> 32);
}

struct K3Params {
  const int32_t* key;
  const int32_t* src[HX_MAX_COLS];
  int32_t* dst[HX_MAX_COLS];
  int32_t n_cols;
  int32_t n_parts;
  int64_t n_rows;
  int64_t chunk;            // rows per CTA
  int64_t* counts;          // [n_parts][grid]: counts, then (after the scan) write cursors
  int64_t* part_offsets;    // [n_parts + 1]
};

// Row counts per part of a CTA's chunk: 16-byte key loads, two in flight per thread, one
// shared-memory atomic per row (SF100, 8 parts: 0.70 -> 0.43 ms; measured and rejected:
// warp-aggregated atomics via __match_any_sync 1.20 ms, per-thread 8-bit counters packed in a
// register 0.64 ms)
__global__ void __launch_bounds__(kK3Threads) k3_count(K3Params p) {
  __shared__ unsigned int cnt[HX_MAX_PARTS];
  for (int i = threadIdx.x; i < p.n_parts; i += blockDim.x) cnt[i] = 0;
  __syncthreads();
  const int64_t r0 = (int64_t)blockIdx.x * p.chunk;
  const int64_t r1 = min(p.n_rows, r0 + p.chunk);
  auto count = [&](int32_t key) { atomicAdd(&cnt[part_of(key, p.n_parts)], 1u); };
  int64_t r = r0;
  if ((reinterpret_cast<uintptr_t>(p.key + r0) & 15u) == 0) {
    constexpr int kStep = 8 * kK3Threads;
    for (; r + kStep <= r1; r += kStep) {
      const int4 a = __ldg(reinterpret_cast<const int4*>(p.key + r) + threadIdx.x);
      const int4 b = __ldg(reinterpret_cast<const int4*>(p.key + r) + kK3Threads + threadIdx.x);
      count(a.x); count(a.y); count(a.z); count(a.w);
      count(b.x); count(b.y); count(b.z); count(b.w);
    }
  }
  for (r += threadIdx.x; r < r1; r += blockDim.x) count(__ldg(p.key + r));  // the rest
  __syncthreads();
  for (int i = threadIdx.x; i < p.n_parts; i += blockDim.x)
    p.counts[(int64_t)i * gridDim.x + blockIdx.x] = cnt[i];
}

// exclusive scan of counts in (part, cta) order: the rows of part 0 from every CTA, then
// part 1, ... — each CTA's rows of a part land contiguously at its cursor
__global__ void __launch_bounds__(1024) k3_scan(K3Params p, int grid) {
  using Scan = cub::BlockScan<long long, 1024>;
  __shared__ typename Scan::TempStorage tmp;
  __shared__ long long running;
  if (threadIdx.x == 0) running = 0;
  __syncthreads();
  const int64_t n = (int64_t)p.n_parts * grid;
  for (int64_t base = 0; base < n; base += 1024) {
    const int64_t i = base + threadIdx.x;
    const long long v = i < n ? p.counts[i] : 0;
    long long excl, total;
    Scan(tmp).ExclusiveSum(v, excl, total);
    if (i < n) {
      p.counts[i] = running + excl;
      if (i % grid == 0) p.part_offsets[i / grid] = running + excl;
    }
    __syncthreads();
    if (threadIdx.x == 0) running += total;
    __syncthreads();
  }
  if (threadIdx.x == 0) p.part_offsets[p.n_parts] = running;
}

// Scatter through shared memory: each 2,048-row tile is first regrouped by part in shared
// memory (one column at a time), then written out as one contiguous run per part (~T/P rows),
// so the writes coalesce like a copy instead of landing row by row in P places.
constexpr int kK3Tile = 2048;
constexpr int kK3PerThread = kK3Tile / kK3Threads;
__global__ void __launch_bounds__(kK3Threads) k3_scatter(K3Params p) {
  __shared__ unsigned long long cur[HX_MAX_PARTS];  // next output row of each part
  __shared__ unsigned tcnt[HX_MAX_PARTS], tstart[HX_MAX_PARTS];
  extern __shared__ int32_t buf[];  // [n_cols][kK3Tile]: every column of the tile in flight at once
  __shared__ uint8_t psorted[kK3Tile];
  const int tid = threadIdx.x, lane = tid & 31;
  for (int i = tid; i < p.n_parts; i += blockDim.x)
    cur[i] = (unsigned long long)p.counts[(int64_t)i * gridDim.x + blockIdx.x];
  const int64_t r0 = (int64_t)blockIdx.x * p.chunk;
  const int64_t r1 = min(p.n_rows, r0 + p.chunk);
  for (int64_t t0 = r0; t0 < r1; t0 += kK3Tile) {
    const int rows = (int)(r1 - t0 < kK3Tile ? r1 - t0 : (int64_t)kK3Tile);
    for (int i = tid; i < p.n_parts; i += blockDim.x) tcnt[i] = 0;
    __syncthreads();
    int mypart[kK3PerThread], myslot[kK3PerThread];
#pragma unroll
    for (int k = 0; k < kK3PerThread; ++k) {
      const int j = tid + k * kK3Threads;
      const bool live = j < rows;
      const int part = live ? part_of(__ldg(p.key + t0 + j), p.n_parts) : 0;
      const unsigned act = __ballot_sync(0xFFFFFFFFu, live);
      int slot = 0;
      if (live) {  // warp-aggregated slot within the tile's part
        const unsigned same = __match_any_sync(act, part);
        const int leader = __ffs(same) - 1;
        unsigned base = 0;
        if (lane == leader) base = atomicAdd(&tcnt[part], (unsigned)__popc(same));
        base = __shfl_sync(same, base, leader);
        slot = (int)(base + __popc(same & ((1u << lane) - 1u)));
      }
      mypart[k] = part;
      myslot[k] = live ? slot : -1;
    }
    __syncthreads();
    if (tid < 32) {  // exclusive scan of the (<= 64) tile counts
      const unsigned a = lane < p.n_parts ? tcnt[lane] : 0u;
      const unsigned b = lane + 32 < p.n_parts ? tcnt[lane + 32] : 0u;
      unsigned ia = a;
#pragma unroll
      for (int o = 1; o < 32; o <<= 1) {
        const unsigned v = __shfl_up_sync(0xFFFFFFFFu, ia, o);
        if (lane >= o) ia += v;
      }
      const unsigned tot_a = __shfl_sync(0xFFFFFFFFu, ia, 31);
      unsigned ib = b;
#pragma unroll
      for (int o = 1; o < 32; o <<= 1) {
        const unsigned v = __shfl_up_sync(0xFFFFFFFFu, ib, o);
        if (lane >= o) ib += v;
      }
      if (lane < p.n_parts) tstart[lane] = ia - a;
      if (lane + 32 < p.n_parts) tstart[lane + 32] = tot_a + ib - b;
    }
    __syncthreads();
#pragma unroll
    for (int k = 0; k < kK3PerThread; ++k)
      if (myslot[k] >= 0) psorted[tstart[mypart[k]] + myslot[k]] = (uint8_t)mypart[k];
    for (int c = 0; c < p.n_cols; ++c) {
      const int32_t* src = p.src[c] + t0;
      int32_t* b = buf + c * kK3Tile;
#pragma unroll
      for (int k = 0; k < kK3PerThread; ++k)
        if (myslot[k] >= 0) b[tstart[mypart[k]] + myslot[k]] = __ldg(src + tid + k * kK3Threads);
    }
    __syncthreads();
    for (int c = 0; c < p.n_cols; ++c) {
      int32_t* dst = p.dst[c];
      const int32_t* b = buf + c * kK3Tile;
      for (int i = tid; i < rows; i += kK3Threads) {
        const int part = psorted[i];
        dst[cur[part] + (unsigned)(i - (int)tstart[part])] = b[i];
      }
    }
    __syncthreads();
    for (int i = tid; i < p.n_parts; i += blockDim.x) cur[i] += tcnt[i];
    __syncthreads();
  }
}

// ---- k3_scatter_tma: the same scatter with the tiles staged by the bulk-copy engine --------
// r02: each CTA's next tile (every column, the key among them) is copied HBM -> shared memory
// with cp.async.bulk while the current one is regrouped, so no thread waits on a global load;
// the regroup is a permutation (src_of: the tile row of each part-sorted position) applied
// column by column while writing, instead of copying every column into a second buffer.
// Requires 16-byte aligned column bases and CTA chunks of whole tiles (checked by the host).
__device__ __forceinline__ uint32_t k3_smem_u32(const void* p) {
  return (uint32_t)__cvta_generic_to_shared(p);
}
__device__ __forceinline__ void k3_mbar_init(uint64_t* bar, uint32_t count) {
  asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(k3_smem_u32(bar)), "r"(count));
}
__device__ __forceinline__ void k3_mbar_expect_tx(uint64_t* bar, uint32_t bytes) {
  asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(k3_smem_u32(bar)),
               "r"(bytes)
               : "memory");
}
__device__ __forceinline__ void k3_mbar_wait(uint64_t* bar, uint32_t parity) {
  asm volatile(
      "{\n"
      ".reg .pred p;\n"
      "K3WAIT_%=:\n"
      "mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n"
      "@!p bra K3WAIT_%=;\n"
      "}\n" ::"r"(k3_smem_u32(bar)),
      "r"(parity)
      : "memory");
}
__device__ __forceinline__ void k3_bulk_g2s(void* dst, const void* src, uint32_t bytes, uint64_t* bar) {
  asm volatile(
      "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
          k3_smem_u32(dst)),
      "l"(src), "r"(bytes), "r"(k3_smem_u32(bar))
      : "memory");
}

constexpr int kK3MaxTmaCols = 12;
constexpr size_t k3_tma_smem(int n_cols) { return 2 * (size_t)n_cols * kK3Tile * 4; }

__global__ void __launch_bounds__(kK3Threads) k3_scatter_tma(K3Params p, int key_c) {
  __shared__ unsigned long long cur[HX_MAX_PARTS];
  __shared__ unsigned tcnt[HX_MAX_PARTS], tstart[HX_MAX_PARTS];
  __shared__ uint16_t src_of[kK3Tile];
  __shared__ uint8_t psorted[kK3Tile];
  __shared__ __align__(8) uint64_t full[2];
  extern __shared__ __align__(128) int32_t stage[];  // [2][n_cols][kK3Tile]
  const int tid = threadIdx.x, lane = tid & 31;
  for (int i = tid; i < p.n_parts; i += blockDim.x) {
    cur[i] = (unsigned long long)p.counts[(int64_t)i * gridDim.x + blockIdx.x];
    tcnt[i] = 0;
  }
  if (tid == 0) {
    k3_mbar_init(full + 0, 1);
    k3_mbar_init(full + 1, 1);
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  __syncthreads();
  const int64_t r0 = (int64_t)blockIdx.x * p.chunk;
  const int64_t r1 = min(p.n_rows, r0 + p.chunk);
  const size_t stage_elems = (size_t)p.n_cols * kK3Tile;
  auto issue = [&](int64_t t0, int s) {  // one thread: every column of the tile at t0
    const int rows = (int)(r1 - t0 < kK3Tile ? r1 - t0 : (int64_t)kK3Tile);
    const uint32_t bytes = (uint32_t)(rows & ~3) * 4u;
    k3_mbar_expect_tx(full + s, bytes * p.n_cols);
    if (bytes)
      for (int c = 0; c < p.n_cols; ++c)
        k3_bulk_g2s(stage + s * stage_elems + (size_t)c * kK3Tile, p.src[c] + t0, bytes, full + s);
  };
  if (tid == 0 && r0 < r1) issue(r0, 0);
  uint32_t phases = 0u;  // bit s: the parity the next wait on stage s expects
  int s = 0;
  for (int64_t t0 = r0; t0 < r1; t0 += kK3Tile, s ^= 1) {
    const int rows = (int)(r1 - t0 < kK3Tile ? r1 - t0 : (int64_t)kK3Tile);
    // the other stage was last used by the previous tile, finished at the barrier below
    if (tid == 0 && t0 + kK3Tile < r1) issue(t0 + kK3Tile, s ^ 1);
    k3_mbar_wait(full + s, (phases >> s) & 1u);
    phases ^= 1u << s;
    int32_t* st = stage + s * stage_elems;
    const int copied = rows & ~3;
    if (copied != rows) {  // the chunk's last <= 3 rows: not a 16-byte multiple
      if (tid < rows - copied)
        for (int c = 0; c < p.n_cols; ++c) st[(size_t)c * kK3Tile + copied + tid] = p.src[c][t0 + copied + tid];
      __syncthreads();
    }
    const int32_t* keys = st + (size_t)key_c * kK3Tile;
    int mypart[kK3PerThread], myslot[kK3PerThread];
#pragma unroll
    for (int k = 0; k < kK3PerThread; ++k) {
      const int j = tid + k * kK3Threads;
      const bool live = j < rows;
      const int part = live ? part_of(keys[j], p.n_parts) : 0;
      const unsigned act = __ballot_sync(0xFFFFFFFFu, live);
      int slot = 0;
      if (live) {  // warp-aggregated slot within the tile's part
        const unsigned same = __match_any_sync(act, part);
        const int leader = __ffs(same) - 1;
        unsigned base = 0;
        if (lane == leader) base = atomicAdd(&tcnt[part], (unsigned)__popc(same));
        base = __shfl_sync(same, base, leader);
        slot = (int)(base + __popc(same & ((1u << lane) - 1u)));
      }
      mypart[k] = part;
      myslot[k] = live ? slot : -1;
    }
    __syncthreads();
    if (tid < 32) {  // exclusive scan of the (<= 64) tile counts
      const unsigned a = lane < p.n_parts ? tcnt[lane] : 0u;
      const unsigned b = lane + 32 < p.n_parts ? tcnt[lane + 32] : 0u;
      unsigned ia = a, ib = b;
#pragma unroll
      for (int o = 1; o < 32; o <<= 1) {
        const unsigned va = __shfl_up_sync(0xFFFFFFFFu, ia, o);
        const unsigned vb = __shfl_up_sync(0xFFFFFFFFu, ib, o);
        if (lane >= o) ia += va, ib += vb;
      }
      const unsigned tot_a = __shfl_sync(0xFFFFFFFFu, ia, 31);
      if (lane < p.n_parts) tstart[lane] = ia - a;
      if (lane + 32 < p.n_parts) tstart[lane + 32] = tot_a + ib - b;
    }
    __syncthreads();
#pragma unroll
    for (int k = 0; k < kK3PerThread; ++k)
      if (myslot[k] >= 0) {
        const int pos = (int)tstart[mypart[k]] + myslot[k];
        src_of[pos] = (uint16_t)(tid + k * kK3Threads);
        psorted[pos] = (uint8_t)mypart[k];
      }
    __syncthreads();
    for (int i = tid; i < rows; i += kK3Threads) {  // part-sorted position i: one run per part
      const int part = psorted[i];
      const unsigned long long o = cur[part] + (unsigned)(i - (int)tstart[part]);
      const int j = src_of[i];
      for (int c = 0; c < p.n_cols; ++c) p.dst[c][o] = st[(size_t)c * kK3Tile + j];
    }
    __syncthreads();
    for (int i = tid; i < p.n_parts; i += blockDim.x) {
      cur[i] += tcnt[i];
      tcnt[i] = 0;
    }
    __syncthreads();
  }
}

int table_alloc_like(hx_ctx* ctx, const hx_table* t, int64_t n_rows, hx_table** out) {
  hx_table* o = new hx_table();
  o->ctx = ctx;
  o->n_cols = t->n_cols;
  o->n_rows = n_rows;
  o->placement = HX_PLACE_COPY;
  o->owned = true;
  for (int c = 0; c < t->n_cols; ++c) {
    o->col_id[c] = t->col_id[c];
    o->dev[c] = nullptr;
    if (n_rows == 0) continue;
    cudaError_t e = cudaMallocAsync(&o->dev[c], ((size_t)n_rows * 4 + 255) & ~size_t(255), ctx->stream);
    if (e != cudaSuccess) {
      for (int d = 0; d < c; ++d) cudaFreeAsync(o->dev[d], ctx->stream);
      delete o;
      return cuda_fail(e, "cudaMallocAsync(partitioned column)", __FILE__, __LINE__);
    }
  }
  *out = o;
  return HX_OK;
}

}  // namespace
}  // namespace hx

using namespace hx;

extern "C" {

int hx_hash_partition(hx_ctx* ctx, const hx_table* t, int32_t key_col, int n_parts,
                      hx_table** out, int64_t* part_offsets) {
  HX_REQUIRE(ctx && t && out && part_offsets, HX_EINVAL, "hx_hash_partition: null argument");
  HX_REQUIRE(n_parts >= 1 && n_parts <= HX_MAX_PARTS, HX_EINVAL, "hx_hash_partition: bad n_parts");
  HX_REQUIRE(t->placement == HX_PLACE_COPY || t->placement == HX_PLACE_VIEW, HX_EUNSUPPORTED,
             "hx_hash_partition: the table must be device resident");
  HX_REQUIRE(table_has_col(t, key_col), HX_EINVAL, "hx_hash_partition: key column not in table");
  HX_CK(cudaSetDevice(ctx->device));
  hx_table* o = nullptr;
  int rc = table_alloc_like(ctx, t, t->n_rows, &o);
  if (rc != HX_OK) return rc;
  if (t->n_rows == 0) {
    for (int i = 0; i <= n_parts; ++i) part_offsets[i] = 0;
    *out = o;
    return HX_OK;
  }
  // the bulk-copy scatter when every column base is 16-byte aligned (CTA chunks are whole
  // tiles), else the load-based one; one wave of either (shared memory grows with the columns)
  int key_c = 0;
  bool tma = t->n_cols <= kK3MaxTmaCols && std::getenv("HX_K3_LDG") == nullptr;
  for (int c = 0; c < t->n_cols; ++c) {
    tma = tma && (reinterpret_cast<uintptr_t>(t->dev[c]) & 15u) == 0;
    if (t->col_id[c] == key_col) key_c = c;
  }
  const size_t scatter_smem = tma ? k3_tma_smem(t->n_cols) : (size_t)t->n_cols * kK3Tile * sizeof(int32_t);
  const void* scatter_fn = tma ? (const void*)k3_scatter_tma : (const void*)k3_scatter;
  cudaFuncSetAttribute(scatter_fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)scatter_smem);
  int occ = 1;
  cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, scatter_fn, kK3Threads, scatter_smem);
  const int64_t grid = std::max<int64_t>(1, std::min<int64_t>((int64_t)ctx->n_sms * std::max(1, occ),
                                                             (t->n_rows + 4095) / 4096));
  K3Params p{};
  p.key = table_col(t, key_col);
  p.n_cols = t->n_cols;
  for (int c = 0; c < t->n_cols; ++c) {
    p.src[c] = t->dev[c];
    p.dst[c] = o->dev[c];
  }
  p.n_parts = n_parts;
  p.n_rows = t->n_rows;
  p.chunk = (t->n_rows + grid - 1) / grid;
  if (tma) p.chunk = (p.chunk + kK3Tile - 1) / kK3Tile * kK3Tile;  // whole (aligned) tiles
  void* scratch = nullptr;
  const size_t sbytes = sizeof(int64_t) * ((size_t)n_parts * grid + n_parts + 1);
  cudaError_t e = cudaMallocAsync(&scratch, sbytes, ctx->stream);
  if (e != cudaSuccess) {
    hx_table_free(o);
    return cuda_fail(e, "cudaMallocAsync(partition counters)", __FILE__, __LINE__);
  }
  p.counts = static_cast<int64_t*>(scratch);
  p.part_offsets = p.counts + (size_t)n_parts * grid;
  k3_count<<<(unsigned)grid, kK3Threads, 0, ctx->stream>>>(p);
  k3_scan<<<1, 1024, 0, ctx->stream>>>(p, (int)grid);
  if (tma)
    k3_scatter_tma<<<(unsigned)grid, kK3Threads, scatter_smem, ctx->stream>>>(p, key_c);
  else
    k3_scatter<<<(unsigned)grid, kK3Threads, scatter_smem, ctx->stream>>>(p);
  ctx->launches += 3;
  e = cudaGetLastError();
  if (e == cudaSuccess)
    e = cudaMemcpyAsync(part_offsets, p.part_offsets, sizeof(int64_t) * (n_parts + 1),
                        cudaMemcpyDeviceToHost, ctx->stream);
  cudaFreeAsync(scratch, ctx->stream);
  if (e == cudaSuccess) e = cudaStreamSynchronize(ctx->stream);
  if (e != cudaSuccess) {
    hx_table_free(o);
    return cuda_fail(e, "hx_hash_partition", __FILE__, __LINE__);
  }
  ctx->d2h_bytes += sizeof(int64_t) * (n_parts + 1);
  *out = o;
  return HX_OK;
}

int hx_exchange_partitions(hx_ctx* ctx, const hx_table* parted, const int64_t* part_offsets,
                           int n_parts, hx_table** out) {
  HX_REQUIRE(ctx && parted && part_offsets && out, HX_EINVAL, "hx_exchange_partitions: null argument");
  HX_REQUIRE(part_offsets[0] == 0 && part_offsets[n_parts] == parted->n_rows, HX_EINVAL,
             "hx_exchange_partitions: offsets do not match the table");
  HX_CK(cudaSetDevice(ctx->device));
  const int nr = ctx->comm ? ctx->nranks : 1;
  HX_REQUIRE(n_parts == nr, HX_EINVAL, "hx_exchange_partitions: n_parts must equal the rank count");
  if (!use_collectives(ctx)) {  // no exchange: this rank keeps its one part (a library-owned copy)
    hx_table* o = nullptr;
    int rc = table_alloc_like(ctx, parted, parted->n_rows, &o);
    if (rc != HX_OK) return rc;
    for (int c = 0; c < parted->n_cols; ++c)
      if (parted->n_rows)
        HX_CK(cudaMemcpyAsync(o->dev[c], parted->dev[c], (size_t)parted->n_rows * 4,
                              cudaMemcpyDeviceToDevice, ctx->stream));
    HX_CK(cudaStreamSynchronize(ctx->stream));
    *out = o;
    return HX_OK;
  }
  // part sizes of every rank: sizes[src * nr + dst]
  int64_t* dsz = nullptr;
  HX_CK(cudaMallocAsync(&dsz, sizeof(int64_t) * nr * (nr + 1), ctx->stream));
  std::vector<int64_t> mine(nr), sizes((size_t)nr * nr);
  for (int p = 0; p < nr; ++p) mine[p] = part_offsets[p + 1] - part_offsets[p];
  HX_CK(cudaMemcpyAsync(dsz, mine.data(), sizeof(int64_t) * nr, cudaMemcpyHostToDevice, ctx->stream));
  coll_log(ctx, HX_COLL_ALLGATHER, dsz, nr, 8);
  ncclResult_t r = ncclAllGather(dsz, dsz + nr, nr, ncclInt64, ctx->comm, ctx->stream);
  if (r != ncclSuccess) {
    cudaFreeAsync(dsz, ctx->stream);
    return fail(HX_ENCCL, std::string("ncclAllGather: ") + ncclGetErrorString(r));
  }
  HX_CK(cudaMemcpyAsync(sizes.data(), dsz + nr, sizeof(int64_t) * nr * nr, cudaMemcpyDeviceToHost,
                        ctx->stream));
  HX_CK(cudaStreamSynchronize(ctx->stream));
  cudaFreeAsync(dsz, ctx->stream);
  int64_t n_in = 0;
  std::vector<int64_t> recv_off(nr);
  for (int s = 0; s < nr; ++s) {
    recv_off[s] = n_in;
    n_in += sizes[(size_t)s * nr + ctx->rank];
  }
  hx_table* o = nullptr;
  int rc = table_alloc_like(ctx, parted, n_in, &o);
  if (rc != HX_OK) return rc;
  r = ncclGroupStart();
  for (int c = 0; c < parted->n_cols && r == ncclSuccess; ++c) {
    for (int peer = 0; peer < nr && r == ncclSuccess; ++peer) {
      const int64_t ns = part_offsets[peer + 1] - part_offsets[peer];
      const int64_t nrv = sizes[(size_t)peer * nr + ctx->rank];
      if (ns > 0) coll_log(ctx, HX_COLL_SEND, parted->dev[c] + part_offsets[peer], ns, 4, peer);
      if (ns > 0)
        r = ncclSend(parted->dev[c] + part_offsets[peer], (size_t)ns, ncclInt32, peer, ctx->comm,
                     ctx->stream);
      if (r == ncclSuccess && nrv > 0) coll_log(ctx, HX_COLL_RECV, o->dev[c] + recv_off[peer], nrv, 4, peer);
      if (r == ncclSuccess && nrv > 0)
        r = ncclRecv(o->dev[c] + recv_off[peer], (size_t)nrv, ncclInt32, peer, ctx->comm,
                     ctx->stream);
    }
  }
  const ncclResult_t r2 = ncclGroupEnd();
  if (r == ncclSuccess) r = r2;
  if (r != ncclSuccess) {
    hx_table_free(o);
    return fail(HX_ENCCL, std::string("hash-routing exchange: ") + ncclGetErrorString(r));
  }
  HX_CK(cudaStreamSynchronize(ctx->stream));
  *out = o;
  return HX_OK;
}

}  // extern "C"

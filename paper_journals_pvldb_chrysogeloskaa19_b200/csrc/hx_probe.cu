// hx_probe.cu — K1: the fused scan -> filter -> probe x k -> group-by aggregate pipeline
// (§8(a) a5), the one hot loop of HetExchange's GPU execution of an SSB query.
//
// What it computes follows Listing 1 pipeline 9: every GPU thread walks
// its share of the block (unpack), evaluates the predicate (filter), accumulates into a
// thread-local value, reduces over its neighbourhood and the neighbourhood leader adds the
// result to the pipeline state with one atomic (reduce; Fig. 3). SSB
// pipelines add the broadcast-hash-join probes between filter and reduce
// and a GROUP BY (the paper does not describe its group-by; R17).
//
// How (B200-first, not the paper's 2019 LLVM-generated sm_61 code):
//   * persistent CTAs (one per SM), each with one PRODUCER warp that streams lineorder tiles
//     (2560 rows x the query's streamed columns) from HBM into a shared-memory ring with
//     cp.async.bulk (the TMA bulk-copy engine) completing on mbarriers, L2 evict-first, and 20
//     CONSUMER warps that take the tiles two at a time while the next ones are in flight
//     (mem-move's "prefetch to the consumer's local memory", done at tile
//     granularity inside the kernel);
//   * each consumer lane owns 4 consecutive rows of each tile (one 128-bit shared-memory load
//     per column) and runs the pipeline stage-wise: predicates, the most selective join's
//     shared-memory structure, compaction of the survivors into a per-warp queue, then the
//     remaining joins for 32 queued rows at a time (one row per lane, lookups issued
//     together);
//   * joins are probed in direct maps (plans over dense keys: rank + 1 per key, exact, staged
//     in shared memory when they fit) or in open-addressing hash tables with shared-memory
//     Bloom filters (hx_build.cu); measure columns no stage reads are gathered for the rows
//     that pass every join instead of being streamed (late materialisation);
//   * GROUP BY: a dense per-CTA shared-memory table (int64 SUM, int32 COUNT) indexed by the
//     mixed radix of the probed dimensions' dense ranks, flushed with one global atomic per
//     non-empty group per CTA; ungrouped queries reduce warp -> CTA -> one global atomic.
#include <algorithm>
#include <cmath>
#include <cstdio>
#include <cstdlib>
#include <mutex>

#include "hx_internal.cuh"

namespace hx {

namespace {

constexpr unsigned kFull = 0xFFFFFFFFu;
// Consumer warps per CTA: every K1 instance is compiled for two counts and k1_setup picks one
// per pipeline. More warps hide more latency (L2 map reads) but their per-warp queues and carry
// buffers take shared memory from the filters and maps (measured at SF100: 26 warps 4.5%
// faster than 20 in sum; SF10 Q4.1 loses its customer bitmap with 26 and is 30% slower).
constexpr int kWarpsLo = 20, kWarpsHi = 26;
#ifndef HX_WARPS_HI_HT
#define HX_WARPS_HI_HT 26
#endif
constexpr int kWarpsHiHt = HX_WARPS_HI_HT;  // the hash-table instances' larger warp count
#ifndef HX_K1_STAGE_KB
#define HX_K1_STAGE_KB 160  // max shared memory for the tile ring (the rest: Bloom filters)
#endif
#ifndef HX_PROBE_HINT
#define HX_PROBE_HINT 0   // probe loads with an L2 evict_last hint (0: plain ld.global.nc;
                          // measured: the hint costs 2-9% on Q4.x)
#endif
#ifndef HX_GATHER_HINT
#define HX_GATHER_HINT 0  // gathered measures with an L2 evict_first hint (0: plain)
#endif
#ifndef HX_CLAIM_SPAN
#define HX_CLAIM_SPAN 1   // consecutive chunks claimed per shared atomic
#endif
#ifndef HX_BALLOT_COMPACT
#define HX_BALLOT_COMPACT 0  // survivors' queue slots from 8 ballots instead of a shuffle scan
#endif
#ifndef HX_DM_STATIC_CHUNKS
#define HX_DM_STATIC_CHUNKS 1  // chunk assignment of the direct-map instances (0: claimed)
#endif
#ifndef HX_HT_STATIC_CHUNKS
#define HX_HT_STATIC_CHUNKS 1  // ... of the hash-table instances
#endif
#ifndef HX_HT_CLAIM_NJ
#define HX_HT_CLAIM_NJ 4  // hash-table instances with at least this many joins claim chunks
#endif
#ifndef HX_STAGE_B_ROWS
#define HX_STAGE_B_ROWS 4  // hash-table stage B: probes in flight per lane (4 or 8)
#endif
#ifndef HX_HT_GIVEUP_MINCOLS
#define HX_HT_GIVEUP_MINCOLS 4  // hash tables: narrower pipelines never give up a ring stage
                                // for filters (SF100 HT K1 sum -0.45%: Q3.2 -9%, Q2.2 +3%)
#endif
#ifndef HX_HT_SEQ
#define HX_HT_SEQ 0       // hash-table joins probed one round trip per join in stage C
#endif
#ifndef HX_TAG_SLEEP_DM
#define HX_TAG_SLEEP_DM 32  // ns slept between polls of a ring slot's tile tag, direct-map
                            // instances (measured at SF100: K1 sum -0.55% vs spinning)
#endif
#ifndef HX_TAG_SLEEP_HT
#define HX_TAG_SLEEP_HT 0   // ... hash-table instances (0: spin; 32 ns measured +1.9%)
#endif
#ifndef HX_PROD_SLEEP
#define HX_PROD_SLEEP 128  // ns the producer sleeps between polls of a slot's empty barrier
#endif
#ifndef HX_K1_CTAS
#define HX_K1_CTAS 1    // resident CTAs per SM the launch bounds / smem budget target
                        // (one CTA per SM shares one copy of the Bloom filters)
#endif
constexpr int k1_threads(int warps) { return warps * 32 + 32; }  // + one producer warp
constexpr int kRowsPerThread = 4;          // R
#ifndef HX_K1_TILE_ROWS
#define HX_K1_TILE_ROWS 2560
#endif
// rows per ring stage (one bulk copy per column); independent of the warp count since warps
// claim chunks dynamically
constexpr int kTileRows = HX_K1_TILE_ROWS;  // T = 2560 rows
// A CHUNK is one consumer warp's unit of work: 256 consecutive rows of a tile, two halves of
// 128 (lane l holds rows 4l..4l+3 of each half: one conflict-free 128-bit shared-memory load
// per column and half). Warps claim chunks dynamically (a shared counter), so a warp that
// drew a chunk with many survivors does not hold the others back.
constexpr int kHalfRows = 32 * kRowsPerThread;             // 128
constexpr int kChunkRows = 2 * kHalfRows;                  // 256
constexpr int kChunksPerTile = kTileRows / kChunkRows;     // 10
static_assert(kTileRows % kChunkRows == 0, "a tile is a whole number of chunks");
// rows per K1 launch: whole tiles, < 2^32 - kTileRows (32-bit row offsets inside a launch)
constexpr int64_t kSegRows = int64_t(kTileRows) * (int64_t(1) << 20);  // 2.68e9 rows
constexpr int kCtasPerSm = HX_K1_CTAS;    // target residency (registers, smem budget)
constexpr int kMaxStageCols = 8;
constexpr int kSmemGroups = 1024;          // per-CTA group table capacity
// dynamic smem: [barriers 128 | head 8 cols x 4 rows | chunk scheduling | per-warp queues: 256
// row bytes (+ 256 group indices, hash-table instances) | per-warp carry buffers | groups |
// Bloom filters | direct maps | tile ring]. (The ungrouped final reduce writes the warps' partials
// at kSmemQueueOff once every consumer is done — all of those regions are dead by then — so it
// needs no region of its own.)
// ring depth cap and the depth pick_stages starts from, in tiles: the same bytes (4 x 2560 rows)
// whatever the tile size
constexpr int kMaxStages = 8 * 2560 / kTileRows;  // 80 KB per column
static_assert(kMaxStages >= 2 && kMaxStages <= 16, "ring depth");
constexpr int kBaseStages = (4 * 2560 + kTileRows - 1) / kTileRows;
static_assert(kBaseStages <= kMaxStages, "ring");
constexpr int kSmemBarOff = 0;                                    // 2 x kMaxStages x 8 B
constexpr int kSmemHeadOff = 2 * kMaxStages * 8;
constexpr int kSmemHeadBytes = 128;                               // kMaxStageCols x 4 x 4 B
// chunk scheduling: [next chunk counter | ring slot tags (the tile each slot was last filled
// with) x 8]
constexpr int kSmemCtlOff = kSmemHeadOff + kSmemHeadBytes;
constexpr int kSmemCtlBytes = (4 * (1 + kMaxStages) + 63) & ~63;
constexpr int kSmemQueueOff = kSmemCtlOff + kSmemCtlBytes;       // 320 (2560-row tiles)
static_assert(kSmemHeadOff - kSmemBarOff >= 2 * kMaxStages * 8, "barriers overlap the head rows");
static_assert(kSmemCtlBytes >= 4 * (1 + kMaxStages), "counter + slot tags");
static_assert(kSmemQueueOff % 64 == 0, "queues / carry buffers / group table alignment");
constexpr int kQueueRows = 2 * kRowsPerThread * 32;       // per warp: one tile pair's rows
constexpr int kCarryBytes = (HX_MAX_JOINS + 4) * 32 * 4;  // one CarryBuf per consumer warp
constexpr int smem_carry_off(bool dm, int warps) {
  return kSmemQueueOff + warps * kQueueRows * (dm ? 1 : 5);
}
constexpr int smem_fixed(bool dm, int warps) {
  return smem_carry_off(dm, warps) + warps * kCarryBytes;
}

struct JoinDev {
  int32_t c;                               // staged column of the FK
  const unsigned long long* slots;
  const HtHeader* hdr;
  const uint32_t* bloom;                   // the table's Bloom filter (global)
  int32_t bloom_words;                     // shared-memory words reserved for it (0: none)
  // direct map (dense keys; hx_internal.cuh): nullptr -> hash-table join
  const uint32_t* dm;
  int32_t dm_kmin;
  uint32_t dm_span;
  int32_t dm_lw;
  uint32_t dm_vmask;
  int32_t dm_words;
  int32_t dm_smem;                         // byte offset of its copy in the DM smem region (-1: L2)
  const uint32_t* bm;                      // its membership bitmap (1 bit per key of the range)
  int32_t bm_words;
  int32_t bm_smem;                         // byte offset of a staged bitmap (-1: none)
  int32_t in_s;                            // 1: its shared-memory structure runs in stage S
};

struct K1Params {
  const int32_t* col[kMaxStageCols];       // staged fact columns (table base + head offset)
  int32_t n_cols;
  int32_t stages;                          // tile ring depth (kBaseStages..kMaxStages)
  uint32_t stage_magic;                    // floor(2^32 / stages) + 1: i / stages = umulhi(i, magic)
                                           // exactly for i < 2^32 / stages (a CTA has < 2^21 tiles)
  int32_t prefetch;                        // L2 prefetch distance in tiles of this CTA (0: off)
  int32_t smem_fixed;                      // bytes before the group table (no per-warp queues
                                           // when every join resolves in stage S)
  int64_t n_rows;                          // rows after the head
  int64_t n_tiles;
  const int32_t* head_col[kMaxStageCols];  // misaligned head rows (read directly)
  int32_t head_rows;                       // 0..3
  int32_t n_preds;
  DevPred preds[HX_MAX_PREDS];
  JoinDev joins[HX_MAX_JOINS];
  int32_t agg_op, agg_a, agg_b;            // measure operands: staged column (if staged)
  // late materialisation: a measure column no predicate or join reads is not streamed; its
  // value is gathered (one 32-byte sector) for the rows that pass every join only
  int32_t ga, gb;                          // operand a / b gathered
  const int32_t* gat_a;                    // fact columns indexed by fact row
  const int32_t* gat_b;
  const AggMeta* meta;
  unsigned long long* g_sum;
  unsigned long long* g_cnt;
  int32_t smem_groups;                     // 0 for ungrouped instances
  int32_t filter_words;                    // sum of joins[].bloom_words
  int32_t dm_bytes;                        // shared memory of the staged direct maps
  // per-join bit masks (bit j = join j) of the shared-memory plan, tested with one
  // instruction against the constant bank instead of re-reading the join descriptors
  uint32_t m_dm;                           // direct-map join
  uint32_t m_dmsm;                         // its full map is staged in shared memory
  uint32_t m_bm;                           // its bitmap is staged in shared memory
  uint32_t m_ins;                          // its shared-memory structure runs in stage S
  uint32_t m_l2;                           // stage C reads its map from L2 (rank, or no
                                           // exact verdict yet)
  uint32_t m_l2s;                          // stage S reads its map from L2 on every row (no
                                           // shared-memory structure: exact verdict + rank)
  uint32_t m_res;                          // resolved in stage S (full map staged, or m_l2s)
  int32_t l2_hint;                         // 1: probe loads evict_last (0: evict_normal; A/B)
  int32_t ht_seq;                          // hash tables: stage C probes one join alone (ht_first
                                           // if still pending, else the first), the others
                                           // only for its hits
  int32_t ht_first;
};

// join kinds (uniform per launch: read from the kernel parameters)
// (DM: the kernel instance whose joins are all direct maps; hash-table instances have none)
__device__ __forceinline__ bool jbit(uint32_t m, int jx) { return (m >> jx) & 1u; }
template <bool DM>
__device__ __forceinline__ bool dm_smem(const K1Params& p, int jx) { return DM && jbit(p.m_dmsm, jx); }
template <bool DM>
__device__ __forceinline__ bool resolved_in_s(const K1Params& p, int jx) {
  return DM && jbit(p.m_dmsm & p.m_ins, jx);
}
template <bool DM>
__device__ __forceinline__ bool dm_l2(const K1Params& p, int jx) {
  return DM && jbit(p.m_l2, jx);
}
// Direct-map entry (rank + 1, or 0) of a key from the map's 32-bit word array
__device__ __forceinline__ uint32_t dm_bit(const JoinDev& d, int32_t key) {
  return ((uint32_t)key - (uint32_t)d.dm_kmin) << d.dm_lw;
}
__device__ __forceinline__ bool dm_in(const JoinDev& d, int32_t key) {
  return (uint32_t)key - (uint32_t)d.dm_kmin < d.dm_span;
}
__device__ __forceinline__ uint32_t dm_entry(const JoinDev& d, uint32_t word, uint32_t bit) {
  return __funnelshift_r(word, word, bit) & d.dm_vmask;  // shf.r.wrap: bit mod 32
}

// ---- PTX helpers: mbarrier, bulk copy, cache policies -------------------------------------
__device__ __forceinline__ uint32_t smem_u32(const void* p) {
  return (uint32_t)__cvta_generic_to_shared(p);
}
__device__ __forceinline__ void mbar_init(uint64_t* bar, uint32_t count) {
  asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(count));
}
__device__ __forceinline__ void mbar_arrive_expect_tx(uint64_t* bar, uint32_t bytes) {
  asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)),
               "r"(bytes)
               : "memory");
}
__device__ __forceinline__ void mbar_arrive(uint64_t* bar) {
  asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(smem_u32(bar)) : "memory");
}
__device__ __forceinline__ void mbar_wait(uint64_t* bar, uint32_t parity) {
  asm volatile(
      "{\n"
      ".reg .pred p;\n"
      "WAIT_%=:\n"
      "mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n"
      "@!p bra WAIT_%=;\n"
      "}\n" ::"r"(smem_u32(bar)),
      "r"(parity)
      : "memory");
}
__device__ __forceinline__ uint64_t policy_evict_first() {
  uint64_t pol;
  asm volatile("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(pol));
  return pol;
}
__device__ __forceinline__ uint64_t policy_evict_last() {
  uint64_t pol;
  asm volatile("createpolicy.fractional.L2::evict_last.b64 %0, 1.0;" : "=l"(pol));
  return pol;
}
__device__ __forceinline__ void bulk_g2s(void* dst, const void* src, uint32_t bytes,
                                         uint64_t* bar, uint64_t pol) {
  asm volatile(
      "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes.L2::cache_hint"
      " [%0], [%1], %2, [%3], %4;" ::"r"(smem_u32(dst)),
      "l"(src), "r"(bytes), "r"(smem_u32(bar)), "l"(pol)
      : "memory");
}
// Prefetch `bytes` (multiple of 16) of global memory into L2 (bulk engine; no completion).
__device__ __forceinline__ void bulk_prefetch_l2(const void* src, uint32_t bytes) {
  asm volatile("cp.async.bulk.prefetch.L2.global [%0], %1;" ::"l"(src), "r"(bytes) : "memory");
}
__device__ __forceinline__ uint64_t policy_evict_normal() {
  uint64_t pol;
  asm volatile("createpolicy.fractional.L2::evict_normal.b64 %0, 1.0;" : "=l"(pol));
  return pol;
}
// Loads of the probe structures (direct-map words, hash-table buckets) and of gathered
// measures, with an L2 eviction-priority hint: probes evict_last (the maps and tables stay
// L2-resident against the evict-first lineorder stream; ncu then counts their sectors as
// evict_last, which isolates the probe tables' L2 hit rate), gathers evict_first (read once).
// Not volatile: pure loads of read-only data that the compiler may schedule freely.
__device__ __forceinline__ uint32_t ld_hint(const uint32_t* p, uint64_t pol) {
  uint32_t v;
  asm("ld.global.nc.L2::cache_hint.u32 %0, [%1], %2;" : "=r"(v) : "l"(p), "l"(pol));
  return v;
}
__device__ __forceinline__ int32_t ld_hint(const int32_t* p, uint64_t pol) {
  int32_t v;
  asm("ld.global.nc.L2::cache_hint.s32 %0, [%1], %2;" : "=r"(v) : "l"(p), "l"(pol));
  return v;
}
__device__ __forceinline__ ulonglong2 ld_hint(const ulonglong2* p, uint64_t pol) {
  ulonglong2 v;
  asm("ld.global.nc.L2::cache_hint.v2.u64 {%0, %1}, [%2], %3;"
      : "=l"(v.x), "=l"(v.y)
      : "l"(p), "l"(pol));
  return v;
}
// The two policies of a K1 launch (created once per thread).
struct Pols {
  uint64_t probe, gather;
};
__device__ __forceinline__ uint32_t ld_probe(const uint32_t* p, const Pols& pol) {
  return HX_PROBE_HINT ? ld_hint(p, pol.probe) : __ldg(p);
}
__device__ __forceinline__ ulonglong2 ld_probe(const ulonglong2* p, const Pols& pol) {
  return HX_PROBE_HINT ? ld_hint(p, pol.probe) : __ldg(p);
}
__device__ __forceinline__ int32_t ld_gather(const int32_t* p, const Pols& pol) {
  return HX_GATHER_HINT ? ld_hint(p, pol.gather) : __ldg(p);
}
template <int W>
__device__ __forceinline__ void consumer_sync() {
  asm volatile("bar.sync 1, %0;" ::"n"(W * 32) : "memory");
}

__device__ __forceinline__ long long measure(int op, int32_t a, int32_t b) {
  if (op == HX_AGG_SUM_MUL) return (long long)a * (long long)b;
  if (op == HX_AGG_SUM_SUB) return (long long)a - (long long)b;
  return (long long)a;
}
// Per-warp view of one join's hash table (loaded once per CTA).
struct JoinState {
  const ulonglong2* buckets;  // 16-byte buckets of two {key, rank} slots
  int32_t c;                  // staged column of the FK
  int32_t shift;              // 33 - log2cap (bucket hash)
  uint32_t bmask;             // n_buckets - 1
  int32_t jstride;            // weight of this join's rank in the group index
  const uint32_t* sbloom;     // Bloom filter staged in shared memory (nullptr: none)
  int32_t blw;                // its log2 word count
};

// Same test as (word & bloom_mask(key)) == bloom_mask(key), in fewer instructions: the two
// bit positions are tested with rotates (shf.r.wrap takes the shift modulo 32). blw >= 1.
__device__ __forceinline__ bool bloom_pass(const JoinState& j, int32_t key) {
  const uint32_t h = bloom_hash(key);
  const uint32_t w = j.sbloom[h >> (32 - j.blw)];
  return (__funnelshift_r(w, w, h >> 6) & __funnelshift_r(w, w, h >> 11)) & 1u;
}

__device__ __forceinline__ uint32_t bucket_of(int32_t key, int shift) {
  return ((uint32_t)key * 2654435769u) >> shift;
}

// One probe step for one row: hit (rank returned), miss, or continue at the next bucket.
// Within a bucket slot 1 is filled only after slot 0, so an empty slot 1 proves a miss.
__device__ __forceinline__ void probe_step(const ulonglong2 v, int32_t key, bool& hit, bool& miss,
                                           int32_t& rank) {
  const bool h0 = (int32_t)(uint32_t)v.x == key;
  const bool h1 = (int32_t)(uint32_t)v.y == key;
  hit = h0 || h1;
  miss = !hit && (int32_t)(uint32_t)v.y == kEmptyKey;
  rank = (int32_t)((h0 ? v.x : v.y) >> 32);
}

template <bool GROUPED>
__device__ __forceinline__ void accumulate(const K1Params& p, bool smem_table,
                                           unsigned long long* s_sum, uint32_t* s_cnt,
                                           int32_t g, long long m, long long& acc_sum,
                                           long long& acc_cnt) {
  if (GROUPED) {
    if (smem_table) {
      // the shared-memory SUM is kept as two 32-bit words (sm_100 has no native 64-bit
      // shared atomic add): add the low word, carry into the high word on wrap-around —
      // exact modulo 2^64 like the int64 sum
      uint32_t* s_lo = reinterpret_cast<uint32_t*>(s_sum);
      uint32_t* s_hi = s_lo + p.smem_groups;
      const unsigned long long um = (unsigned long long)m;
      const uint32_t lo = (uint32_t)um, hi = (uint32_t)(um >> 32);
      const uint32_t old = atomicAdd(s_lo + g, lo);
      const uint32_t up = hi + (uint32_t)(old + lo < old);
      if (up) atomicAdd(s_hi + g, up);
      atomicAdd(s_cnt + g, 1u);
    } else {
      atomicAdd(p.g_sum + g, (unsigned long long)m);
      atomicAdd(p.g_cnt + g, 1ull);
    }
  } else {
    acc_sum += m;
    acc_cnt += 1;
  }
}

// Hash-table join whose Bloom filter runs on every row (the first filtered one in probe
// order), or -1. (Direct-map joins apply their shared-memory filters in stage S.)
template <int NJ, bool DM>
__device__ __forceinline__ int first_filter(const JoinState (&js)[HX_MAX_JOINS]) {
  int jf = -1;
#pragma unroll
  for (int jx = NJ - 1; jx >= 0; --jx)
    if (!DM && js[jx].sbloom) jf = jx;
  return jf;
}
template <int NJ, bool DM>
__device__ __forceinline__ bool all_resolved_in_s(const K1Params& p) {
  return DM && (p.m_res & ((1u << NJ) - 1u)) == ((1u << NJ) - 1u);
}
// 1 when stage B probes the first join in place (hash-table joins, no lineorder predicate,
// no filter on the first join).
template <int NJ, bool DM>
__device__ __forceinline__ int first_join_in_place(const K1Params& p,
                                                   const JoinState (&js)[HX_MAX_JOINS]) {
  return (!DM && NJ > 0 && p.n_preds == 0 && !js[0].sbloom) ? 1 : 0;
}
// Group-index origin: a direct map yields rank + 1, so each join contributes one extra
// stride, subtracted once up front.
template <int NJ, bool GROUPED, bool DM>
__device__ __forceinline__ int32_t group_origin(const JoinState (&js)[HX_MAX_JOINS]) {
  int32_t g = 0;
#pragma unroll
  for (int jx = 0; jx < NJ; ++jx)
    if (GROUPED && DM) g -= js[jx].jstride;
  return g;
}

// A queued row for stage C, by value: the FK of every join, the measure operands, and the
// group-index part known so far (or ~next_bucket of a deferred first-join probe).
struct CarryEntry {
  int32_t key[HX_MAX_JOINS];
  int32_t a, b, g;
  uint32_t row;  // fact row (gathered measures)
};
// A stage-C row that passed, whose accumulation is deferred by one batch so that its gathered
// measure operands (issued loads) arrive while the next batch runs (latency hiding).
struct Pending {
  int32_t g, a, b;
  bool alive;
};
// Per-warp buffer of the (< 32) queued rows carried to the next tile (SoA, one slot per lane).
struct CarryBuf {
  int32_t key[HX_MAX_JOINS][32];
  int32_t a[32], b[32], g[32];
  uint32_t row[32];
};

// Entry idx of the combined sequence [carried rows..., this tile's queue...].
template <int NJ, bool DM>
__device__ __forceinline__ CarryEntry load_entry(const K1Params& p,
                                                 const JoinState (&js)[HX_MAX_JOINS],
                                                 const CarryBuf* cb, int n_carry,
                                                 const uint8_t* q_row, const int32_t* q_g,
                                                 bool carry_g, const int32_t* wcol0,
                                                 const int32_t* wcol1, uint32_t wrow0,
                                                 uint32_t wrow1, int stride, int idx) {
  CarryEntry e;
  if (idx < n_carry) {
#pragma unroll
    for (int jx = 0; jx < NJ; ++jx) e.key[jx] = cb->key[jx][idx];
    e.a = p.ga ? 0 : cb->a[idx];
    e.b = p.gb ? 0 : cb->b[idx];
    e.g = cb->g[idx];
    e.row = (p.ga | p.gb) ? cb->row[idx] : 0u;
  } else {
    const int i = idx - n_carry;
    const int q = q_row[i];  // bit 7: which tile of the pair; bits 0-6: row in the warp's slice
    const int32_t* wcol = (q & 128) ? wcol1 : wcol0;
    const int r = q & 127;
#pragma unroll
    for (int jx = 0; jx < NJ; ++jx)
      e.key[jx] = wcol[js[jx].c * stride + r];
    e.a = p.ga ? 0 : wcol[p.agg_a * stride + r];
    e.b = p.gb ? 0 : wcol[p.agg_b * stride + r];
    e.g = carry_g ? q_g[i] : 0;
    e.row = ((q & 128) ? wrow1 : wrow0) + (uint32_t)r;
  }
  return e;
}

// Stage C for one row: the remaining shared-memory filters, then the probes of every join
// not yet resolved issued together (one L2 round trip), then measure + group atomic.
template <int NJ, bool GROUPED, bool DM>
__device__ __forceinline__ void stage_c_row(const K1Params& p, const JoinState (&js)[HX_MAX_JOINS],
                                            const unsigned char* sdm, const CarryEntry& e,
                                            int j0, int jf, bool smem_table,
                                            unsigned long long* s_sum, uint32_t* s_cnt,
                                            long long& acc_sum, long long& acc_cnt, Pending& pd,
                                            const Pols& pol) {
  // (direct maps: the group index is computed here from scratch; stage S only filtered)
  int32_t gg = DM ? group_origin<NJ, GROUPED, DM>(js) : e.g;
  bool alive = true;
  uint32_t b[NJ > 0 ? NJ : 1];
  uint32_t wdm[NJ > 0 ? NJ : 1];
  uint32_t pend = 0;
  // direct-map joins not resolved in stage S: their shared-memory structures first (a full
  // map resolves the join, a bitmap or Bloom filter only drops rows) ...
#pragma unroll
  for (int jx = 0; jx < NJ; ++jx) {
    const JoinDev& d = p.joins[jx];
    if (!DM) continue;
    // the stage-S join: its filter already ran; a full map is read again for the rank
    if (jbit(p.m_ins, jx) && !(GROUPED && dm_smem<DM>(p, jx))) continue;
    const int32_t key = e.key[jx];
    if (dm_smem<DM>(p, jx)) {
      const uint32_t bit = dm_bit(d, key);
      const uint32_t* w = reinterpret_cast<const uint32_t*>(sdm + d.dm_smem);
      const uint32_t v = dm_entry(d, dm_in(d, key) ? w[bit >> 5] : 0u, bit);
      alive = alive && v != 0u;
      if (GROUPED) gg += (int32_t)v * js[jx].jstride;
    } else if (jbit(p.m_bm, jx)) {
      const uint32_t u = (uint32_t)key - (uint32_t)d.dm_kmin;
      const uint32_t* w = reinterpret_cast<const uint32_t*>(sdm + d.bm_smem);
      alive = alive && u < d.dm_span && ((w[u >> 5] >> (u & 31u)) & 1u);
    } else if (js[jx].sbloom) {
      alive = alive && bloom_pass(js[jx], key);
    }
  }
  // ... then the maps read from L2 (one 32-bit load each, only for rows still alive), issued
  // together with the hash probes below
#pragma unroll
  for (int jx = 0; jx < NJ; ++jx) {
    const JoinDev& d = p.joins[jx];
    wdm[jx] = 0u;
    if (dm_l2<DM>(p, jx) && alive && dm_in(d, e.key[jx]))
      wdm[jx] = ld_probe(d.dm + (dm_bit(d, e.key[jx]) >> 5), pol);
  }
#pragma unroll
  for (int jx = 0; jx < NJ; ++jx) {
    if (DM) {  // direct map: resolved above or in stage S
      b[jx] = 0u;
    } else if (jx < j0) {  // resume a deferred probe of the first join
      const bool deferred = gg < 0;
      b[jx] = deferred ? ~(uint32_t)gg : 0u;
      pend |= (uint32_t)deferred << jx;
    } else {
      b[jx] = bucket_of(e.key[jx], js[jx].shift);
      pend |= 1u << jx;
      if (jx != jf && js[jx].sbloom) alive = alive && bloom_pass(js[jx], e.key[jx]);
    }
  }
  if (j0 && gg < 0) gg = 0;  // deferred-probe encoding (stage B runs only without direct maps)
#pragma unroll
  for (int jx = 0; jx < NJ; ++jx) {
    const JoinDev& d = p.joins[jx];
    if (!dm_l2<DM>(p, jx)) continue;
    const uint32_t v = dm_entry(d, wdm[jx], dm_bit(d, e.key[jx]));
    alive = alive && v != 0u;
    if (GROUPED) gg += (int32_t)v * js[jx].jstride;
  }
  if (!alive) pend = 0;
  // (hash tables, p.ht_seq) one join alone (p.ht_first, the likeliest miss), the others only for its hits:
  // the open-addressing tables are large and mostly missed, so fewer probes beat one round trip
  uint32_t later = 0;
  if ((HX_HT_SEQ || p.ht_seq) && !DM) {
    const uint32_t fb = 1u << p.ht_first;
    const uint32_t first = (pend & fb) ? fb : pend & (0u - pend);
    later = pend & ~first;
    pend = first;
  }
  while (pend) {
    ulonglong2 v[NJ > 0 ? NJ : 1];
#pragma unroll
    for (int jx = 0; jx < NJ; ++jx)
      if ((pend >> jx) & 1u) v[jx] = ld_probe(js[jx].buckets + b[jx], pol);
#pragma unroll
    for (int jx = 0; jx < NJ; ++jx) {
      if (!((pend >> jx) & 1u)) continue;
      bool hit, miss;
      int32_t rank;
      probe_step(v[jx], e.key[jx], hit, miss, rank);
      if (hit) gg += rank * js[jx].jstride;
      alive = alive && !miss;
      pend &= ~((uint32_t)(hit || miss) << jx);
      b[jx] = (b[jx] + 1) & js[jx].bmask;
    }
    if (!alive) pend = later = 0;
    if (!pend && later) {
      pend = later;
      later = 0;
    }
  }
  Pending cur{gg, e.a, e.b, alive};
  if (alive) {  // issue the gathers now, consume them one batch later
    if (p.ga) cur.a = ld_gather(p.gat_a + e.row, pol);
    if (p.gb) cur.b = ld_gather(p.gat_b + e.row, pol);
  }
  if (pd.alive)
    accumulate<GROUPED>(p, smem_table, s_sum, s_cnt, pd.g, measure(p.agg_op, pd.a, pd.b), acc_sum,
                        acc_cnt);
  pd = cur;
}

// Process a PAIR of staged tiles (two consecutive tiles of this CTA, so the per-iteration
// costs — compaction, the stage-C batch bookkeeping, the carry — are paid once per 256 rows
// of a warp). Warp w owns rows [w*128, w*128+128) of each tile; lane l holds the 4
// consecutive rows w*128 + 4l .. +3 of each, read with one 128-bit shared-memory load per
// column and tile (512 contiguous bytes per warp: conflict-free). Row k of a lane (k = 0..7)
// is row (k & 3) of its slice of tile k >> 2. Column c, row r of a tile is at
// sbase[c * stride + r]; a missing second tile has rows_valid 0.
//   stage A  predicates on lineorder columns, branch-free;
//   stage S  (direct maps) the shared-memory structure of the most selective join: full map,
//            membership bitmap or Bloom filter;
//   stage F  (hash tables) the first join's Bloom filter; stage B (no predicate, no filter)
//            the first join probed in place, 4 independent 128-bit L2 loads in flight;
//   compact  survivors are appended to a per-warp queue (warp prefix sum of the lanes'
//            counts), so the remaining joins run with every lane busy;
//   stage C  in full batches of 32 queued rows, one row per lane: the remaining filters,
//            then the lookups / probes of ALL remaining joins issued together (one L2 round
//            trip), the measure and the group-table atomic.
template <int NJ, bool GROUPED, bool DM>
__device__ __forceinline__ void process_tile(const K1Params& p, const JoinState (&js)[HX_MAX_JOINS],
                                             const unsigned char* sdm, const int32_t* sbase0,
                                             const int32_t* sbase1, uint32_t frow0,
                                             uint32_t frow1, int stride, int rows_valid0,
                                             int rows_valid1, int warp, int lane,
                                             bool smem_table,
                                             unsigned long long* s_sum, uint32_t* s_cnt,
                                             uint8_t* q_row, int32_t* q_g, CarryBuf* cb,
                                             int& n_carry, long long& acc_sum,
                                             long long& acc_cnt, Pending& pd, const Pols& pol) {
  constexpr int R = kRowsPerThread;  // rows per lane per tile
  const int wbase = warp * (32 * R);
  const int r0 = wbase + lane * R;
  const int32_t* tb[2] = {sbase0 + r0, sbase1 + r0};
  uint32_t m = 0;
  if (rows_valid0 == kHalfRows) {  // full halves (all but the last): no per-row bound checks
    m = rows_valid1 == kHalfRows ? (1u << (2 * R)) - 1u : rows_valid1 == 0 ? (1u << R) - 1u : 0u;
  }
  if (m == 0u) {
#pragma unroll
    for (int k = 0; k < R; ++k) {
      m |= (uint32_t)(r0 + k < rows_valid0) << k;
      m |= (uint32_t)(r0 + k < rows_valid1) << (R + k);
    }
  }
  if (__ballot_sync(kFull, m) == 0) return;
  // the 8 values of staged column c for this lane
  auto load8 = [&](int c, int32_t (&v)[2 * R]) {
#pragma unroll
    for (int h = 0; h < 2; ++h) {
      const int4 x = *reinterpret_cast<const int4*>(tb[h] + c * stride);
      v[h * R + 0] = x.x;
      v[h * R + 1] = x.y;
      v[h * R + 2] = x.z;
      v[h * R + 3] = x.w;
    }
  };

  // stage A: lineorder predicates (kind is uniform: one branch per predicate, not per row)
  for (int q = 0; q < p.n_preds; ++q) {
    const DevPred& pr = p.preds[q];
    int32_t vv[2 * R];
    load8(pr.c, vv);
    if (pr.kind == HX_PRED_RANGE) {
      const uint32_t lo = (uint32_t)pr.lo, span = (uint32_t)pr.hi - (uint32_t)pr.lo;
#pragma unroll
      for (int k = 0; k < 2 * R; ++k)
        if (((uint32_t)vv[k] - lo) > span) m &= ~(1u << k);
    } else {
#pragma unroll
      for (int k = 0; k < 2 * R; ++k) {
        bool ok = false;
#pragma unroll
        for (int i = 0; i < 4; ++i) ok |= (i < pr.n_in) && vv[k] == pr.in[i];
        if (!ok) m &= ~(1u << k);
      }
    }
  }

  // stage F (hash tables): semi-join reduction with the shared-memory Bloom filter of the
  // first filtered join (the most selective: joins are in ascending pass fraction) on every
  // row; the other joins' filters are applied to the survivors in stage C. No false
  // negatives; the ~5% false positives are removed by the exact probe.
  const int jf = first_filter<NJ, DM>(js);
#pragma unroll
  for (int jx = 0; jx < NJ; ++jx) {
    if (jx != jf) continue;
    int32_t key[2 * R];
    load8(js[jx].c, key);
#pragma unroll
    for (int k = 0; k < 2 * R; ++k) if (!bloom_pass(js[jx], key[k])) m &= ~(1u << k);
  }

  // stage S (direct maps): the shared-memory structure of the most selective join, on every
  // row (branch-free). A full map clears a missing row (and, when it resolves the pipeline's
  // only join, yields the group index); a bitmap or Bloom filter only clears rows.
  const bool all_res = all_resolved_in_s<NJ, DM>(p);
  int32_t g[2 * R];
  const int32_t g0 = group_origin<NJ, GROUPED, DM>(js);
#pragma unroll
  for (int k = 0; k < 2 * R; ++k) g[k] = g0;
#pragma unroll
  for (int jx = 0; jx < NJ; ++jx) {
    const JoinDev& d = p.joins[jx];
    if (!DM || !jbit(p.m_ins, jx)) continue;
    int32_t key[2 * R];
    load8(d.c, key);
    if (dm_smem<DM>(p, jx)) {  // the full map: exact verdict and rank
      const uint32_t* w = reinterpret_cast<const uint32_t*>(sdm + d.dm_smem);
#pragma unroll
      for (int k = 0; k < 2 * R; ++k) {
        const uint32_t bit = dm_bit(d, key[k]);
        const uint32_t word = dm_in(d, key[k]) ? w[bit >> 5] : 0u;
        const uint32_t v = dm_entry(d, word, bit);
        if (v == 0u) m &= ~(1u << k);
        if (GROUPED && all_res) g[k] += (int32_t)v * js[jx].jstride;
      }
    } else if (jbit(p.m_bm, jx)) {  // its membership bitmap: exact verdict (rank from L2)
      const uint32_t* w = reinterpret_cast<const uint32_t*>(sdm + d.bm_smem);
#pragma unroll
      for (int k = 0; k < 2 * R; ++k) {
        const uint32_t u = (uint32_t)key[k] - (uint32_t)d.dm_kmin;
        const uint32_t word = u < d.dm_span ? w[u >> 5] : 0u;
        if (((word >> (u & 31u)) & 1u) == 0u) m &= ~(1u << k);
      }
    } else if (jbit(p.m_l2s, jx)) {  // its map from L2, every live row (8 loads in flight)
      uint32_t w[2 * R];
#pragma unroll
      for (int k = 0; k < 2 * R; ++k)
        w[k] = ((m >> k) & 1u) && dm_in(d, key[k]) ? ld_probe(d.dm + (dm_bit(d, key[k]) >> 5), pol) : 0u;
#pragma unroll
      for (int k = 0; k < 2 * R; ++k) {
        const uint32_t v = dm_entry(d, w[k], dm_bit(d, key[k]));
        if (v == 0u) m &= ~(1u << k);
        if (GROUPED && all_res) g[k] += (int32_t)v * js[jx].jstride;
      }
    } else {  // its Bloom filter: no false negatives
#pragma unroll
      for (int k = 0; k < 2 * R; ++k) if (!bloom_pass(js[jx], key[k])) m &= ~(1u << k);
    }
  }

  const int j0 = first_join_in_place<NJ, DM>(p, js);
  if (j0) {
    // stage B (hash tables): ONE probe step of the first join per row, 4 independent 128-bit
    // loads in flight per tile. Rows whose bucket was full without a verdict (rare at load
    // factor 1/4) are queued with ~next_bucket in place of the group index and finish in
    // stage C, so the warp never waits on its longest probe chain here.
    const JoinState& j = js[0];
    int32_t key[2 * R];
    load8(j.c, key);
    // HX_STAGE_B_ROWS rows' probes in flight per lane (4: one tile half at a time)
    constexpr int RB = HX_STAGE_B_ROWS;
#pragma unroll
    for (int h = 0; h < 2 * R / RB; ++h) {
      ulonglong2 v[RB];
      uint32_t b[RB];
#pragma unroll
      for (int k = 0; k < RB; ++k) {
        b[k] = bucket_of(key[h * RB + k], j.shift);
        if ((m >> (h * RB + k)) & 1u) v[k] = ld_probe(j.buckets + b[k], pol);
      }
#pragma unroll
      for (int k = 0; k < RB; ++k) {
        const int kk = h * RB + k;
        if (!((m >> kk) & 1u)) continue;
        bool hit, miss;
        int32_t rank;
        probe_step(v[k], key[kk], hit, miss, rank);
        g[kk] = hit ? rank * j.jstride : (int32_t)~((b[k] + 1) & j.bmask);
        if (miss) m &= ~(1u << kk);
      }
    }
  }

  if (NJ == 0 || all_res) {  // every join resolved: aggregate in place
    int32_t a8[2 * R] = {}, b8[2 * R] = {};
    if (!p.ga) load8(p.agg_a, a8);
    if (!p.gb) load8(p.agg_b, b8);
    if (p.ga | p.gb) {
      // late materialisation: the gathers of a passing row are issued now and consumed at the
      // lane's NEXT passing row (the one-deep Pending slot stage C uses), so their latency
      // overlaps the following chunks instead of stalling this one (gathers are planned only
      // when at most 1/16 of the rows pass: mostly one pending row per lane at a time)
      for (uint32_t bits = m; bits; bits &= bits - 1u) {
        const int k = __ffs(bits) - 1;
        int32_t gk = g0, ak = 0, bk = 0;
#pragma unroll
        for (int kk = 0; kk < 2 * R; ++kk)
          if (kk == k) gk = g[kk], ak = a8[kk], bk = b8[kk];
        const uint32_t row = (k < R ? frow0 : frow1) + r0 + (k & 3);
        Pending cur{gk, p.ga ? ld_gather(p.gat_a + row, pol) : ak,
                    p.gb ? ld_gather(p.gat_b + row, pol) : bk, true};
        if (pd.alive)
          accumulate<GROUPED>(p, smem_table, s_sum, s_cnt, pd.g, measure(p.agg_op, pd.a, pd.b),
                              acc_sum, acc_cnt);
        pd = cur;
      }
      return;
    }
    if (!GROUPED) {  // branch-free: predicated adds, one population count
      long long sum = 0;
#pragma unroll
      for (int k = 0; k < 2 * R; ++k)
        sum += ((m >> k) & 1u) ? measure(p.agg_op, a8[k], b8[k]) : 0ll;
      acc_sum += sum;
      acc_cnt += __popc(m);
      return;
    }
#pragma unroll
    for (int k = 0; k < 2 * R; ++k)
      if ((m >> k) & 1u)
        accumulate<GROUPED>(p, smem_table, s_sum, s_cnt, g[k], measure(p.agg_op, a8[k], b8[k]),
                            acc_sum, acc_cnt);
    return;
  }

  // compaction: append this warp's survivors to its queue — a warp prefix sum of the lanes'
  // survivor counts gives each lane its slots; a lane then writes only its surviving rows
  const bool carry_g = j0;
#if HX_BALLOT_COMPACT
  // row k of every lane: one ballot; its slot = the rows before it (earlier k, lower lanes)
  const uint32_t lt = (1u << lane) - 1u;
  int qn = 0;
#pragma unroll
  for (int k = 0; k < 2 * R; ++k) {
    const uint32_t b = __ballot_sync(kFull, (m >> k) & 1u);
    if ((m >> k) & 1u) {
      const int pos = qn + __popc(b & lt);
      q_row[pos] = (uint8_t)(((k >> 2) << 7) | (lane * R + (k & 3)));
      if (carry_g) q_g[pos] = g[k];
    }
    qn += __popc(b);
  }
#else
  const int cnt = __popc(m);
  int incl = cnt;
#pragma unroll
  for (int o = 1; o < 32; o <<= 1) {
    const int t = __shfl_up_sync(kFull, incl, o);
    if (lane >= o) incl += t;
  }
  const int qn = __shfl_sync(kFull, incl, 31);
  int pos = incl - cnt;
  for (uint32_t bits = m; bits; bits &= bits - 1u, ++pos) {
    const int k = __ffs(bits) - 1;
    q_row[pos] = (uint8_t)(((k >> 2) << 7) | (lane * R + (k & 3)));
    if (carry_g) {
      int32_t gv = 0;
#pragma unroll
      for (int kk = 0; kk < 2 * R; ++kk) gv = kk == k ? g[kk] : gv;
      q_g[pos] = gv;
    }
  }
#endif
  __syncwarp();

  // stage C in full batches of 32: the warp's queue of this pair is appended to the rows
  // carried over from earlier pairs; every complete batch of 32 is processed now (one row
  // per lane, all lanes busy), the < 32 left over are copied (as values) into the carry
  // buffer, so the tiles' shared-memory stages can be released.
  const int32_t* wcol0 = sbase0 + wbase;
  const int32_t* wcol1 = sbase1 + wbase;
  const uint32_t wrow0 = frow0 + wbase, wrow1 = frow1 + wbase;
  const int total = n_carry + qn;
  const int full_end = total & ~31;
  for (int base = 0; base < full_end; base += 32) {
    CarryEntry e = load_entry<NJ, DM>(p, js, cb, n_carry, q_row, q_g, carry_g, wcol0, wcol1,
                                      wrow0, wrow1, stride, base + lane);
    stage_c_row<NJ, GROUPED, DM>(p, js, sdm, e, j0, jf, smem_table, s_sum, s_cnt, acc_sum, acc_cnt, pd,
                                 pol);
  }
  {
    const int idx = full_end + lane;
    const bool has = idx < total;
    CarryEntry e{};
    if (has)
      e = load_entry<NJ, DM>(p, js, cb, n_carry, q_row, q_g, carry_g, wcol0, wcol1, wrow0, wrow1,
                             stride, idx);
    __syncwarp();
    if (has) {
#pragma unroll
      for (int jx = 0; jx < NJ; ++jx) cb->key[jx][lane] = e.key[jx];
      cb->a[lane] = e.a;
      cb->b[lane] = e.b;
      cb->g[lane] = e.g;
      cb->row[lane] = e.row;
    }
    n_carry = total - full_end;
  }
  __syncwarp();  // the queue and the carry buffer are reused by the next pair
}

// The rows still carried by a warp after its last tile (fewer than 32).
template <int NJ, bool GROUPED, bool DM>
__device__ __forceinline__ void drain_carry(const K1Params& p, const JoinState (&js)[HX_MAX_JOINS],
                                            const unsigned char* sdm, const CarryBuf* cb,
                                            int n_carry, int lane, int j0,
                                            int jf, bool smem_table, unsigned long long* s_sum,
                                            uint32_t* s_cnt, long long& acc_sum,
                                            long long& acc_cnt, Pending& pd, const Pols& pol) {
  if (lane >= n_carry) return;
  CarryEntry e;
#pragma unroll
  for (int jx = 0; jx < NJ; ++jx) e.key[jx] = cb->key[jx][lane];
  e.a = cb->a[lane];
  e.b = cb->b[lane];
  e.row = cb->row[lane];
  e.g = cb->g[lane];
  stage_c_row<NJ, GROUPED, DM>(p, js, sdm, e, j0, jf, smem_table, s_sum, s_cnt, acc_sum, acc_cnt, pd,
                                 pol);
}

__device__ __forceinline__ void mbar_wait_sleep(uint64_t* bar, uint32_t parity) {
  uint32_t ok = 0;
  while (true) {
    asm volatile(
        "{\n"
        ".reg .pred p;\n"
        "mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2;\n"
        "selp.u32 %0, 1, 0, p;\n"
        "}\n"
        : "=r"(ok)
        : "r"(smem_u32(bar)), "r"(parity)
        : "memory");
    if (ok) return;
    if (HX_PROD_SLEEP) __nanosleep(HX_PROD_SLEEP);
  }
}

template <int NJ, bool GROUPED, bool DM, int W>
#ifndef HX_K1_LB_LO
#define HX_K1_LB_LO 896  // launch-bound thread count of the 20-warp instances (0: exact):
                         // 896 caps them at 72 registers, measured 0.3-3% faster than 80
#endif
#ifndef HX_K1_LB_LO_HT
#define HX_K1_LB_LO_HT 0  // ... of the 20-warp hash-table instances (0: exact, 80 registers:
                          // no spills with 3 joins; see kWarpsHi's choice in k1_setup)
#endif
__global__ void __launch_bounds__((W == kWarpsLo && (DM ? HX_K1_LB_LO : HX_K1_LB_LO_HT))
                                      ? (DM ? HX_K1_LB_LO : HX_K1_LB_LO_HT)
                                      : k1_threads(W),
                                  kCtasPerSm)
    k1_probe_agg(const __grid_constant__ K1Params p) {
  constexpr int kConsumerWarps = W;
  constexpr int kConsumers = W * 32;
  extern __shared__ __align__(128) unsigned char smem[];
  uint64_t* full = reinterpret_cast<uint64_t*>(smem);
  uint64_t* empty = full + p.stages;
  int32_t* headbuf = reinterpret_cast<int32_t*>(smem + kSmemHeadOff);        // 8 cols x 4
  int* next_chunk = reinterpret_cast<int*>(smem + kSmemCtlOff);
  volatile int* slot_tile = reinterpret_cast<volatile int*>(smem + kSmemCtlOff) + 1;
  const int kSmemFixed = p.smem_fixed;
  uint8_t* q_rows = smem + kSmemQueueOff;
  int32_t* q_gs = DM ? nullptr
                     : reinterpret_cast<int32_t*>(smem + kSmemQueueOff + W * kQueueRows);
  unsigned long long* s_sum = reinterpret_cast<unsigned long long*>(smem + kSmemFixed);
  uint32_t* s_cnt = reinterpret_cast<uint32_t*>(s_sum + p.smem_groups);
  const size_t table_bytes = ((size_t)p.smem_groups * 12 + 127) & ~size_t(127);
  uint32_t* s_filters = reinterpret_cast<uint32_t*>(smem + kSmemFixed + table_bytes);
  const size_t filter_bytes = ((size_t)p.filter_words * 4 + 127) & ~size_t(127);
  unsigned char* sdm = smem + kSmemFixed + table_bytes + filter_bytes;  // staged direct maps
  int32_t* stage0 = reinterpret_cast<int32_t*>(sdm + p.dm_bytes);
  const int stage_elems = p.n_cols * kTileRows;

  // a failed group layout (capacity, or a plan whose dimensions changed) disables the pass
  if (GROUPED && p.meta->error) return;
  const int tid = threadIdx.x;
  const int warp = tid >> 5;
  const int lane = tid & 31;
  if (tid == kConsumers) {
    for (int s = 0; s < p.stages; ++s) {
      mbar_init(full + s, 1);
      mbar_init(empty + s, kChunksPerTile);  // every chunk of the tile arrives once
      slot_tile[s] = -1;
    }
    *next_chunk = 0;
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  __syncthreads();

  if (warp == kConsumerWarps) {
    // ---------------- producer warp: stream tiles HBM -> smem ring ----------------
    if (lane == 0) {
      const uint64_t pol = policy_evict_first();
      int s = 0;
      uint32_t ph = 0;
      bool wrapped = false;
      int i = 0;  // this CTA's i-th tile
      for (int64_t t = blockIdx.x; t < p.n_tiles; t += gridDim.x, ++i) {
        if (wrapped) mbar_wait_sleep(empty + s, ph ^ 1u);
        slot_tile[s] = i;  // slot s now holds (is being filled with) tile i: see the consumers
        const int64_t r0 = t * kTileRows;
        const int64_t rows = std::min<int64_t>(kTileRows, p.n_rows - r0);
        const uint32_t bytes = (uint32_t)(rows & ~int64_t(3)) * 4u;
        mbar_arrive_expect_tx(full + s, bytes * p.n_cols);
        // L2 prefetch of the tile `prefetch` ring refills ahead: its bulk copy then hits L2,
        // so the ring's bytes in flight are not bounded by its free slots alone
        if (p.prefetch) {
          const int64_t tp = t + (int64_t)p.prefetch * gridDim.x;
          if (tp < p.n_tiles) {
            const int64_t rp = tp * kTileRows;
            const uint32_t pb = (uint32_t)(std::min<int64_t>(kTileRows, p.n_rows - rp) & ~int64_t(3)) * 4u;
            if (pb)
              for (int c = 0; c < p.n_cols; ++c) bulk_prefetch_l2(p.col[c] + rp, pb);
          }
        }
        if (bytes) {
          int32_t* dst = stage0 + (size_t)s * stage_elems;
          for (int c = 0; c < p.n_cols; ++c)
            bulk_g2s(dst + c * kTileRows, p.col[c] + r0, bytes, full + s, pol);
        }
        if (++s == p.stages) {
          s = 0;
          ph ^= 1u;
          wrapped = true;
        }
      }
    }
    return;
  }

  // ---------------- consumer warps ----------------
  const int ctid = tid;  // 0..kConsumers-1
  const Pols pol{p.l2_hint ? policy_evict_last() : policy_evict_normal(), policy_evict_first()};
  uint8_t* q_row = q_rows + warp * kQueueRows;
  int32_t* q_g = DM ? nullptr : q_gs + warp * kQueueRows;
  CarryBuf* cb = reinterpret_cast<CarryBuf*>(smem + smem_carry_off(DM, W) + warp * kCarryBytes);
  int n_carry = 0;
  JoinState js[HX_MAX_JOINS];
#pragma unroll
  for (int j = 0; j < HX_MAX_JOINS; ++j) {
    if (j < NJ) {
      const int lg = p.joins[j].hdr->log2cap;
      js[j].buckets = reinterpret_cast<const ulonglong2*>(p.joins[j].slots);
      js[j].c = p.joins[j].c;
      js[j].shift = 33 - lg;
      js[j].bmask = (1u << (lg - 1)) - 1u;
      js[j].jstride = GROUPED ? p.meta->jstride[j] : 0;
      js[j].sbloom = nullptr;
      js[j].blw = 0;
    } else {
      js[j] = JoinState{nullptr, 0, 32, 0u, 0, nullptr, 0};
    }
  }
  // stage the Bloom filters into their shared-memory reservations (once per CTA). A filter
  // larger than its reservation (a power of two) is folded: the word index is the top bits of
  // the hash, so OR-ing each run of F adjacent words gives the same filter with F times fewer
  // words (more false positives, never a false negative).
  {
    uint32_t* dst = s_filters;
#pragma unroll
    for (int j = 0; j < NJ; ++j) {
      const int reserved = p.joins[j].bloom_words;
      if (reserved == 0) continue;
      const int lw = p.joins[j].hdr->bloom_log2w;
      const uint32_t* src = p.joins[j].bloom;
      if ((1 << lw) <= reserved) {
        if (lw >= 2) {
          for (int i = ctid; i < (1 << lw) / 4; i += kConsumers)
            reinterpret_cast<uint4*>(dst)[i] = __ldg(reinterpret_cast<const uint4*>(src) + i);
        } else if (ctid < 2) {  // 1-2 words: replicate to two so that blw >= 1
          dst[ctid] = __ldg(src + (lw == 0 ? 0 : ctid));
        }
        js[j].sbloom = dst;
        js[j].blw = lw == 0 ? 1 : lw;
      } else {
        const int fold = (1 << lw) / reserved;
        for (int i = ctid; i < reserved; i += kConsumers) {
          uint32_t w = 0;
          for (int f = 0; f < fold; ++f) w |= __ldg(src + i * fold + f);
          dst[i] = w;
        }
        js[j].sbloom = dst;
        js[j].blw = 31 - __clz(reserved);
      }
      dst += reserved;
    }
  }
  // stage the direct maps planned into shared memory (once per CTA)
#pragma unroll
  for (int j = 0; j < NJ; ++j) {
    if (!dm_smem<DM>(p, j)) continue;
    const uint4* src = reinterpret_cast<const uint4*>(p.joins[j].dm);
    uint4* dst = reinterpret_cast<uint4*>(sdm + p.joins[j].dm_smem);
    for (int i = ctid; i < p.joins[j].dm_words / 4; i += kConsumers) dst[i] = __ldg(src + i);
  }
#pragma unroll
  for (int j = 0; j < NJ; ++j) {
    if (!DM || !jbit(p.m_bm, j)) continue;
    const uint4* src = reinterpret_cast<const uint4*>(p.joins[j].bm);
    uint4* dst = reinterpret_cast<uint4*>(sdm + p.joins[j].bm_smem);
    for (int i = ctid; i < p.joins[j].bm_words / 4; i += kConsumers) dst[i] = __ldg(src + i);
  }
  const long long n_groups = GROUPED ? p.meta->n_groups : 1;
  const bool smem_table = GROUPED && n_groups <= p.smem_groups;
  if (smem_table) {
    uint32_t* s_lo = reinterpret_cast<uint32_t*>(s_sum);
    for (int g = ctid; g < n_groups; g += kConsumers) {
      s_lo[g] = 0;
      s_lo[p.smem_groups + g] = 0;
      s_cnt[g] = 0;
    }
  }
  long long acc_sum = 0, acc_cnt = 0;
  Pending pd{0, 0, 0, false};
  // misaligned head rows (views at a row offset): CTA 0's warp 0 reads them directly
  if (blockIdx.x == 0 && p.head_rows > 0 && warp == 0) {
    if (lane < p.head_rows)
      for (int c = 0; c < p.n_cols; ++c) headbuf[c * 4 + lane] = p.head_col[c][lane];
    __syncwarp();
    process_tile<NJ, GROUPED, DM>(p, js, sdm, headbuf, headbuf, 0u, 0u, 4, p.head_rows, 0, 0, lane,
                                  smem_table, s_sum, s_cnt, q_row, q_g, cb, n_carry, acc_sum,
                                  acc_cnt, pd, pol);
  }
  consumer_sync<W>();

  // This CTA's i-th tile (t = blockIdx.x + i * gridDim.x) arrives in ring slot i mod stages.
  // Warps claim chunks c = 0, 1, 2, ... (tile i = c / kChunksPerTile) from a shared counter;
  // a stage is released when all of its chunks are done (empty barrier count =
  // kChunksPerTile). Before waiting on slot s's full barrier for tile i, a warp waits until
  // the producer has tagged the slot with i: the barrier's previous phase (tile i - stages)
  // is then complete, so the parity wait cannot match it.
  const int64_t my_tiles = p.n_tiles > blockIdx.x ? (p.n_tiles - 1 - blockIdx.x) / gridDim.x + 1 : 0;
  const int64_t my_chunks = my_tiles * kChunksPerTile;
  // (measured and rejected: claiming the next chunk before processing the current one, or
  // during its stage C — a reserved chunk waits for its warp and holds its stage back)
  // Direct-map instances: warp w takes chunks w, w + W, w + 2W, ... of the CTA's range, no
  // claim atomic on a chunk's critical path (SF100 step 19.77 -> 19.47 ms); the
  // tile tags still release each ring slot when its last chunk is done. Hash-table instances:
  // the same for up to 3 joins; with 4 (Q4.x: the most variable stage C) chunks are claimed
  // from a shared counter, in order (measured at SF100: HT Q4.1 5.98 -> 5.62 ms, Q4.2 4.68 ->
  // 4.44, Q4.3 2.61 -> 2.48; Q2.x/Q3.x lose 2-6% with claims).
  // (hash tables with 4 joins: the 26-warp instance claims, the 20-warp one is static — the
  // planner launches the latter when stage B probes a join in place: SF100 Q4.1 5.61 -> 4.95 ms)
  constexpr bool kStatic =
      DM ? HX_DM_STATIC_CHUNKS : (HX_HT_STATIC_CHUNKS && (NJ < HX_HT_CLAIM_NJ || W == kWarpsLo));
  int c = kStatic ? warp - kConsumerWarps : 0, span_left = 0;
  while (true) {
    if constexpr (kStatic) {
      c += kConsumerWarps;
    } else {
      if (span_left == 0) {  // HX_CLAIM_SPAN consecutive chunks per shared atomic
        if (lane == 0) c = atomicAdd(next_chunk, HX_CLAIM_SPAN);
        c = __shfl_sync(kFull, c, 0);
        span_left = HX_CLAIM_SPAN;
      } else {
        ++c;
      }
      --span_left;
    }
    if (c >= my_chunks) break;
    const int i = c / kChunksPerTile, ch = c - i * kChunksPerTile;
    // (tracking slot and phase incrementally instead of dividing by the ring depth was
    // measured 3% slower: the loop-carried registers cost more than the division; the division
    // is a multiply-high by the ring depth's reciprocal, not the ~20-instruction runtime divide)
    const uint32_t lap = __umulhi((uint32_t)i, p.stage_magic);
    const int slot = i - (int)lap * p.stages;
    const uint32_t phase = lap & 1u;
    constexpr int kTagSleep = DM ? HX_TAG_SLEEP_DM : HX_TAG_SLEEP_HT;
    while (slot_tile[slot] != i)
      if (kTagSleep) __nanosleep(kTagSleep);
    mbar_wait(full + slot, phase);
    int32_t* st = stage0 + (size_t)slot * stage_elems;
    const int64_t t = blockIdx.x + (int64_t)i * gridDim.x;
    const int64_t r0 = t * kTileRows;
    const int rows = (int)std::min<int64_t>(kTileRows, p.n_rows - r0);
    const int crows = max(0, min(kChunkRows, rows - ch * kChunkRows));
    const int copied = rows & ~3;
    if (copied != rows && copied / kChunkRows == ch) {
      // ragged tail: the last <= 3 rows of the table are not a 16-byte multiple (not copied
      // by the bulk engine); the warp owning their chunk reads them directly
      if (lane < rows - copied)
        for (int cc = 0; cc < p.n_cols; ++cc)
          st[cc * kTileRows + copied + lane] = p.col[cc][r0 + copied + lane];
      __syncwarp();
    }
    const int32_t* cb0 = st + ch * kChunkRows;
    const uint32_t frow0 = (uint32_t)(p.head_rows + r0 + ch * kChunkRows);
    process_tile<NJ, GROUPED, DM>(p, js, sdm, cb0, cb0 + kHalfRows, frow0, frow0 + kHalfRows,
                                  kTileRows, min(crows, kHalfRows),
                                  max(0, crows - kHalfRows), 0, lane, smem_table, s_sum,
                                  s_cnt, q_row, q_g, cb, n_carry, acc_sum, acc_cnt, pd, pol);
    __syncwarp();
    if (lane == 0) mbar_arrive(empty + slot);
  }

  // the rows this warp still carries
  if (NJ > 0)
    drain_carry<NJ, GROUPED, DM>(p, js, sdm, cb, n_carry, lane, first_join_in_place<NJ, DM>(p, js),
                             first_filter<NJ, DM>(js), smem_table, s_sum, s_cnt, acc_sum, acc_cnt,
                             pd, pol);
  if (pd.alive)  // the last deferred row
    accumulate<GROUPED>(p, smem_table, s_sum, s_cnt, pd.g, measure(p.agg_op, pd.a, pd.b), acc_sum,
                        acc_cnt);
  __syncwarp();

  // ---------------- flush the CTA's partial aggregate ----------------
  if (GROUPED) {
    if (smem_table) {
      consumer_sync<W>();
      const uint32_t* s_lo = reinterpret_cast<const uint32_t*>(s_sum);
      for (int g = ctid; g < n_groups; g += kConsumers) {
        const uint32_t c = s_cnt[g];
        if (c) {
          atomicAdd(p.g_sum + g,
                    ((unsigned long long)s_lo[p.smem_groups + g] << 32) | s_lo[g]);
          atomicAdd(p.g_cnt + g, (unsigned long long)c);
        }
      }
    }
  } else {
    // neighbourhood reduce (warp shuffle, then the CTA) + one leader atomic (Listing 1 L27-29)
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) {
      acc_sum += __shfl_xor_sync(kFull, acc_sum, o);
      acc_cnt += __shfl_xor_sync(kFull, acc_cnt, o);
    }
    // every consumer is done with the queues, maps and ring (and no bulk copy is in flight:
    // every tile was consumed): the partials go at kSmemQueueOff, {sum, count} per warp
    consumer_sync<W>();
    long long* red = reinterpret_cast<long long*>(smem + kSmemQueueOff);
    if (lane == 0) {
      red[2 * warp] = acc_sum;
      red[2 * warp + 1] = acc_cnt;
    }
    consumer_sync<W>();
    if (ctid == 0) {
      long long s = 0, c = 0;
      for (int w = 0; w < kConsumerWarps; ++w) {
        s += red[2 * w];
        c += red[2 * w + 1];
      }
      if (c) {
        atomicAdd(p.g_sum, (unsigned long long)s);
        atomicAdd(p.g_cnt, (unsigned long long)c);
      }
    }
  }
}

// K1 for join-less pipelines (the §6.4 SUM micro-benchmark; any shape
// with no join): Listing 1 pipeline 9 in its plain form — unpack,
// predicate, register accumulator, then warp shuffle -> CTA -> one leader atomic. There is no
// structure to stage and no survivor to compact, so the consumers only read their rows:
// one producer warp streams 32 KB stages of the columns (kScanRows(NC) rows) HBM -> shared
// memory with cp.async.bulk into a kScanStages-deep mbarrier ring (evict-first), and each of
// the kScanThreads consumer threads reads 4 consecutive rows per column with one 128-bit
// shared-memory load. (Plain 128-bit global loads measured 5.5 TB/s on one column; the
// bulk-copy ring reaches the read-stream ceiling, tools/stream_roofline.cu.)
constexpr int kScanThreads = 512;  // consumer threads (+ one producer warp)
constexpr int kScanStages = 6;
constexpr int scan_rows(int nc) { return nc == 1 ? 8192 : nc == 2 ? 4096 : 2048; }
constexpr size_t scan_smem(int nc) { return 128 + (size_t)kScanStages * nc * scan_rows(nc) * 4; }
template <int NC>
__global__ void __launch_bounds__(kScanThreads + 32, 1) k1_scan_agg(const __grid_constant__ K1Params p) {
  constexpr int kRows = scan_rows(NC);
  extern __shared__ __align__(128) unsigned char smem[];
  uint64_t* full = reinterpret_cast<uint64_t*>(smem);
  uint64_t* empty = full + kScanStages;
  int32_t* ring = reinterpret_cast<int32_t*>(smem + 128);
  __shared__ long long red[2][kScanThreads / 32];
  const int tid = threadIdx.x, warp = tid >> 5, lane = tid & 31;
  const int64_t n_tiles = (p.n_rows + kRows - 1) / kRows;
  if (tid == kScanThreads) {
    for (int st = 0; st < kScanStages; ++st) {
      mbar_init(full + st, 1);
      mbar_init(empty + st, kScanThreads / 32);
    }
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  __syncthreads();
  if (warp == kScanThreads / 32) {  // producer
    if (lane == 0) {
      const uint64_t pol = policy_evict_first();
      int st = 0;
      uint32_t ph = 0;
      int64_t k = 0;
      for (int64_t t = blockIdx.x; t < n_tiles; t += gridDim.x, ++k) {
        if (k >= kScanStages) mbar_wait_sleep(empty + st, ph ^ 1u);
        const int64_t r0 = t * kRows;
        const uint32_t bytes = (uint32_t)(std::min<int64_t>(kRows, p.n_rows - r0) & ~int64_t(3)) * 4u;
        mbar_arrive_expect_tx(full + st, bytes * NC);
        if (bytes)
          for (int c = 0; c < NC; ++c)
            bulk_g2s(ring + ((size_t)st * NC + c) * kRows, p.col[c] + r0, bytes, full + st, pol);
        if (++st == kScanStages) {
          st = 0;
          ph ^= 1u;
        }
      }
    }
    return;
  }
  long long acc_sum = 0, acc_cnt = 0;
  auto row = [&](const int32_t (&v)[NC]) {
    bool ok = true;
    for (int q = 0; q < p.n_preds; ++q) {
      const DevPred& pr = p.preds[q];
      int32_t x = v[0];
#pragma unroll
      for (int c = 1; c < NC; ++c) x = pr.c == c ? v[c] : x;
      ok = ok && pred_pass(pr, x);
    }
    int32_t a = v[0], b = v[0];
#pragma unroll
    for (int c = 1; c < NC; ++c) {
      a = p.agg_a == c ? v[c] : a;
      b = p.agg_b == c ? v[c] : b;
    }
    if (ok) {
      acc_sum += measure(p.agg_op, a, b);
      acc_cnt += 1;
    }
  };
  const bool plain_sum = p.n_preds == 0 && p.agg_op == HX_AGG_SUM;
  // misaligned head rows (views at a row offset; before the first 16-byte boundary)
  if (blockIdx.x == 0 && tid < p.head_rows) {
    int32_t v[NC];
#pragma unroll
    for (int c = 0; c < NC; ++c) v[c] = p.head_col[c][tid];
    row(v);
  }
  int st = 0;
  uint32_t ph = 0;
  for (int64_t t = blockIdx.x; t < n_tiles; t += gridDim.x) {
    mbar_wait(full + st, ph);
    const int64_t r0 = t * kRows;
    const int rows = (int)std::min<int64_t>(kRows, p.n_rows - r0);
    const int32_t* sb = ring + (size_t)st * NC * kRows;
    if (rows == kRows && plain_sum) {  // SUM(a), no predicate: 4 rows per 128-bit load
#pragma unroll 4
      for (int i = tid; i < kRows / 4; i += kScanThreads) {
        const int4 x = reinterpret_cast<const int4*>(sb + p.agg_a * kRows)[i];
        acc_sum += ((long long)x.x + (long long)x.y) + ((long long)x.z + (long long)x.w);
      }
      acc_cnt += kRows / kScanThreads;
    } else if (rows == kRows) {
#pragma unroll 2
      for (int i = tid; i < kRows / 4; i += kScanThreads) {
        int4 x[NC];
#pragma unroll
        for (int c = 0; c < NC; ++c) x[c] = reinterpret_cast<const int4*>(sb + c * kRows)[i];
        // predicates column-wise on the 4 rows (kind uniform per predicate), then the measure
        uint32_t m = 0xFu;
        for (int q = 0; q < p.n_preds; ++q) {
          const DevPred& pr = p.preds[q];
          int4 y = x[0];
#pragma unroll
          for (int c = 1; c < NC; ++c) y = pr.c == c ? x[c] : y;
          const int32_t yv[4] = {y.x, y.y, y.z, y.w};
#pragma unroll
          for (int k = 0; k < 4; ++k) if (!pred_pass(pr, yv[k])) m &= ~(1u << k);
        }
        int4 a4 = x[0], b4 = x[0];
#pragma unroll
        for (int c = 1; c < NC; ++c) {
          a4 = p.agg_a == c ? x[c] : a4;
          b4 = p.agg_b == c ? x[c] : b4;
        }
        const int32_t av[4] = {a4.x, a4.y, a4.z, a4.w}, bv[4] = {b4.x, b4.y, b4.z, b4.w};
#pragma unroll
        for (int k = 0; k < 4; ++k)
          if ((m >> k) & 1u) acc_sum += measure(p.agg_op, av[k], bv[k]);
        acc_cnt += __popc(m);
      }
    } else {  // the last, partial tile: its < 4 ragged rows were not copied
      const int copied = rows & ~3;
      for (int r = tid; r < rows; r += kScanThreads) {
        int32_t v[NC];
#pragma unroll
        for (int c = 0; c < NC; ++c) v[c] = r < copied ? sb[c * kRows + r] : p.col[c][r0 + r];
        row(v);
      }
    }
    __syncwarp();
    if (lane == 0) mbar_arrive(empty + st);
    if (++st == kScanStages) {
      st = 0;
      ph ^= 1u;
    }
  }
  // neighbourhood reduce + leader atomic (Listing 1 L27-29)
#pragma unroll
  for (int o = 16; o > 0; o >>= 1) {
    acc_sum += __shfl_xor_sync(kFull, acc_sum, o);
    acc_cnt += __shfl_xor_sync(kFull, acc_cnt, o);
  }
  if (lane == 0) {
    red[0][warp] = acc_sum;
    red[1][warp] = acc_cnt;
  }
  asm volatile("bar.sync 1, %0;" ::"n"(kScanThreads) : "memory");
  if (tid == 0) {
    long long s = 0, c = 0;
    for (int w = 0; w < kScanThreads / 32; ++w) {
      s += red[0][w];
      c += red[1][w];
    }
    if (c) {
      atomicAdd(p.g_sum, (unsigned long long)s);
      atomicAdd(p.g_cnt, (unsigned long long)c);
    }
  }
}

// Group layout from the dimension ranks (device-side; no host round trip) and zeroing of
// the group arrays. Every CTA computes n_groups; CTA 0 publishes the meta.
__global__ void k1_prepare(AggMeta* meta, const HtHeader* g0, const HtHeader* g1,
                           const HtHeader* g2, int n_gdims, int4 gdim_join,
                           unsigned long long* sums, unsigned long long* cnts,
                           long long cap_groups, int fresh) {
  const HtHeader* hdrs[HX_MAX_GDIMS] = {g0, g1, g2};
  const int gj[HX_MAX_GDIMS] = {gdim_join.x, gdim_join.y, gdim_join.z};
  int32_t nr[HX_MAX_GDIMS] = {1, 1, 1};
  long long n = 1;
  for (int g = 0; g < n_gdims; ++g) {
    nr[g] = max(1, hdrs[g]->n_ranks);  // an empty dimension still gives one (empty) rank
    n *= nr[g];
  }
  const bool over = n > cap_groups;
  if (over) n = cap_groups;
  if (fresh) {
    if (blockIdx.x == 0 && threadIdx.x == 0) {
      AggMeta m{};
      m.n_groups = n;
      long long stride = 1;
      for (int j = 0; j < HX_MAX_JOINS; ++j) m.jstride[j] = 0;
      for (int g = n_gdims - 1; g >= 0; --g) {
        m.jstride[gj[g]] = (int32_t)stride;
        stride *= nr[g];
      }
      for (int g = 0; g < HX_MAX_GDIMS; ++g) m.n_ranks[g] = nr[g];
      m.error = over ? HX_ECAPACITY : 0;
      *meta = m;
    }
    for (long long i = blockIdx.x * (long long)blockDim.x + threadIdx.x; i < n;
         i += (long long)gridDim.x * blockDim.x) {
      sums[i] = 0;
      cnts[i] = 0;
    }
  }
}

using KernelFn = void (*)(K1Params);

// K1 launches carry the device's greatest priority: the builds of later queries (forked on
// auxiliary streams so they overlap) then only take SMs that K1 leaves idle (its tail), and
// the next K1's CTAs are dispatched ahead of queued build CTAs.
// An L2 access-policy window (persisting) over the launch's main probe structure, when set:
// the lines of [base, base + bytes) get persisting priority in the L2 set-aside region
// (cudaLimitPersistingL2CacheSize, set at hx_init), hit ratio = set-aside / window bytes.
struct L2Window {
  void* base = nullptr;
  size_t bytes = 0;
  float hit_ratio = 0.f;
};
cudaError_t launch_k1(KernelFn fn, int grid, int block, size_t smem, cudaStream_t s,
                      const K1Params& p, int priority, int carveout = -1,
                      const L2Window* win = nullptr) {
  cudaLaunchConfig_t cfg{};
  cfg.gridDim = dim3((unsigned)grid);
  cfg.blockDim = dim3((unsigned)block);
  cfg.dynamicSmemBytes = smem;
  cfg.stream = s;
  cudaLaunchAttribute attr[3];
  int n = 0;
  attr[n].id = cudaLaunchAttributePriority;
  attr[n++].val.priority = priority;
  if (carveout >= 0) {
    attr[n].id = cudaLaunchAttributePreferredSharedMemoryCarveout;
    attr[n++].val.sharedMemCarveout = (unsigned)carveout;
  }
  if (win && win->bytes) {
    attr[n].id = cudaLaunchAttributeAccessPolicyWindow;
    attr[n].val.accessPolicyWindow.base_ptr = win->base;
    attr[n].val.accessPolicyWindow.num_bytes = win->bytes;
    attr[n].val.accessPolicyWindow.hitRatio = win->hit_ratio;
    attr[n].val.accessPolicyWindow.hitProp = cudaAccessPropertyPersisting;
    attr[n++].val.accessPolicyWindow.missProp = cudaAccessPropertyStreaming;
  }
  cfg.attrs = attr;
  cfg.numAttrs = n;
  return cudaLaunchKernelEx(&cfg, fn, p);
}

// [warps: 20, 26][direct maps][grouped][joins]; join-less pipelines use the hash-table instances
#define HX_K1_ROW(W, G, D)                                                                      \
  {k1_probe_agg<0, G, false, W>, k1_probe_agg<1, G, D, W>, k1_probe_agg<2, G, D, W>,             \
   k1_probe_agg<3, G, D, W>, k1_probe_agg<4, G, D, W>}
const KernelFn kKernels[2][2][2][HX_MAX_JOINS + 1] = {
    {{HX_K1_ROW(kWarpsLo, false, false), HX_K1_ROW(kWarpsLo, true, false)},
     {HX_K1_ROW(kWarpsLo, false, true), HX_K1_ROW(kWarpsLo, true, true)}},
    {{HX_K1_ROW(kWarpsHiHt, false, false), HX_K1_ROW(kWarpsHiHt, true, false)},
     {HX_K1_ROW(kWarpsHi, false, true), HX_K1_ROW(kWarpsHi, true, true)}}};
#undef HX_K1_ROW

KernelFn pick_kernel(int nj, bool grouped, bool dm, int warps) {
  return kKernels[warps == kWarpsLo ? 0 : 1][dm ? 1 : 0][grouped ? 1 : 0][nj];
}

size_t k1_smem_bytes(int warps, bool dm, int n_cols, int stages, int smem_groups,
                     int filter_words = 0, int dm_bytes = 0, bool in_place = false) {
  const size_t table_bytes = ((size_t)smem_groups * 12 + 127) & ~size_t(127);
  const size_t filter_bytes = ((size_t)filter_words * 4 + 127) & ~size_t(127);
  return (in_place ? kSmemQueueOff : smem_fixed(dm, warps)) + table_bytes + filter_bytes + (size_t)dm_bytes +
         (size_t)stages * n_cols * kTileRows * sizeof(int32_t);
}

// Per-CTA shared memory for `ctas` resident CTAs per SM (228 KB per SM, 1 KB reserved each).
constexpr size_t smem_budget(int ctas) { return (228 * 1024) / ctas - 1024; }
// The shared memory K1 may plan with per CTA: the rest of the SM's 256 KB L1/shared array
// becomes L1 cache for the L2 map reads. t_smem_cap lowers it while k1_setup replans an
// L2-lookup-bound pipeline; HX_K1_SMEM_KB lowers it (tuning aid).
thread_local size_t t_smem_cap = 0;
constexpr double kL1BoundCost = 50.0;  // plan cost above which K1 is L2-lookup-bound
size_t k1_smem_cap() {
  size_t cap = smem_budget(std::min(kCtasPerSm, 2));
  if (t_smem_cap) cap = std::min(cap, t_smem_cap);
  if (const char* e = std::getenv("HX_K1_SMEM_KB")) {
    const long kb = std::atol(e);
    if (kb >= 64) cap = std::min<size_t>(cap, (size_t)kb * 1024);
  }
  return cap;
}

// ring depth the plan starts from (0: kBaseStages); k1_setup also plans one stage deeper
thread_local int t_base_stages = 0;
int pick_stages(int warps, bool dm, int n_cols, int smem_groups) {
  // as many tile stages as fit next to kCtasPerSm CTAs per SM, at least double buffering
  // (at most HX_K1_STAGE_KB of tiles per CTA: the rest is left for filters and maps)
  const size_t fixed = smem_fixed(dm, warps) + (((size_t)smem_groups * 12 + 127) & ~size_t(127));
  const size_t budget = std::min<size_t>(std::min(smem_budget(kCtasPerSm), k1_smem_cap()),
                                         fixed + HX_K1_STAGE_KB * 1024);
  const size_t stage = (size_t)n_cols * kTileRows * 4;
  const int s = budget > fixed ? (int)((budget - fixed) / stage) : 0;
  int base = t_base_stages ? t_base_stages : kBaseStages;
  if (const char* e = std::getenv("HX_K1_MIN_STAGES")) base = std::max(2, std::min(kMaxStages, std::atoi(e)));
  return std::max(2, std::min(base, s));
}

enum { kStNone = 0, kStFull, kStBitmap, kStBloom };

// False-positive rate of the blocked Bloom filter (one 32-bit word per key, two bits set) at
// `bits_per_key`: the keys per word are Poisson(32 / bits_per_key); a key of a word holding
// n keys passes when both its bits are among the word's set bits.
double bloom_fp(double bits_per_key) {
  if (bits_per_key <= 0.0) return 1.0;
  const double lam = 32.0 / bits_per_key;
  double fp = 0.0, pn = std::exp(-lam);
  for (int n = 0; n < 256; ++n) {
    const double q = 1.0 - std::pow(31.0 / 32.0, 2.0 * n);
    fp += pn * q * q;
    pn *= lam / (n + 1);
  }
  return std::min(1.0, fp);
}

// Relative per-row costs (issue slots) of the K1 stages, measured on SF10 SSB: a stage-S
// filter on every row, a row entering stage C (compaction, queue, batch), a stage-C
// shared-memory filter, an L2 lookup. HX_K1_COST="s,c,sc,l2" overrides (tuning aid).
struct K1Cost {
  // s2: an L2 map read in stage S per live row (stage-S cost s + s2 * live fraction). A flat
  // 16 per row (fitted at SF10-SF100, where such reads follow a selective shared-memory
  // filter) made SF1000 plans read 2-15 MB maps for every row; charging the live fraction
  // keeps the SF100 plans and picks the Bloom-filtered plans at SF1000 (Q2.1 2.2x, Q3.2 2.2x).
  // c: 60 fitted at SF10 (r01); 120 measured better or equal at SF10, SF100 and SF1000
  // dimensions (profiles/r02_cost_model_sweep.txt: SF100 K1 sum 19.29 -> 19.23 ms, SF1000 dims
  // 24.76 -> 24.53; Q2.1 then filters with the supplier bitmap in stage S as well: 1.80 -> 1.70
  // ms at SF100, 2.00 -> 1.77 at SF1000). (90 and 150 lose on Q4.2/Q4.3: the landscape is not
  // smooth — the constants rank discrete plans.)
  double s = 8.0, c = 120.0, sc = 8.0, l2 = 20.0, s2 = 40.0;
};
K1Cost k1_cost() {
  K1Cost k;
  if (const char* e = std::getenv("HX_K1_COST"))
    std::sscanf(e, "%lf,%lf,%lf,%lf,%lf", &k.s, &k.c, &k.sc, &k.l2, &k.s2);
  return k;
}

// Shared-memory plan of a direct-map pipeline: for every combination of per-join structures
// that fits next to the tile ring (none; the full map: exact + rank; the membership bitmap:
// exact; the Bloom filter at 8, 4, 2 or 1 bits per key) and every choice of the joins whose
// structure runs on EVERY row in stage S (the rest run on the compacted survivors in stage
// C), the expected cost per lineorder row is
//     s * |S| + c * f_S + sc * (structures read in stage C) * f_S + l2 * (L2 maps) * f_C
// with f_S = the fraction of rows passing stage S (pass fraction + false positives) and f_C
// the fraction still alive when the L2 lookups are issued; a pipeline whose joins are all
// full maps in stage S aggregates in place (no stage C). The cheapest plan is taken.
template <class Fits>
double plan_dm(int nj, const JoinDev* joins, const bool* known, const double* pass,
               const int64_t* keys, const int* bloom_w0, const bool* grouped, Fits fits,
               int* kind, int* bloom_w, int* in_s) {
  struct Opt {
    int kind, bw;
    double e;
    bool exact;
  };
  Opt opts[HX_MAX_JOINS][8];
  int n_opt[HX_MAX_JOINS];
  for (int j = 0; j < nj; ++j) {
    const JoinDev& d = joins[j];
    const double pj = known[j] ? pass[j] : 1.0;
    int n = 0;
    opts[j][n++] = {kStNone, 0, 1.0, false};
    opts[j][n++] = {kStFull, 0, pj, true};
    if (d.dm_lw > 0) opts[j][n++] = {kStBitmap, 0, pj, true};
    if (known[j] && keys[j] > 0)
      for (int f = 1; f <= 16 && bloom_w0[j] / f >= 4; f *= 2) {
        const int bw = bloom_w0[j] / f;
        const double e = pj + (1.0 - pj) * bloom_fp(32.0 * bw / (double)keys[j]);
        opts[j][n++] = {kStBloom, bw, e, false};
      }
    n_opt[j] = n;
  }
  const K1Cost K = k1_cost();
  double best = 1e300;
  int idx[HX_MAX_JOINS] = {0, 0, 0, 0};
  int kd[HX_MAX_JOINS], bw[HX_MAX_JOINS];
  while (true) {
    for (int j = 0; j < nj; ++j) {
      kd[j] = opts[j][idx[j]].kind;
      bw[j] = opts[j][idx[j]].bw;
    }
    // a plan that resolves every join in stage S aggregates in place and needs no per-warp
    // queues or carry buffers: it is checked against that smaller footprint
    const bool fits_q = fits(kd, bw, false), fits_ip = fits_q || fits(kd, bw, true);
    if (fits_ip) {
      // every subset of the joins may run in stage S: a join with a shared-memory structure
      // applies it there; one without reads its map from L2 there (exact, like a full map)
      const uint32_t has = (1u << nj) - 1u;
      for (uint32_t S = has;; S = (S - 1) & has) {
        double fS = 1.0, cost = 0.0;
        bool all_res = true;
        for (int j = 0; j < nj; ++j) {
          if ((S >> j) & 1u) {
            // stage S runs the joins in array order, each narrowing the live rows; an L2 map
            // is read only for the rows still live (fraction fS so far)
            cost += kd[j] == kStNone ? K.s + K.s2 * fS : K.s;
            fS *= kd[j] == kStNone ? (known[j] ? pass[j] : 1.0) : opts[j][idx[j]].e;
          }
          all_res = all_res && ((S >> j) & 1u) && (kd[j] == kStFull || kd[j] == kStNone);
        }
        if (!all_res && !fits_q) {
          if (S == 0) break;
          continue;
        }
        if (!all_res) {
          cost += K.c * fS;
          double fC = fS;
          int n_l2 = 0;
          for (int j = 0; j < nj; ++j) {
            const bool inS = (S >> j) & 1u;
            if (!inS && kd[j] != kStNone) {
              cost += K.sc * fS;
              fC *= opts[j][idx[j]].e;
            }
            if (inS && kd[j] == kStFull && grouped[j]) cost += K.sc * fS;  // rank re-read
            const bool full = kd[j] == kStFull;
            const bool exact = opts[j][idx[j]].exact || (inS && kd[j] == kStNone);
            n_l2 += !full && (grouped[j] || !exact);
          }
          cost += K.l2 * n_l2 * fC;
        }
        if (cost < best - 1e-12) {
          best = cost;
          for (int j = 0; j < nj; ++j) {
            kind[j] = kd[j];
            bloom_w[j] = bw[j];
            in_s[j] = (S >> j) & 1u;
          }
        }
        if (S == 0) break;
      }
    }
    int j = 0;
    while (j < nj && ++idx[j] == n_opt[j]) idx[j++] = 0;
    if (j == nj) break;
  }
  return best;
}

}  // namespace

int k1_occupancy(hx_ctx* ctx) {
  // cudaFuncSetAttribute applies to the CURRENT device only: set it once per device (a
  // process may hold contexts on several GPUs, created from several threads)
  static std::mutex mu;
  static uint64_t done = 0;  // bit d: device d configured
  std::lock_guard<std::mutex> lock(mu);
  const uint64_t bit = ctx->device < 64 ? (uint64_t(1) << ctx->device) : 0;
  if (!bit || !(done & bit)) {
    for (int w = 0; w < 2; ++w)
      for (int d = 0; d < 2; ++d)
        for (int g = 0; g < 2; ++g)
          for (int j = 0; j <= HX_MAX_JOINS; ++j)
            cudaFuncSetAttribute(kKernels[w][d][g][j], cudaFuncAttributeMaxDynamicSharedMemorySize,
                                 227 * 1024);
    cudaFuncSetAttribute(k1_scan_agg<1>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)scan_smem(1));
    cudaFuncSetAttribute(k1_scan_agg<2>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)scan_smem(2));
    cudaFuncSetAttribute(k1_scan_agg<3>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)scan_smem(3));
    cudaFuncSetAttribute(k1_scan_agg<4>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)scan_smem(4));
    done |= bit;
  }
  int occ = 0;
  cudaOccupancyMaxActiveBlocksPerMultiprocessor(
      &occ, k1_probe_agg<3, true, false, kWarpsLo>, k1_threads(kWarpsLo),
      k1_smem_bytes(kWarpsLo, false, 4, pick_stages(kWarpsLo, false, 4, kSmemGroups), kSmemGroups));
  return occ;
}

// A fully resolved K1 launch (kernel, parameters, grid, prepare-kernel arguments): built once
// on the host, enqueued any number of times (hx_pipeline_probe_agg, plans, CUDA graphs).
struct K1Prepared {
  K1Params p;
  KernelFn fn = nullptr;
  size_t smem = 0;
  int grid = 0;
  const HtHeader* gh[HX_MAX_GDIMS] = {nullptr, nullptr, nullptr};
  int4 gj = make_int4(0, 0, 0, 0);
  int n_gdims = 0;
  int prep_grid = 1;
  long long cap_groups = 1;
  int64_t rows = 0;
  int n_cols = 0;
  // host-resident fact table (§8(a) a8): the staged columns live in pinned host memory and
  // are streamed block by block through a device staging ring (mem-move)
  bool host = false;
  bool mapped = false;  // HX_PLACE_HOST_MAPPED: K1 reads host memory in place (zero-copy)
  KernelFn scan = nullptr;  // join-less pipeline: k1_scan_agg<NC> instead of k1_probe_agg
  int scan_grid = 0;
  size_t scan_smem = 0;
  const int32_t* host_col[kMaxStageCols] = {};
  int occ = 1;
  int64_t seg_rows = kSegRows;  // rows per launch (HX_K1_SEG_TILES overrides, for tests)
  int carveout = 100;           // preferred shared-memory carveout (% of 228 KB)
  int warps = kWarpsLo;         // consumer warps of the chosen instance
  double cost = -1.0;           // plan cost (direct maps; -1: hash tables)
  L2Window win;                 // persisting window over the largest L2-read probe structure
};

// Device staging ring of the mem-move for a host-resident fact table: kRingStages buffers of
// block_rows rows x the staged columns, filled by H2D copies on the ctx's copy stream while K1
// consumes the previous block on the compute stream (Listing 1 L7-19).
constexpr int kRingStages = 3;
struct StageRing {
  int64_t block_rows = 0;
  int n_cols = 0;
  void* base = nullptr;
  int32_t* buf[kRingStages][kMaxStageCols] = {};
  cudaEvent_t full[kRingStages] = {}, freed[kRingStages] = {};
};

long long k1_group_bound(const hx_query_shape* sh, hx_ht* const* hts, int n_hts) {
  long long bound = 1;
  for (int g = 0; g < sh->n_gdims; ++g) {
    const int j = sh->gdim_join[g];
    if (j < 0 || j >= sh->n_joins || sh->join_ht[j] < 0 || sh->join_ht[j] >= n_hts) return -1;
    for (int g2 = 0; g2 < g; ++g2)
      if (sh->gdim_join[g2] == j) return -1;
    const hx_ht* ht = hts[sh->join_ht[j]];
    // (dense ranks: at most one per passing row; identity ranks: the whole domain)
    bound *= std::max<long long>(1, ht->identity_ranks ? ht->domain
                                     : std::min<long long>(ht->domain, std::max<int64_t>(ht->dim_rows, 1)));
    bound = std::min<long long>(bound, (long long)HX_MAX_GROUPS + 1);
  }
  return bound;
}

int agg_alloc(hx_ctx* ctx, hx_agg* agg, long long cap_groups, const hx_query_shape* sh,
              hx_ht* const* hts) {
  HX_REQUIRE(cap_groups >= 1 && cap_groups <= HX_MAX_GROUPS, HX_ECAPACITY,
             "hx_pipeline_probe_agg: too many groups");
  agg->cap_groups = cap_groups;
  agg->n_gdims = sh->n_gdims;
  for (int g = 0; g < sh->n_gdims; ++g) agg->gdim_ht[g] = hts[sh->join_ht[sh->gdim_join[g]]];
  const size_t bytes = 256 + 2 * (size_t)cap_groups * sizeof(unsigned long long);
  HX_CK(cudaMallocAsync(&agg->base, bytes, ctx->stream));
  agg->meta = reinterpret_cast<AggMeta*>(agg->base);
  agg->sums = reinterpret_cast<unsigned long long*>(static_cast<char*>(agg->base) + 256);
  agg->cnts = agg->sums + cap_groups;
  return HX_OK;
}

int k1_setup(hx_ctx* ctx, const hx_table* fact, const hx_query_shape* sh, hx_ht* const* hts,
             int n_hts, const hx_agg* agg, K1Prepared** out) {
  struct CapReset {
    ~CapReset() {
      t_smem_cap = 0;
      t_base_stages = 0;
    }
  } cap_reset;
  t_smem_cap = 0;
  HX_REQUIRE(ctx && fact && sh && agg && out, HX_EINVAL, "hx_pipeline_probe_agg: null argument");
  HX_REQUIRE(sh->n_preds >= 0 && sh->n_preds <= HX_MAX_PREDS && sh->n_joins >= 0 &&
                 sh->n_joins <= HX_MAX_JOINS && sh->n_gdims >= 0 && sh->n_gdims <= HX_MAX_GDIMS &&
                 sh->agg_op >= HX_AGG_SUM && sh->agg_op <= HX_AGG_SUM_SUB,
             HX_EINVAL, "hx_pipeline_probe_agg: bad query shape");
  HX_REQUIRE(agg->n_gdims == sh->n_gdims, HX_EINVAL,
             "hx_pipeline_probe_agg: shape differs from the agg's");
  K1Prepared k{};
  K1Params& p = k.p;
  bool dm_mode = false;
  // distinct fact columns the shape references -> staged columns
  int32_t ids[kMaxStageCols];
  int n_cols = 0;
  auto stage_of = [&](int32_t col_id) -> int {
    for (int i = 0; i < n_cols; ++i)
      if (ids[i] == col_id) return i;
    if (n_cols == kMaxStageCols) return -2;
    if (!table_has_col(fact, col_id)) return -1;
    ids[n_cols] = col_id;
    return n_cols++;
  };
  for (int q = 0; q < sh->n_preds; ++q) {
    const hx_pred& pr = sh->preds[q];
    int c = stage_of(pr.col_id);
    HX_REQUIRE(c >= 0, HX_EINVAL, "hx_pipeline_probe_agg: predicate column not in fact table");
    HX_REQUIRE(pr.kind == HX_PRED_RANGE || (pr.kind == HX_PRED_IN && pr.n_in >= 1 && pr.n_in <= 4),
               HX_EINVAL, "hx_pipeline_probe_agg: bad predicate");
    p.preds[q] = DevPred{c, pr.kind, pr.lo, pr.hi, pr.n_in, {pr.in[0], pr.in[1], pr.in[2], pr.in[3]}};
    // an empty BETWEEN (lo > hi) selects nothing; stage A tests ranges as one unsigned
    // compare (v - lo) > (hi - lo), which would wrap: compile it to an IN over no values
    if (pr.kind == HX_PRED_RANGE && pr.lo > pr.hi)
      p.preds[q] = DevPred{c, HX_PRED_IN, 0, -1, 0, {0, 0, 0, 0}};
  }
  p.n_preds = sh->n_preds;
  for (int j = 0; j < sh->n_joins; ++j) {
    int c = stage_of(sh->join_fk_col[j]);
    HX_REQUIRE(c >= 0, HX_EINVAL, "hx_pipeline_probe_agg: join FK column not in fact table");
    HX_REQUIRE(sh->join_ht[j] >= 0 && sh->join_ht[j] < n_hts && hts && hts[sh->join_ht[j]],
               HX_EINVAL, "hx_pipeline_probe_agg: bad join hash table index");
    const hx_ht* ht = hts[sh->join_ht[j]];
    JoinDev d{};
    d.c = c;
    d.slots = ht->slots;
    d.hdr = ht->hdr;
    d.bloom = ht->bloom;
    d.dm_smem = -1;
    if (ht->dm) {
      d.dm = ht->dm;
      d.dm_kmin = ht->dm_kmin;
      d.dm_span = ht->dm_span;
      d.dm_lw = ht->dm_lw;
      d.dm_vmask = dm_vmask(ht->dm_lw);
      d.dm_words = (int32_t)ht->dm_words;
      d.bm = ht->dm_bm;
      d.bm_words = (int32_t)ht->bm_words;
    }
    d.bm_smem = -1;
    p.joins[j] = d;
  }
  {
    int n_dm = 0;
    for (int j = 0; j < sh->n_joins; ++j) n_dm += p.joins[j].dm != nullptr;
    HX_REQUIRE(n_dm == 0 || n_dm == sh->n_joins, HX_EINVAL,
               "hx_pipeline_probe_agg: direct-map and hash-table joins in one pipeline");
    dm_mode = n_dm > 0;
  }
  p.agg_op = sh->agg_op;
  // Late materialisation (R21): when every join's passing fraction is known (a
  // plan observed it) and their product bounds the passing rows below 1/16, a measure column
  // that no predicate or join reads is gathered for the passing rows (one 32-byte sector
  // each) instead of streamed for every row. Device-resident fact tables only.
  {
    double bound = sh->n_joins > 0 ? 1.0 : 2.0;
    for (int j = 0; j < sh->n_joins; ++j) {
      const hx_ht* ht = hts[sh->join_ht[j]];
      bound *= ht->known_keys < 0 ? 2.0
                                  : (double)ht->known_keys / (double)std::max<int64_t>(1, ht->dim_rows);
    }
    const bool ok = bound * 16.0 <= 1.0 && fact->placement != HX_PLACE_HOST_PINNED &&
                    fact->placement != HX_PLACE_HOST_MAPPED &&
                    std::getenv("HX_NO_GATHER") == nullptr;  // (any size: launch segments keep
                                                             // row offsets 32-bit)
    auto read_by_stages = [&](int32_t col) {
      for (int q = 0; q < sh->n_preds; ++q)
        if (sh->preds[q].col_id == col) return true;
      for (int j = 0; j < sh->n_joins; ++j)
        if (sh->join_fk_col[j] == col) return true;
      return false;
    };
    HX_REQUIRE(table_has_col(fact, sh->agg_a) &&
                   (sh->agg_op == HX_AGG_SUM || table_has_col(fact, sh->agg_b)),
               HX_EINVAL, "hx_pipeline_probe_agg: measure column not in fact table");
    p.ga = ok && !read_by_stages(sh->agg_a);
    p.gb = sh->agg_op == HX_AGG_SUM ? p.ga : (ok && !read_by_stages(sh->agg_b));
    p.gat_a = p.ga ? table_col(fact, sh->agg_a) : nullptr;
    p.gat_b = p.gb ? table_col(fact, sh->agg_op == HX_AGG_SUM ? sh->agg_a : sh->agg_b) : nullptr;
  }
  p.agg_a = p.ga ? 0 : stage_of(sh->agg_a);
  p.agg_b = sh->agg_op == HX_AGG_SUM ? p.agg_a : (p.gb ? 0 : stage_of(sh->agg_b));
  HX_REQUIRE(p.agg_a >= 0 && p.agg_b >= 0, HX_EINVAL,
             "hx_pipeline_probe_agg: measure column not in fact table (or > 8 columns)");
  HX_REQUIRE(k1_group_bound(sh, hts, n_hts) >= 1, HX_EINVAL, "hx_pipeline_probe_agg: bad gdim_join");
  for (int g = 0; g < sh->n_gdims; ++g) {
    k.gh[g] = hts[sh->join_ht[sh->gdim_join[g]]]->hdr;
    (&k.gj.x)[g] = sh->gdim_join[g];
  }
  k.n_gdims = sh->n_gdims;
  k.cap_groups = agg->cap_groups;
  k.prep_grid = (int)std::max<long long>(1, std::min<long long>((agg->cap_groups + 255) / 256,
                                                                (long long)ctx->n_sms * 4));
  // tiles: the head rows up to 16-byte alignment are handled separately (device tables; a
  // host-resident table is staged block by block into aligned device buffers instead)
  k.host = fact->placement == HX_PLACE_HOST_PINNED;
  k.mapped = fact->placement == HX_PLACE_HOST_MAPPED;
  const uintptr_t mis = k.host ? 0 : reinterpret_cast<uintptr_t>(table_col(fact, ids[0])) & 15u;
  for (int c = 0; c < n_cols && !k.host; ++c)
    HX_REQUIRE((reinterpret_cast<uintptr_t>(table_col(fact, ids[c])) & 15u) == mis &&
                   (mis & 3u) == 0,
               HX_EUNSUPPORTED, "hx_pipeline_probe_agg: columns with different alignment");
  for (int c = 0; c < n_cols && k.host; ++c) k.host_col[c] = table_col(fact, ids[c]);
  const int64_t head = std::min<int64_t>(fact->n_rows, mis ? (16 - (int64_t)mis) / 4 : 0);
  p.n_cols = n_cols;
  for (int c = 0; c < n_cols; ++c) {
    p.head_col[c] = table_col(fact, ids[c]);
    p.col[c] = p.head_col[c] + head;
  }
  p.head_rows = (int32_t)head;
  p.n_rows = fact->n_rows - head;
  p.n_tiles = (p.n_rows + kTileRows - 1) / kTileRows;
  p.meta = agg->meta;
  p.g_sum = agg->sums;
  p.g_cnt = agg->cnts;
  const bool grouped = sh->n_gdims > 0;
  p.smem_groups = grouped ? (int32_t)std::min<long long>(kSmemGroups, agg->cap_groups) : 0;
  // Shared-memory plan. The tile ring keeps pick_stages' depth (measured: shrinking it to fit
  // more filters lost 6% at SF100); the rest of the CTA's shared memory holds per-join
  // structures: hash-table pipelines get Bloom filters greedily (plan_ht below); direct-map
  // pipelines are planned by a cost model over every combination (plan_dm).
  // The shared-memory plan, for one consumer-warp count W (both instances are planned and the
  // better one launched, see kWarpsHi).
  auto plan_with = [&](const int W, K1Prepared& k) {
    K1Params& p = k.p;
    t_smem_cap = 0;
    p.stages = pick_stages(W, dm_mode, n_cols, p.smem_groups);
    int kind[HX_MAX_JOINS] = {kStNone, kStNone, kStNone, kStNone};
    int bloom_w[HX_MAX_JOINS] = {0, 0, 0, 0};
    int in_s[HX_MAX_JOINS] = {0, 0, 0, 0};
    double pass[HX_MAX_JOINS] = {1, 1, 1, 1};
    bool known[HX_MAX_JOINS] = {false, false, false, false};
    int bloom_w0[HX_MAX_JOINS] = {0, 0, 0, 0};
    int64_t keys[HX_MAX_JOINS] = {0, 0, 0, 0};
    for (int j = 0; j < sh->n_joins; ++j) {
      const hx_ht* ht = hts[sh->join_ht[j]];
      if (ht->known_keys < 0) continue;
      known[j] = true;
      keys[j] = ht->known_keys;
      pass[j] = (double)ht->known_keys / (double)std::max<int64_t>(1, ht->dim_rows);
      bloom_w0[j] = std::max(4, 1 << std::min(ht->max_bloom_log2w, bloom_log2w_for(ht->known_keys)));
    }
    auto fits_sizes = [&](const int* kd, const int* bw, bool in_place) {
      int fw = 0, db = 0;
      for (int j = 0; j < sh->n_joins; ++j) {
        const JoinDev& d = p.joins[j];
        if (kd[j] == kStFull) db += d.dm_words * 4;
        if (kd[j] == kStBitmap) db += d.bm_words * 4;
        if (kd[j] == kStBloom) fw += bw[j];
      }
      return k1_smem_bytes(W, dm_mode, n_cols, p.stages, p.smem_groups, fw, db, in_place) <=
             k1_smem_cap();
    };
    double plan_cost = -1.0;
    if (dm_mode) {
      bool grouped_j[HX_MAX_JOINS] = {false, false, false, false};
      for (int g = 0; g < sh->n_gdims; ++g) grouped_j[sh->gdim_join[g]] = true;
      plan_cost = plan_dm(sh->n_joins, p.joins, known, pass, keys, bloom_w0, grouped_j, fits_sizes,
                          kind, bloom_w, in_s);
      // An L2-lookup-bound plan (SF1000 Q3.1/Q4.1: 2-15 MB maps read for most rows) runs faster
      // with less shared memory and the freed part of the SM's array as L1 for the map reads:
      // replan within 164 KB, or within a 4-stage ring (tile pairs) for wide pipelines
      // (measured at SF1000 per 600 M rows: Q3.1 4.68 -> 3.59 ms, Q4.1 6.55 -> 4.02 ms; a
      // 3-stage ring (no pairs) gave Q4.1 5.03; plans below the threshold — every SF10/SF100
      // plan — lose with the cap).
      if (plan_cost > kL1BoundCost && !std::getenv("HX_K1_SMEM_KB")) {
        t_smem_cap = std::max<size_t>(164 * 1024, k1_smem_bytes(W, dm_mode, n_cols, kBaseStages, p.smem_groups));
        p.stages = pick_stages(W, dm_mode, n_cols, p.smem_groups);
        for (int j = 0; j < HX_MAX_JOINS; ++j) kind[j] = kStNone, bloom_w[j] = 0, in_s[j] = 0;
        plan_cost = plan_dm(sh->n_joins, p.joins, known, pass, keys, bloom_w0, grouped_j,
                            fits_sizes, kind, bloom_w, in_s);
      }
      // every join read from L2 in stage S and no shared-memory structure (the §6.4 1:N join):
      // a 100 KB ring leaves the rest as L1 for the map (measured: 248 -> 273 G rows/s)
      bool all_l2s = sh->n_joins > 0 && !std::getenv("HX_K1_SMEM_KB");
      for (int j = 0; j < sh->n_joins; ++j) all_l2s = all_l2s && kind[j] == kStNone && in_s[j];
      if (all_l2s) t_smem_cap = 100 * 1024;
    } else {
      // hash tables: selective joins (at most half the dimension passes), most selective first,
      // get a Bloom filter (folded to 4 or 2 bits per key when the full one does not fit).
      // The ring gives up a stage when that lets more selective joins carry a filter of >= 4
      // bits per key (measured at SF100: Q2.1 3.10 -> 2.55 ms, Q4.1 10.3 -> 8.5, Q4.2 5.3 ->
      // 4.4; plans that already had their filters lose 5-15% with the shallower ring)
      int ord[HX_MAX_JOINS] = {0, 1, 2, 3};
      std::stable_sort(ord, ord + sh->n_joins, [&](int x, int y) { return pass[x] < pass[y]; });
      auto allocate = [&]() {  // greedy Bloom budget at the current ring depth -> good filters
        int good = 0;
        for (int j = 0; j < HX_MAX_JOINS; ++j) kind[j] = kStNone, bloom_w[j] = 0;
        for (int i = 0; i < sh->n_joins; ++i) {
          const int j = ord[i];
          if (!known[j] || 2 * pass[j] > 1.0) continue;
          for (int f = 1; f <= 8 && kind[j] == kStNone && bloom_w0[j] / f >= 4; f *= 2) {
            kind[j] = kStBloom;
            bloom_w[j] = bloom_w0[j] / f;
            if (!fits_sizes(kind, bloom_w, false)) {
              kind[j] = kStNone;
              bloom_w[j] = 0;
            }
          }
          good += kind[j] == kStBloom && 32.0 * bloom_w[j] >= 4.0 * (double)keys[j];
        }
        return good;
      };
      const int stages0 = p.stages;
      const int good0 = allocate();
      const int ht3 = (3 * kBaseStages + 3) / 4;  // 3/4 of the base ring
      int ht_stages = stages0 > ht3 ? ht3 : stages0;
#if HX_HT_GIVEUP_MINCOLS
      if (n_cols < HX_HT_GIVEUP_MINCOLS) ht_stages = stages0;
#endif
      if (const char* e = std::getenv("HX_HT_STAGES")) ht_stages = std::max(2, std::min(stages0, std::atoi(e)));
      if (ht_stages < stages0) {
        p.stages = ht_stages;
        const int good1 = allocate();
        if (good1 <= good0 && !std::getenv("HX_HT_STAGES")) {  // no better: keep the deeper ring
          p.stages = stages0;
          allocate();
        }
      }
    }
    // hash tables: stage C probes the join a row most likely fails (given that it passed
  // every Bloom filter) alone, and the others only for its hits, when that saves at least
  // kHtSeqMin probes per row (the second round trip costs one L2 latency per batch).
  // Measured at SF100 (saved -> K1 ms): Q4.1 0.62: 8.74 -> 5.97, Q3.1 0.42: 4.70 -> 3.78;
  // Q4.2 0.18: 4.67 -> 5.09 and Q2.1 0.09: 2.93 -> 3.18 lose.
  constexpr double kHtSeqMin = 0.3;
  p.ht_seq = 0;
  p.ht_first = 0;
  double ht_saved = 0.0;
  if (!dm_mode && sh->n_joins > 1) {
    const int j0 = (p.n_preds == 0 && kind[0] != kStBloom) ? 1 : 0;  // stage B probes join 0
    double f_c = 1.0, cmin = 2.0;
    int ht_first_c = j0;
    for (int j = j0; j < sh->n_joins; ++j) {
      double c = known[j] ? pass[j] : 1.0;
      if (kind[j] == kStBloom) {
        const double fp = bloom_fp(32.0 * bloom_w[j] / (double)std::max<int64_t>(1, keys[j]));
        f_c *= c + (1.0 - c) * fp;
        c = c / std::max(1e-9, c + (1.0 - c) * fp);
      }
      if (c < cmin) cmin = c, ht_first_c = j;
    }
    // probes per row saved by probing it alone: (stage-C joins - 1) x its miss fraction
    ht_saved = f_c * (sh->n_joins - j0 - 1) * (1.0 - cmin);
    double min_saved = kHtSeqMin;
    if (const char* e = std::getenv("HX_HT_FIRST_MIN")) min_saved = std::atof(e);
    p.ht_seq = ht_saved >= min_saved;
    p.ht_first = ht_first_c;
  }
  if (const char* e = std::getenv("HX_HT_SEQ")) p.ht_seq = std::atoi(e) != 0;
  // hash tables: stage B probes join 0 in place for the rows the stage-F Bloom filter passed
  // (no lineorder predicate, join 0 unfiltered). When join 0 carries the filter instead, the
  // join stage C would probe alone (rule 1) — or else the most selective unfiltered join
  // passing at most half the rows (rule 2; HX_HT_INPLACE = 0 off, 1, 2, 3 both: default) — is
  // moved to the front of the probe order
  // (results do not depend on it; the group layout follows the grouping joins wherever they
  // sit), so that it is probed in place, 4 loads in flight per lane, instead of in stage C.
  // Measured at SF100 (profiles/r02_ab_reentry.txt): 3 joins, Q3.1 3.79 -> 3.00 ms; 4 joins,
  // Q4.1 5.61 -> 4.95 with the 20-warp static-chunk instance (7.04 with the claiming one).
  int ht_inplace = -1;
  int ht_inplace_maxj = 4;
  if (const char* e = std::getenv("HX_HT_INPLACE_MAXJ")) ht_inplace_maxj = std::atoi(e);
  if (!dm_mode && sh->n_joins > 1 && sh->n_joins <= ht_inplace_maxj && p.n_preds == 0 &&
      kind[0] == kStBloom) {
    int rule = 3;
    if (const char* e = std::getenv("HX_HT_INPLACE")) rule = std::atoi(e);
    if ((rule & 1) && p.ht_seq && kind[p.ht_first] != kStBloom) ht_inplace = p.ht_first;
    // rule 2: the most selective unfiltered join (pass <= 1/2) — when the stage-C Bloom
    // filters of the other joins keep at least 1/10 of the rows stage F passed (else stage C
    // would probe that join for far fewer rows than stage B: Q4.3 2.40 -> 2.91 ms; Q4.2, whose
    // stage-C filters keep 0.29, 4.38 -> 3.72)
    if ((rule & 2) && ht_inplace < 0) {
      double keep = 1.0;
      for (int j = 1; j < sh->n_joins; ++j)
        if (kind[j] == kStBloom && known[j])
          keep *= pass[j] + (1.0 - pass[j]) *
                                bloom_fp(32.0 * bloom_w[j] / (double)std::max<int64_t>(1, keys[j]));
      double best = 0.5 + 1e-9;
      if (keep >= 0.1)
        for (int j = 0; j < sh->n_joins; ++j)
          if (kind[j] != kStBloom && known[j] && pass[j] < best) best = pass[j], ht_inplace = j;
    }
  }
  // offsets: Bloom filters in the filter region, maps and bitmaps in the direct-map region
    p.filter_words = 0;
    p.dm_bytes = 0;
    for (int j = 0; j < sh->n_joins; ++j) {
      JoinDev& d = p.joins[j];
      d.bloom_words = 0;
      d.dm_smem = -1;
      d.bm_smem = -1;
      if (kind[j] == kStBloom) {
        d.bloom_words = bloom_w[j];
        p.filter_words += bloom_w[j];
      } else if (kind[j] == kStFull) {
        d.dm_smem = p.dm_bytes;
        p.dm_bytes += d.dm_words * 4;
      } else if (kind[j] == kStBitmap) {
        d.bm_smem = p.dm_bytes;
        p.dm_bytes += d.bm_words * 4;
      }
      d.in_s = in_s[j];
    }
    p.m_dm = p.m_dmsm = p.m_bm = p.m_ins = p.m_l2 = p.m_l2s = p.m_res = 0u;
    {
      bool grouped_j[HX_MAX_JOINS] = {false, false, false, false};
      for (int g = 0; g < sh->n_gdims; ++g) grouped_j[sh->gdim_join[g]] = true;
      for (int j = 0; j < sh->n_joins; ++j) {
        const JoinDev& d = p.joins[j];
        const bool dm = d.dm != nullptr, full = dm && d.dm_smem >= 0, bm = dm && d.bm_smem >= 0;
        p.m_dm |= (uint32_t)dm << j;
        p.m_dmsm |= (uint32_t)full << j;
        p.m_bm |= (uint32_t)bm << j;
        p.m_ins |= (uint32_t)(d.in_s != 0) << j;
        const bool l2s = dm && d.in_s && !full && !bm && d.bloom_words == 0;
        p.m_l2s |= (uint32_t)l2s << j;
        p.m_res |= (uint32_t)(d.in_s && (full || l2s)) << j;
        // the L2 map in stage C: for the rank of a grouping join, or for the verdict when no
        // exact one is known (no structure, or a Bloom filter)
        p.m_l2 |= (uint32_t)(dm && !full && (grouped_j[j] || !(bm || l2s))) << j;
      }
    }
    // a pipeline whose joins all resolve in stage S aggregates in place: no per-warp queues or
    // carry buffers. Shared memory the plan left over deepens the tile ring (up to 80 KB per column:
    // more bytes in flight per SM while the consumers hold a pair of tiles).
    const bool in_place = sh->n_joins == 0 ||
                          (dm_mode && p.m_res == (1u << sh->n_joins) - 1u);
    p.smem_fixed = in_place ? kSmemQueueOff : smem_fixed(dm_mode, W);
    {
      int max_stages = kMaxStages;
      if (const char* e = std::getenv("HX_K1_MAX_STAGES")) max_stages = std::max(2, std::min(kMaxStages, std::atoi(e)));
      while (p.stages < max_stages &&
             k1_smem_bytes(W, dm_mode, n_cols, p.stages + 1, p.smem_groups, p.filter_words, p.dm_bytes,
                           in_place) <= k1_smem_cap())
        ++p.stages;
    }
    p.stage_magic = (uint32_t)((uint64_t(1) << 32) / (uint64_t)p.stages + 1);
    // (measured, SF10: a distance of 2 gains 4-7% on the 4-column pipelines whose ring stays at
    // 4 stages, and loses 3-6% on 3-column ones, whose rings are deeper or whose tiles are
    // consumed faster)
    p.prefetch = (n_cols >= 4 && p.stages <= kBaseStages && fact->placement != HX_PLACE_HOST_MAPPED)
                     ? 2 * kBaseStages / 4 : 0;
    // L2 residency of the probe structures (north_star; PAPER.md:1016-1022 operator state in
    // device memory): probe loads carry an evict_last hint, and the largest structure K1 reads
    // from L2 (a direct map not staged in shared memory, or a hash table's slots) gets a
    // persisting access-policy window. HX_L2_HINT=0 / hx_ctx_set_option(HX_OPT_L2_PERSIST, 0):
    // A/B switches.
    p.l2_hint = 1;
    if (const char* e = std::getenv("HX_L2_HINT")) p.l2_hint = std::atoi(e) != 0;
    if (ctx->l2_persist && ctx->l2_persist_max > 0) {
      for (int j = 0; j < sh->n_joins; ++j) {
        const JoinDev& d = p.joins[j];
        const hx_ht* ht = hts[sh->join_ht[j]];
        void* base = nullptr;
        size_t bytes = 0;
        if (d.dm) {
          if (d.dm_smem < 0 && (((p.m_l2 | p.m_l2s) >> j) & 1u)) {
            base = const_cast<uint32_t*>(d.dm);
            bytes = (size_t)d.dm_words * 4;
          }
        } else {
          int lg = ht->max_log2cap;
          if (ht->known_keys >= 0) {
            lg = kMinLog2Cap;
            while (lg < ht->max_log2cap && (int64_t(1) << lg) < 4 * ht->known_keys) ++lg;
          }
          base = ht->slots;
          bytes = (size_t(1) << lg) * 8;
        }
        if (bytes > k.win.bytes) {
          k.win.base = base;
          k.win.bytes = std::min<size_t>(bytes, (size_t)ctx->l2_window_max);
        }
      }
      if (k.win.bytes)
        k.win.hit_ratio = (float)std::min(1.0, (double)ctx->l2_persist_max / (double)k.win.bytes);
    }
    if (const char* e = std::getenv("HX_K1_PREFETCH")) p.prefetch = std::max(0, std::min(64, std::atoi(e)));

    if (std::getenv("HX_DEBUG")) {  // launch plan of this K1 (tuning aid)
      std::fprintf(stderr, "[hx] K1 warps=%d joins=%d cols=%d gather=%d%d stages=%d groups=%d filters:",
                   W, sh->n_joins, n_cols, p.ga, p.gb, p.stages, p.smem_groups);
      for (int j = 0; j < sh->n_joins; ++j) std::fprintf(stderr, " %d", p.joins[j].bloom_words);
      std::fprintf(stderr, " dm(words@smem/bitmap@smem):");
      for (int j = 0; j < sh->n_joins; ++j)
        std::fprintf(stderr, " %d@%d/%d@%d", p.joins[j].dm ? p.joins[j].dm_words : 0,
                     p.joins[j].dm_smem, p.joins[j].bm_words, p.joins[j].bm_smem);
      std::fprintf(stderr, " in_s:");
      for (int j = 0; j < sh->n_joins; ++j) std::fprintf(stderr, "%d", p.joins[j].in_s);
      std::fprintf(stderr, " ht_seq=%d first=%d saved=%.3f inplace=%d", p.ht_seq, p.ht_first, ht_saved, ht_inplace);
      std::fprintf(stderr, " l2:%x l2s:%x cost=%.2f stages=%d smem=%zu\n", p.m_l2, p.m_l2s, plan_cost, p.stages,
                   k1_smem_bytes(W, dm_mode, n_cols, p.stages, p.smem_groups, p.filter_words, p.dm_bytes,
                                 in_place));
    }
    if (ht_inplace > 0) {  // rotate join ht_inplace to the front (hash-table plans: no masks)
      const int jb = ht_inplace;
      auto mapj = [jb](int j) { return j == jb ? 0 : (j < jb ? j + 1 : j); };
      const JoinDev moved = p.joins[jb];
      for (int j = jb; j > 0; --j) p.joins[j] = p.joins[j - 1];
      p.joins[0] = moved;
      for (int g = 0; g < sh->n_gdims; ++g) (&k.gj.x)[g] = mapj((&k.gj.x)[g]);
      p.ht_first = mapj(p.ht_first);
    }
    if (ht_inplace >= 0) p.ht_seq = 0;
    k.fn = pick_kernel(sh->n_joins, grouped, p.m_dm != 0u, W);
    k.smem = k1_smem_bytes(W, dm_mode, n_cols, p.stages, p.smem_groups, p.filter_words, p.dm_bytes,
                           in_place);
    // the smallest shared-memory carveout that holds the plan: the rest of the SM's L1/shared
    // array caches the maps read from L2
    k.carveout = (int)std::min<size_t>(100, ((k.smem + 1024) * 100 + 228 * 1024 - 1) / (228 * 1024));
    k.warps = W;
    k.cost = plan_cost;
  };
  // Direct maps: the plan is also made around a ring one stage deeper, and taken when the cost
  // model charges that at most kDeepTol more (a deeper ring keeps more bytes in flight while
  // the consumers hold their chunks; the model does not see it). Measured at SF100
  // (profiles/r02_ab_reentry.txt): Q2.2 1.45 -> 1.29 ms (+5% cost), Q3.2 1.48 -> 1.36 (+8%),
  // Q3.3 1.28 -> 1.15 (+0.3%), Q3.1 2.07 -> 2.03; Q2.1 (+29% cost) 1.69 -> 1.74 keeps 4.
  auto plan_deeper = [&](const int W, K1Prepared& kk) {
    plan_with(W, kk);
    if (!dm_mode || std::getenv("HX_K1_MIN_STAGES")) return;
    constexpr double kDeepTol = 1.10;
    K1Prepared deep = k;
    t_base_stages = kBaseStages + 1;
    plan_with(W, deep);
    t_base_stages = 0;
    if (deep.p.stages > kk.p.stages && deep.cost <= kk.cost * kDeepTol + 1e-9) kk = deep;
  };
  K1Prepared k_lo = k, k_hi = k;
  plan_deeper(kWarpsLo, k_lo);
  plan_deeper(dm_mode ? kWarpsHi : kWarpsHiHt, k_hi);
  // more warps unless the plan they leave room for is costlier by more than kWarpsTol (the
  // cost model's per-row issue cost; tolerance measured) or the ring is shallower
  double tol = 1.10;
  if (const char* e = std::getenv("HX_K1_W_TOL")) tol = std::atof(e);
  bool hi = k_hi.p.stages >= std::min(k_lo.p.stages, kBaseStages) &&
            (dm_mode ? k_hi.cost <= k_lo.cost * tol + 1e-9
                     : k_hi.p.filter_words >= k_lo.p.filter_words);
  // (an L2-lookup-bound plan runs with a reduced carveout so that L1 caches its map reads:
  // the extra warps' queues take from that L1 and their misses thrash it — SF1000 Q4.1
  // measured 6.16 ms with 26 warps vs 4.11 with 20, same plan)
  if (dm_mode && k_lo.cost > kL1BoundCost) hi = false;
  // hash tables: the 20-warp instances run at 80 registers (the 26-warp ones at 72, spilling
  // with 3-4 joins); 26 warps pay where latency hiding dominates — stage B probing a join in
  // place for most rows, or 4 joins — and 20 where stage C's per-row work does (measured at
  // SF100, profiles/r02_ab_reentry.txt: Q2.1 3.26 -> 2.61 ms, Q3.2 2.92 -> 1.95 with 20;
  // Q3.1 in place 2.97 vs 3.03, Q4.1 5.56 vs 5.71 with 26)
  if (!dm_mode && sh->n_joins >= 2 && sh->n_joins <= 3) {
    // (a 26-warp plan that probes in place beats a 20-warp one with one more Bloom filter:
    // Q2.1 2.62 -> 2.42 ms)
    const bool stage_b = k_hi.p.n_preds == 0 && k_hi.p.joins[0].bloom_words == 0;
    hi = stage_b && k_hi.p.stages >= std::min(k_lo.p.stages, kBaseStages);
  }
  // (4 joins: the claiming 26-warp instance unless stage B probes in place, which the static
  // 20-warp one does best)
  if (!dm_mode && sh->n_joins == 4 && k_lo.p.n_preds == 0 && k_lo.p.joins[0].bloom_words == 0)
    hi = false;
  if (const char* e = std::getenv("HX_K1_W")) hi = std::atoi(e) != kWarpsLo;
  k = hi ? k_hi : k_lo;
  t_smem_cap = 0;
  int occ = 0;
  HX_CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, k.fn, k1_threads(k.warps), k.smem));
  occ = std::max(1, occ);
  k.occ = occ;
  k.grid = (int)std::max<int64_t>(1, std::min<int64_t>(p.n_tiles, (int64_t)ctx->n_sms * occ));
  k.rows = fact->n_rows;
  k.n_cols = n_cols;
  if (const char* e = std::getenv("HX_K1_SEG_TILES")) {
    const long long t = std::atoll(e);
    if (t > 0 && t <= (1LL << 20)) k.seg_rows = t * kTileRows;
  }
  if (sh->n_joins == 0 && n_cols >= 1 && n_cols <= 4 && !k.host &&
      std::getenv("HX_NO_SCAN") == nullptr) {
    const KernelFn scans[4] = {k1_scan_agg<1>, k1_scan_agg<2>, k1_scan_agg<3>, k1_scan_agg<4>};
    k.scan = scans[n_cols - 1];
    k.scan_smem = scan_smem(n_cols);
    const int64_t tiles = (p.n_rows + scan_rows(n_cols) - 1) / scan_rows(n_cols);
    k.scan_grid = (int)std::max<int64_t>(1, std::min<int64_t>(tiles, (int64_t)ctx->n_sms));
  }
  *out = new K1Prepared(k);
  return HX_OK;
}

bool k1_is_host(const K1Prepared* k) { return k->host; }

int ring_create(hx_ctx* ctx, const K1Prepared* k, int64_t block_rows, StageRing** out) {
  HX_REQUIRE(block_rows > 0 && block_rows % 4 == 0, HX_EINVAL, "staging block must be a multiple of 4 rows");
  StageRing* r = new StageRing();
  r->block_rows = std::min<int64_t>(block_rows, std::max<int64_t>(4, (k->rows + 3) & ~int64_t(3)));
  r->n_cols = k->n_cols;
  const size_t col_bytes = ((size_t)r->block_rows * 4 + 255) & ~size_t(255);
  cudaError_t e = cudaMallocAsync(&r->base, col_bytes * r->n_cols * kRingStages, ctx->stream);
  if (e != cudaSuccess) {
    delete r;
    return cuda_fail(e, "cudaMallocAsync(staging ring)", __FILE__, __LINE__);
  }
  for (int s = 0; s < kRingStages; ++s) {
    for (int c = 0; c < r->n_cols; ++c)
      r->buf[s][c] = reinterpret_cast<int32_t*>(static_cast<char*>(r->base) +
                                                col_bytes * (s * r->n_cols + c));
    cudaEventCreateWithFlags(&r->full[s], cudaEventDisableTiming);
    cudaEventCreateWithFlags(&r->freed[s], cudaEventDisableTiming);
  }
  *out = r;
  return HX_OK;
}

void ring_destroy(hx_ctx* ctx, StageRing* r) {
  if (!r) return;
  if (r->base) cudaFreeAsync(r->base, ctx->stream);
  for (int s = 0; s < kRingStages; ++s) {
    if (r->full[s]) cudaEventDestroy(r->full[s]);
    if (r->freed[s]) cudaEventDestroy(r->freed[s]);
  }
  delete r;
}

// K1 over a host-resident fact table: block b is copied H2D into ring slot b % 3 on the copy
// stream (after K1 released that slot), K1 runs on it on the compute stream and accumulates
// into the same group arrays. Copies of the next blocks overlap the current K1.
static int k1_enqueue_host(hx_ctx* ctx, const K1Prepared* k, StageRing* ring, cudaEvent_t e0,
                           cudaEvent_t e1) {
  HX_REQUIRE(ring && ring->n_cols == k->n_cols, HX_EINVAL, "host-resident K1 needs a staging ring");
  const int64_t B = ring->block_rows;
  const int64_t nb = (k->rows + B - 1) / B;
  if (e0) HX_CK(record_event(e0, ctx->stream));
  HX_CK(cudaEventRecord(ctx->fork_ev, ctx->stream));
  HX_CK(cudaStreamWaitEvent(ctx->copy_stream, ctx->fork_ev, 0));
  for (int64_t b = 0; b < nb; ++b) {
    const int s = (int)(b % kRingStages);
    const int64_t r0 = b * B, rows = std::min<int64_t>(B, k->rows - r0);
    if (b >= kRingStages) HX_CK(cudaStreamWaitEvent(ctx->copy_stream, ring->freed[s], 0));
    for (int c = 0; c < k->n_cols; ++c)
      HX_CK(cudaMemcpyAsync(ring->buf[s][c], k->host_col[c] + r0, (size_t)rows * 4,
                            cudaMemcpyHostToDevice, ctx->copy_stream));
    ctx->h2d_bytes += rows * 4 * k->n_cols;
    HX_CK(cudaEventRecord(ring->full[s], ctx->copy_stream));
    HX_CK(cudaStreamWaitEvent(ctx->stream, ring->full[s], 0));
    K1Params p = k->p;
    for (int c = 0; c < k->n_cols; ++c) p.col[c] = p.head_col[c] = ring->buf[s][c];
    p.head_rows = 0;
    p.n_rows = rows;
    p.n_tiles = (rows + kTileRows - 1) / kTileRows;
    const int grid = (int)std::max<int64_t>(1, std::min<int64_t>(p.n_tiles, (int64_t)ctx->n_sms * k->occ));
    HX_CK(launch_k1(k->fn, grid, k1_threads(k->warps), k->smem, ctx->stream, p, ctx->k1_priority));
    ctx->launches += 1;
    HX_CK(cudaEventRecord(ring->freed[s], ctx->stream));
  }
  // the copy stream rejoins the compute stream (required under graph capture)
  HX_CK(cudaEventRecord(ctx->fork_ev, ctx->copy_stream));
  HX_CK(cudaStreamWaitEvent(ctx->stream, ctx->fork_ev, 0));
  if (e1) HX_CK(record_event(e1, ctx->stream));
  return HX_OK;
}

// K1 over a host-resident fact table whose blocks are handed out by a shared router (dynamic
// load balancing across the processes of a node): the host draws a block only when a staging
// slot is free (it waits for the slot's previous K1 with cudaEventSynchronize), so each GPU
// takes blocks at the rate it consumes them. Not capturable (host-driven).
int k1_enqueue_routed(hx_ctx* ctx, const K1Prepared* k, StageRing* ring, hx_shared_router* router,
                      int64_t* n_blocks) {
  HX_REQUIRE(ring && ring->n_cols == k->n_cols && k->host, HX_EINVAL,
             "routed K1 needs a host-resident table and a staging ring");
  const int64_t B = ring->block_rows;
  int64_t mine = 0;
  HX_CK(cudaEventRecord(ctx->fork_ev, ctx->stream));
  HX_CK(cudaStreamWaitEvent(ctx->copy_stream, ctx->fork_ev, 0));
  for (int64_t used = 0;; ++used) {
    const int s = (int)(used % kRingStages);
    if (used >= kRingStages) HX_CK(cudaEventSynchronize(ring->freed[s]));  // slot free: ask for work
    int64_t b = -1;
    int rc = hx_shared_router_next(router, &b);
    if (rc != HX_OK) return rc;
    const int64_t r0 = b * B;
    if (b < 0 || r0 >= k->rows) break;
    const int64_t rows = std::min<int64_t>(B, k->rows - r0);
    if (used >= kRingStages) HX_CK(cudaStreamWaitEvent(ctx->copy_stream, ring->freed[s], 0));
    for (int c = 0; c < k->n_cols; ++c)
      HX_CK(cudaMemcpyAsync(ring->buf[s][c], k->host_col[c] + r0, (size_t)rows * 4,
                            cudaMemcpyHostToDevice, ctx->copy_stream));
    ctx->h2d_bytes += rows * 4 * k->n_cols;
    HX_CK(cudaEventRecord(ring->full[s], ctx->copy_stream));
    HX_CK(cudaStreamWaitEvent(ctx->stream, ring->full[s], 0));
    K1Params p = k->p;
    for (int c = 0; c < k->n_cols; ++c) p.col[c] = p.head_col[c] = ring->buf[s][c];
    p.head_rows = 0;
    p.n_rows = rows;
    p.n_tiles = (rows + kTileRows - 1) / kTileRows;
    const int grid = (int)std::max<int64_t>(1, std::min<int64_t>(p.n_tiles, (int64_t)ctx->n_sms * k->occ));
    HX_CK(launch_k1(k->fn, grid, k1_threads(k->warps), k->smem, ctx->stream, p, ctx->k1_priority));
    ctx->launches += 1;
    HX_CK(cudaEventRecord(ring->freed[s], ctx->stream));
    ++mine;
  }
  HX_CK(cudaEventRecord(ctx->fork_ev, ctx->copy_stream));
  HX_CK(cudaStreamWaitEvent(ctx->stream, ctx->fork_ev, 0));
  if (n_blocks) *n_blocks = mine;
  return HX_OK;
}

int probe_agg_routed(hx_ctx* ctx, const hx_table* fact, const hx_query_shape* sh, hx_ht* const* hts,
                     int n_hts, hx_agg* agg, hx_shared_router* router, int64_t block_rows,
                     int64_t* n_blocks) {
  HX_REQUIRE(ctx && fact && sh && agg && router, HX_EINVAL, "hx_pipeline_probe_agg_routed: null argument");
  HX_REQUIRE(fact->placement == HX_PLACE_HOST_PINNED, HX_EINVAL,
             "hx_pipeline_probe_agg_routed: the fact table must be HX_PLACE_HOST_PINNED");
  HX_REQUIRE(block_rows > 0 && block_rows % 4 == 0, HX_EINVAL,
             "hx_pipeline_probe_agg_routed: block_rows must be a positive multiple of 4");
  const long long bound = k1_group_bound(sh, hts, n_hts);
  HX_REQUIRE(bound >= 1, HX_EINVAL, "hx_pipeline_probe_agg_routed: bad gdim_join / join_ht");
  int rc = agg_alloc(ctx, agg, bound, sh, hts);
  if (rc != HX_OK) return rc;
  K1Prepared* k = nullptr;
  rc = k1_setup(ctx, fact, sh, hts, n_hts, agg, &k);
  if (rc != HX_OK) return rc;
  for (int j = 0; j < sh->n_joins; ++j) agg->deps.push_back(hts[sh->join_ht[j]]);
  StageRing* ring = nullptr;
  rc = k1_enqueue_prepare(ctx, k, true, ctx->stream);
  if (rc == HX_OK && k->rows > 0) rc = ring_create(ctx, k, block_rows, &ring);
  if (rc == HX_OK && k->rows > 0) rc = k1_enqueue_routed(ctx, k, ring, router, n_blocks);
  else if (n_blocks) *n_blocks = 0;
  ring_destroy(ctx, ring);
  k1_free(k);
  return rc;
}

// prepare (group layout + zeroing when `fresh`) then K1; optional timing events around K1.
int k1_enqueue_prepare(hx_ctx* ctx, const K1Prepared* k, bool fresh, cudaStream_t s) {
  const K1Params& p = k->p;
  k1_prepare<<<k->prep_grid, 256, 0, s>>>(const_cast<AggMeta*>(p.meta), k->gh[0], k->gh[1],
                                          k->gh[2], k->n_gdims, k->gj, p.g_sum, p.g_cnt,
                                          k->cap_groups, fresh ? 1 : 0);
  HX_CK_LAUNCH("k1_prepare");
  ctx->launches += 1;
  return HX_OK;
}

int k1_enqueue(hx_ctx* ctx, const K1Prepared* k, bool fresh, cudaEvent_t e0, cudaEvent_t e1,
               StageRing* ring, bool prepare) {
  const K1Params& p = k->p;
  if (prepare) {
    int rc = k1_enqueue_prepare(ctx, k, fresh, ctx->stream);
    if (rc != HX_OK) return rc;
  }
  if (k->rows == 0) return HX_OK;
  if (k->host) return k1_enqueue_host(ctx, k, ring, e0, e1);
  if (e0) HX_CK(record_event(e0, ctx->stream));
  if (k->scan) {
    HX_CK(launch_k1(k->scan, k->scan_grid, kScanThreads + 32, k->scan_smem, ctx->stream, p,
                    ctx->k1_priority));
    ctx->launches += 1;
  } else {
    // K1 addresses gathered measures and carried rows by a 32-bit row offset: a table of
    // more rows (one GPU's SF1000 partition: 6e9) runs as consecutive launches over segments
    // of kSegRows rows (whole tiles, 16-byte aligned), accumulating into the same groups.
    for (int64_t s0 = 0; s0 < p.n_rows; s0 += k->seg_rows) {
      K1Params q = p;
      if (s0 > 0) {
        for (int c = 0; c < p.n_cols; ++c) q.col[c] = q.head_col[c] = p.col[c] + s0;
        q.head_rows = 0;
        if (p.ga) q.gat_a = p.gat_a + p.head_rows + s0;
        if (p.gb) q.gat_b = p.gat_b + p.head_rows + s0;
      }
      q.n_rows = std::min<int64_t>(k->seg_rows, p.n_rows - s0);
      q.n_tiles = (q.n_rows + kTileRows - 1) / kTileRows;
      const int grid = (int)std::max<int64_t>(1, std::min<int64_t>(q.n_tiles, (int64_t)k->grid));
      HX_CK(launch_k1(k->fn, grid, k1_threads(k->warps), k->smem, ctx->stream, q, ctx->k1_priority, k->carveout,
                      &k->win));
      ctx->launches += 1;
    }
  }
  if (k->mapped) ctx->h2d_bytes += k1_bytes(k);  // read over PCIe by the kernel itself
  if (e1) HX_CK(record_event(e1, ctx->stream));
  return HX_OK;
}

void k1_free(K1Prepared* k) { delete k; }
int64_t k1_bytes(const K1Prepared* k) { return k->rows * 4 * k->n_cols; }
int k1_gathered_cols(const K1Prepared* k) {
  return k->p.ga + (k->p.agg_op != HX_AGG_SUM && k->p.gb ? 1 : 0);
}

int probe_agg(hx_ctx* ctx, const hx_table* fact, const hx_query_shape* sh, hx_ht* const* hts,
              int n_hts, hx_agg* agg, bool fresh) {
  HX_REQUIRE(ctx && fact && sh && agg, HX_EINVAL, "hx_pipeline_probe_agg: null argument");
  if (fresh) {
    const long long bound = k1_group_bound(sh, hts, n_hts);
    HX_REQUIRE(bound >= 1 && sh->n_joins <= HX_MAX_JOINS && sh->n_gdims <= HX_MAX_GDIMS,
               HX_EINVAL, "hx_pipeline_probe_agg: bad gdim_join / join_ht");
    int rc = agg_alloc(ctx, agg, bound, sh, hts);
    if (rc != HX_OK) return rc;
  }
  K1Prepared* k = nullptr;
  int rc = k1_setup(ctx, fact, sh, hts, n_hts, agg, &k);
  if (rc != HX_OK) return rc;
  for (int j = 0; j < sh->n_joins; ++j) agg->deps.push_back(hts[sh->join_ht[j]]);
  cudaEvent_t e0 = nullptr, e1 = nullptr;
  if (ctx->prof_on && k->rows > 0) {
    e0 = pooled_event(ctx);
    e1 = pooled_event(ctx);
  }
  StageRing* ring = nullptr;
  if (k->host && k->rows > 0) {
    rc = ring_create(ctx, k, kHostBlockRows, &ring);
    if (rc != HX_OK) {
      k1_free(k);
      return rc;
    }
  }
  rc = k1_enqueue(ctx, k, fresh, e0, e1, ring);
  if (rc == HX_OK && e0) {
    ctx->prof_events.push_back({e0, e1});
    ctx->prof_launches += 1;
    ctx->prof_bytes += k1_bytes(k);
  }
  ring_destroy(ctx, ring);  // stream-ordered free: after the K1 launches that use it
  k1_free(k);
  return rc;
}

}  // namespace hx

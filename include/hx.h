/*
 * hx.h — C-ABI of libhx, the B200-native hot path of HetExchange (Chrysogelos et al.,
 * PVLDB 12(5) 2019): the fused GPU pipeline that runs a Star Schema Benchmark query —
 * scan lineorder → filter → probe k dimension hash tables → group-by aggregate — plus the
 * operators that spread it over GPUs (router, mem-move, broadcast, union-router merge).
 *
 * Citations are PAPER.md line ranges (the paper's text) with the section they fall in.
 * All entry points return an int status (HX_OK = 0, negative on error) and never throw;
 * hx_last_error() returns a thread-local message for the last failure of this thread.
 * Plain pointers and sizes only: no torch (or other framework) types cross this boundary.
 * Device pointers are CUDA device (or UVA) addresses; `stream` arguments are cudaStream_t
 * passed as void*. One hx_ctx drives ONE GPU (one process per GPU; §4.2
 * "pipeline template ... instantiated" per device).
 *
 * Asynchrony: every call that launches device work enqueues it on the context stream and
 * returns without synchronising, EXCEPT hx_ht_info, hx_merge_aggregates, hx_profile_read
 * and hx_ht_broadcast (the latter waits for the HT size on the root), which synchronise
 * that stream. Nothing on the path copies device results to the host before the merge.
 */
#ifndef HX_H
#define HX_H
#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

/* ---- status codes ------------------------------------------------------------------- */
enum {
  HX_OK = 0,
  HX_EINVAL = -1,        /* null / inconsistent argument                                   */
  HX_ECUDA = -2,         /* a CUDA runtime call failed (message in hx_last_error)         */
  HX_ENCCL = -3,         /* an NCCL call failed, or no communicator for a collective      */
  HX_ENOMEM = -4,        /* device or pinned host allocation failed                        */
  HX_ECAPACITY = -5,     /* group count beyond HX_MAX_GROUPS, or too many columns          */
  HX_EDUPKEY = -6,       /* a dimension primary key occurs twice among the filtered rows   */
  HX_EUNSUPPORTED = -7   /* a configuration this build does not implement                 */
};
const char* hx_last_error(void);

/* ---- context (one GPU) ------------------------------------------------------------- */
typedef struct hx_ctx hx_ctx;
/* Binds CUDA device `device`. `stream` (cudaStream_t) is the stream all work is enqueued on;
   NULL makes the library create a non-blocking stream it owns. *out owned by the library. */
int hx_init(int device, void* stream, hx_ctx** out);
int hx_finalize(hx_ctx* ctx);
int hx_ctx_stream(hx_ctx* ctx, void** stream);
/* Number of SMs and resident K1 CTAs per SM chosen for this device (for reporting). */
int hx_ctx_info(hx_ctx* ctx, int* n_sms, int* k1_ctas_per_sm);
/* Context options (read when a plan is created, hx_plan_create):
   HX_OPT_JOIN_LAYOUT: HX_JOIN_AUTO (default) lets a plan whose dimension keys are dense
   (span < 2^27, map no larger than the rule in DESIGN.md R20) probe a direct map — the hash
   table under the identity hash; HX_JOIN_HASH keeps the open-addressing hash tables
    for every plan. Same results either way (keys are unique).
   HX_OPT_L2_PERSIST: 1 reserves the device's persisting-L2 set-aside
   (cudaLimitPersistingL2CacheSize, the maximum; HX_L2_PERSIST_MB lowers it) and gives each K1
   launch an access-policy window (hitProp persisting) over its largest probe structure read
   from L2; 0 (the default) releases the set-aside. Measured on B200: the probe
   structures already hit L2 99.9% without it; the window costs ~2% and the reservation alone
   2-5% on K1 and 2x on K3. Device-wide setting: set it from one context. */
enum { HX_OPT_JOIN_LAYOUT = 1, HX_OPT_L2_PERSIST = 2 };
enum { HX_JOIN_AUTO = 0, HX_JOIN_HASH = 1 };
int hx_ctx_set_option(hx_ctx* ctx, int option, int value);

/* ---- communicator (NCCL over NVLink/NVSwitch; one rank per GPU) ------------------- */
/* The 128-byte ncclUniqueId, created on rank 0 and shipped to the others by the caller
   (e.g. torch.distributed). hx_comm_init is collective over all `nranks` ranks. */
int hx_comm_unique_id(void* id128);
int hx_comm_init(hx_ctx* ctx, int nranks, int rank, const void* id128);
int hx_comm_info(hx_ctx* ctx, int* rank, int* nranks);
/* Collective trace: every NCCL data call libhx issues on this ctx (at issue time on the host;
   a call captured into a CUDA graph is recorded once, at capture) is appended as one record:
   the operation, the element count and element size it was issued with, the root (reduce,
   broadcast) or peer (send, recv; -1 otherwise) and the device buffer. A 1-rank communicator
   turns allreduce / broadcast into identities, so this is how the tests check the sizes the
   multi-rank path would move (2 x n_groups per plan merge, the HT's bytes per broadcast).
   hx_comm_trace copies up to `cap` of the oldest retained records (the last 4096 are kept) into
   `out`, stores the number retained in *n, and clears them if `reset`. Host only; no sync. */
enum { HX_COLL_ALLREDUCE = 1, HX_COLL_REDUCE = 2, HX_COLL_BROADCAST = 3, HX_COLL_ALLGATHER = 4,
       HX_COLL_SEND = 5, HX_COLL_RECV = 6 };
typedef struct { int32_t op; int32_t root_or_peer; int64_t count; int32_t elem_bytes;
                 int32_t reserved; uint64_t buf; } hx_coll_rec;
int hx_comm_trace(hx_ctx* ctx, hx_coll_rec* out, int cap, int* n, int reset);

/* ---- router: segmenter + range / round-robin policy (§8(a) a2) ---------------------
 * PAPER.md:469-473 §3.1 (the segmenter splits the input into block-shaped partitions; the
 * router routes block handles to consumer instances while load-balancing)
 * (round-robin/range policies), Listing 1 pipeline 6. A block handle is a
 * row range plus the consumer it is routed to (handles, not data).
 * Blocks are [b*block_rows, min((b+1)*block_rows, n_rows)); HX_POLICY_RANGE gives each part
 * a contiguous run of whole blocks (balanced to within one block), HX_POLICY_ROUND_ROBIN
 * routes block b to part b % n_parts. Invariant: the blocks are disjoint and cover
 * [0, n_rows). n_rows may be 0 (no blocks). */
enum { HX_POLICY_RANGE = 0, HX_POLICY_ROUND_ROBIN = 1 };
typedef struct { int64_t row_begin, row_end; int32_t part; int32_t reserved; } hx_block;
typedef struct hx_partition hx_partition;
int hx_router_partition(int64_t n_rows, int n_parts, int64_t block_rows, int policy,
                        hx_partition** out);
/* *blocks points into library memory valid until hx_partition_free. */
int hx_partition_info(const hx_partition* p, int64_t* n_blocks, const hx_block** blocks);
/* Rows routed to `part` (sum of its blocks). */
int hx_partition_rows(const hx_partition* p, int part, int64_t* n_rows);
int hx_partition_free(hx_partition* p);

/* ---- columns: mem-move into HBM (§8(a) a1) -----------------------------------------
 * PAPER.md:500-520 §3.2 (mem-move moves each block to the consumer's memory, or only
 * forwards the handle when the data is already local), §6.1 (tables
 * partitioned over the GPUs; dimension columns broadcast to every GPU).
 * A column is `n_rows` int32 values (SoA), identified by `col_id` (ssbgen.h column ids).
 * `data` is a host or device (UVA) pointer, caller-owned, alive until the call's work
 * completes (HX_PLACE_COPY) or for the table's lifetime (HX_PLACE_VIEW).
 *   part == NULL   : all rows (replicated dimension tables).
 *   part != NULL   : only the blocks the router gave to `part_index`, concatenated in
 *                    block order (the rows this GPU owns).
 *   HX_PLACE_COPY  : library-owned device columns (cudaMemcpyAsync on the ctx stream,
 *                    H2D or D2D by UVA); base pointers 256-byte aligned.
 *   HX_PLACE_VIEW  : no copy; every `data` must be device memory and the selected rows one
 *                    contiguous range (always true for part == NULL).
 *   HX_PLACE_HOST_PINNED : no copy; `data` must be page-locked host memory; K1 then streams
 *                    blocks over PCIe through a device staging ring (mem-move, §8(a) a8).
 *   HX_PLACE_HOST_MAPPED : no copy; `data` must be page-locked, device-mapped host memory
 *                    (cudaHostAlloc / cudaHostRegister; UVA); K1's bulk copies read it
 *                    directly over PCIe (zero-copy, the UVA access of the paper's GPU
 *                    baselines, §6.4).
 *                    Fact tables only (dimension builds return HX_EUNSUPPORTED).
 * All columns of one table must have the same number of rows. At most HX_MAX_COLS. */
enum { HX_PLACE_COPY = 0, HX_PLACE_VIEW = 1, HX_PLACE_HOST_PINNED = 2, HX_PLACE_HOST_MAPPED = 3 };
#define HX_MAX_COLS 16
typedef struct { int32_t col_id; int32_t reserved; const int32_t* data; int64_t n_rows; } hx_col;
typedef struct hx_table hx_table;
int hx_load_columns(hx_ctx* ctx, const hx_col* cols, int n_cols, const hx_partition* part,
                    int part_index, int placement, hx_table** out);
int hx_table_info(const hx_table* t, int64_t* n_rows, int* n_cols);
/* A view of rows [row_begin, row_end) of `t` (no copy; lifetime bounded by `t`). */
int hx_table_slice(const hx_table* t, int64_t row_begin, int64_t row_end, hx_table** out);
int hx_table_free(hx_table* t);
/* Copies rows [row_begin, row_begin + n) of column `col_id` of `t` (device or host resident)
   into caller host memory `dst` (n int32). Synchronises the ctx stream. */
int hx_table_read(const hx_table* t, int32_t col_id, int64_t row_begin, int64_t n, int32_t* dst);
/* Copies n int32 values from caller memory `src` (host — pinned for an asynchronous copy — or
   device) into rows [row_begin, row_begin + n) of column `col_id` of the device table `t`
   (HX_PLACE_COPY or HX_PLACE_VIEW), on the ctx stream; asynchronous, `src` must stay valid
   until the stream reaches the copy. Refreshes the data under prepared plans (mem-move into
   existing HBM buffers); a plan must be re-created if a dimension's keys or group codes
   change beyond what it was sized for (hx_plan_enqueue reports it). */
int hx_table_write(hx_table* t, int32_t col_id, int64_t row_begin, int64_t n, const int32_t* src);

/* ---- dimension filter + hash-table build (§8(a) a3, kernel K2) ----------------------
 * PAPER.md:1160-1163 §6.1 (broadcast-hash-join plans: the build side is the filtered
 * dimension), §4.3 (the hash table is operator state owned by the memory
 * manager), PAPER.md:231-233 (build-phase atomics).
 * Rows of `dim` passing the AND of `preds` (range lo <= v <= hi, or v IN in[0..n_in)) are
 * inserted as key -> rank into an open-addressing table in HBM (linear probing, 8-byte
 * slots {int32 key, int32 rank} in 16-byte buckets, capacity the power of two >=
 * 4*n_pass, min 16 — >= 2*n_pass when 4*n_pass slots would exceed 8 MB), built with
 * warp-cooperative CAS inserts. Key -1 is reserved. If group_col >= 0 its values must lie in
 * [group_lo, group_hi]; rank = position of the row's group code among the DISTINCT codes
 * of the passing rows in ascending order (dense ranks; rank_to_code recovers the code).
 * group_col < 0: membership only, rank 0, one rank.
 * Asynchronous and sync-free: the passing count, capacity and rank count live on the
 * device, so a query's builds, K1 and merge enqueue without a host round trip.
 * Errors detected on the device (duplicate key among passing rows, group code out of
 * range) are reported by hx_ht_info / hx_merge_aggregates as HX_EDUPKEY / HX_EINVAL. */
enum { HX_PRED_RANGE = 0, HX_PRED_IN = 1 };
typedef struct {
  int32_t col_id;
  int32_t kind;       /* HX_PRED_RANGE | HX_PRED_IN */
  int32_t lo, hi;     /* RANGE: lo <= v <= hi (inclusive) */
  int32_t n_in;       /* IN: 1..4 values */
  int32_t in[4];
} hx_pred;
typedef struct hx_ht hx_ht;
int hx_build_dim_ht(hx_ctx* ctx, const hx_table* dim, int32_t key_col, const hx_pred* preds,
                    int n_preds, int32_t group_col, int32_t group_lo, int32_t group_hi,
                    hx_ht** out);
/* Synchronises, then reports the table: passing keys, slots in use, distinct group codes,
   rank->code map (caller array of >= n_ranks entries, may be NULL) and HX_OK / the error
   the build detected. Any out pointer may be NULL. */
int hx_ht_info(hx_ht* ht, int64_t* n_keys, int64_t* n_slots, int32_t* n_ranks,
               int32_t* rank_to_code);
/* Mem-move broadcast of a built table from rank `root` to every rank (§8(a) a4;
   PAPER.md:530-537 §3.2 multicast is mem-move's job). Collective: every
   rank calls it; non-root ranks pass a table from hx_build_dim_ht over the same dimension
   (any preds — its contents are replaced). Requires hx_comm_init. */
int hx_ht_broadcast(hx_ctx* ctx, hx_ht* ht, int root);
int hx_ht_free(hx_ht* ht);
/* hx_build_dim_ht with build flags. HX_BUILD_IDENTITY_RANKS: the rank of group code c is
   c - group_lo for every code of [group_lo, group_hi] (n_ranks = the domain size), not its
   position among the codes present — so tables built over DIFFERENT row subsets of one
   dimension (the partitions of a hash-partitioned join, §8(f) NEXT-1) give every group the
   same index, and their partial aggregates add element-wise (union router). */
enum { HX_BUILD_IDENTITY_RANKS = 1 };
int hx_build_dim_ht_ex(hx_ctx* ctx, const hx_table* dim, int32_t key_col, const hx_pred* preds,
                       int n_preds, int32_t group_col, int32_t group_lo, int32_t group_hi,
                       int flags, hx_ht** out);

/* ---- hash-partitioned join: hash-pack + hash-routing exchange (§8(f) NEXT-1) ---------
 * PAPER.md:405-428 §3.1 (hash-based routing policies: the router sends each block's rows to
 * the consumer chosen by a hash of a key, after a hash-pack operator groups the rows by
 * destination), PAPER.md:557-561, 582-587 (Fig. 1d/e: hash-partitioned joins exchange both
 * inputs so that matching keys meet on one device). The alternative to broadcasting a
 * dimension too large to replicate.
 * hx_hash_partition (hash-pack, kernel K3): the rows of the device table `t` are permuted so
 * that the rows of part p = hx_part_of(key, n_parts) are contiguous and in part order (order
 * within a part unspecified). *out: a new library-owned device table with t's columns;
 * part_offsets (caller array of n_parts + 1 int64, host memory): part p is rows
 * [part_offsets[p], part_offsets[p+1]). 1 <= n_parts <= HX_MAX_PARTS. Synchronises (the
 * offsets are read back to size the exchange).
 * Part function: h = fmix32((uint32)key) (murmur3 finaliser: h ^= h >> 16; h *= 0x85EBCA6B;
 * h ^= h >> 13; h *= 0xC2B2AE35; h ^= h >> 16), p = ((uint64)h * n_parts) >> 32 — keys of
 * one value always meet in one part, and the parts are independent of the hash tables'
 * bucket function.
 * Errors: HX_EINVAL (null argument, n_parts outside 1..HX_MAX_PARTS, key column not in t),
 * HX_EUNSUPPORTED (t not device resident), HX_ENOMEM / HX_ECUDA (allocation, launch). */
#define HX_MAX_PARTS 64
int hx_hash_partition(hx_ctx* ctx, const hx_table* t, int32_t key_col, int n_parts,
                      hx_table** out, int64_t* part_offsets);
/* The hash-routing exchange: part p of `parted` (from hx_hash_partition with n_parts ==
   nranks) goes to rank p; *out receives, in rank order, the rows every rank routed here — one
   grouped set of ncclSend/ncclRecv per column over NVLink after an ncclAllGather of the part
   sizes. Collective over the communicator. Without a communicator of > 1 ranks it returns a
   copy of part 0 (n_parts must be 1 then). Synchronises. Errors: HX_EINVAL (offsets that do
   not match the table, n_parts != the rank count), HX_ENCCL (a collective failed; message in
   hx_last_error), HX_ENOMEM / HX_ECUDA. *out is library-owned (hx_table_free). */
int hx_exchange_partitions(hx_ctx* ctx, const hx_table* parted, const int64_t* part_offsets,
                           int n_parts, hx_table** out);

/* ---- fused scan → filter → probe×k → aggregate (§8(a) a5, kernel K1) ----------------
 * PAPER.md:859-869 Listing 1 pipeline 9 (grid-stride unpack, predicate, thread-local
 * accumulator, neighbourhood reduce, leader atomic add to the pipeline state),
 * PAPER.md:919-926, 937-951 §4.1/Fig. 3 (GPU provider: grid-wide thread ids, worker-scoped
 * atomics), §6.1 (SSB query shapes: 1, 3, 3, 4 joins), PAPER.md:240-244,
 * 285-290 (fused pipelines, no materialisation).
 * For every row of `fact`: all `preds` (fact columns) must hold; then for each join in
 * array order the row's FK value is probed in hts[join_ht] (miss drops the row); the
 * measure is  a (HX_AGG_SUM), a*b (HX_AGG_SUM_MUL) or a-b (HX_AGG_SUM_SUB), formed in
 * int64; the group index is the mixed radix of the ranks of the joins listed in gdim_join
 * (first = most significant). SUM (int64, two's complement, exact) and COUNT are added
 * to the agg's group arrays. n_gdims == 0 gives one ungrouped total.
 * The result accumulates into a NEW hx_agg (zeroed on the device first). Asynchronous. */
enum { HX_AGG_SUM = 0, HX_AGG_SUM_MUL = 1, HX_AGG_SUM_SUB = 2 };
#define HX_MAX_PREDS 3
#define HX_MAX_JOINS 4
#define HX_MAX_GDIMS 3
#define HX_MAX_GROUPS (1 << 26)
typedef struct {
  int32_t n_preds;
  hx_pred preds[HX_MAX_PREDS];           /* on fact columns (col_id = fact column id)     */
  int32_t n_joins;
  int32_t join_fk_col[HX_MAX_JOINS];     /* fact FK column id of each join                */
  int32_t join_ht[HX_MAX_JOINS];         /* index into hts[]; probe order = array order   */
  int32_t agg_op;                        /* HX_AGG_*                                       */
  int32_t agg_a, agg_b;                  /* fact column ids of the measure operands        */
  int32_t n_gdims;
  int32_t gdim_join[HX_MAX_GDIMS];       /* joins whose ranks form the group key           */
} hx_query_shape;
typedef struct hx_agg hx_agg;
int hx_pipeline_probe_agg(hx_ctx* ctx, const hx_table* fact, const hx_query_shape* shape,
                          hx_ht* const* hts, int n_hts, hx_agg** out);
/* Accumulate another fact table (e.g. the next block of this GPU) into an existing agg. */
int hx_pipeline_probe_agg_into(hx_ctx* ctx, const hx_table* fact, const hx_query_shape* shape,
                               hx_ht* const* hts, int n_hts, hx_agg* agg);

/* ---- the router's dynamic load balancing across processes (§8(e) host-resident) --------
 * PAPER.md:469-473 §3.1 (the router routes block handles to consumers "while load-balancing"),
 * PAPER.md:1214-1233 §6.2 (SF1000 stays in CPU memory, streamed to the GPUs). One process per
 * GPU: the block counter is a POSIX shared-memory segment `name` ("/word") every process of
 * the node opens. hx_shared_router_next hands out the block indices 0 .. n_blocks-1, each
 * exactly once over all processes (atomic fetch-add), then -1. create = 1 creates the segment
 * (or re-initialises an existing one) with the counter at 0; create = 0 opens a segment created
 * for the same n_blocks (HX_EINVAL otherwise). reset puts the counter back to 0 (between runs,
 * by one process, while no other draws). close(unlink = 1) also removes the name. Host only. */
typedef struct hx_shared_router hx_shared_router;
int hx_shared_router_open(const char* name, int64_t n_blocks, int create, hx_shared_router** out);
int hx_shared_router_next(hx_shared_router* r, int64_t* block);
int hx_shared_router_reset(hx_shared_router* r);
int hx_shared_router_close(hx_shared_router* r, int unlink_name);
/* The host-resident pipeline fed by a shared router: `fact` is HX_PLACE_HOST_PINNED over the
   WHOLE table (every process maps the same pinned host memory); block b is rows
   [b * block_rows, min((b + 1) * block_rows, n_rows)). This GPU draws a block whenever one of
   its staging-ring slots is free (the host waits for that slot's previous K1), copies it H2D
   on the ctx's copy stream and runs K1 on it, accumulating into a NEW agg; blocks beyond the
   table end the loop. *n_blocks = blocks this process ran. Returns once the router is
   exhausted (the last K1s still run on the ctx stream; hx_merge_aggregates then merges over
   the ranks). Not capturable in a CUDA graph. */
int hx_pipeline_probe_agg_routed(hx_ctx* ctx, const hx_table* fact, const hx_query_shape* shape,
                                 hx_ht* const* hts, int n_hts, hx_shared_router* router,
                                 int64_t block_rows, hx_agg** out, int64_t* n_blocks);

/* ---- merge partial aggregates + finalize (§8(a) a6, a7) ----------------------------
 * PAPER.md:485-488 §3.1 (a local reduction per device, then the union router gathers the
 * partial results into one global aggregation), PAPER.md:927-936 (pipelines 8, 3 → 2).
 * With a communicator of > 1 ranks the per-GPU group arrays are summed with
 * ncclAllReduce (root < 0) or ncclReduce to `root` over NVLink; then the (merged) arrays
 * are copied to the host and finalised: groups with count 0 are dropped (a query without
 * GROUP BY always yields its one row), and each group index is decoded back to the
 * dictionary codes of its group columns (keys[i*n_gdims + g], in gdim order).
 * Writes at most `cap` rows; *n_rows = rows produced (HX_ECAPACITY if > cap, with
 * *n_rows set to the required count). Synchronises. Non-root ranks of a reduce get
 * *n_rows = 0. Returns HX_EDUPKEY / HX_EINVAL if a build it depends on failed. */
int hx_merge_aggregates(hx_ctx* ctx, hx_agg* agg, int root, int64_t* sums, int64_t* counts,
                        int32_t* keys, int64_t cap, int64_t* n_rows);
int hx_agg_free(hx_agg* agg);
/* The union router's group layout and the host finalize, callable without a GPU (host
   logic only; the multi-rank CPU tests use them with a gloo all-reduce in place of NCCL).
   hx_group_layout: a group of rank tuple (r_0 .. r_{n-1}) over n_gdims grouping dimensions
   with n_ranks[g] dense ranks each (>= 1) sits at index sum_g r_g * strides[g], strides[n-1]
   = 1, strides[g] = strides[g+1] * n_ranks[g+1]; *n_groups = prod n_ranks (1 for n_gdims 0).
   This is the layout K1 accumulates into (k1_prepare) and the merge reduces: {sums[n_groups],
   counts[n_groups]}, 2 * n_groups int64 per rank. HX_ECAPACITY above HX_MAX_GROUPS.
   hx_group_decode (a7): from merged sums/counts in that layout and each grouping dimension's
   rank -> code map (rank_to_code[g][r], caller-owned), writes the groups with count > 0 (an
   ungrouped query: its one row) in index order: keys[i * n_gdims + g], out_sums[i],
   out_counts[i]; at most `cap` rows; *n_rows = rows produced (HX_ECAPACITY if > cap). */
int hx_group_layout(int n_gdims, const int32_t* n_ranks, int64_t* strides, int64_t* n_groups);
int hx_group_decode(int n_gdims, const int32_t* n_ranks, const int32_t* const* rank_to_code,
                    const int64_t* sums, const int64_t* counts, int64_t n_groups, int32_t* keys,
                    int64_t* out_sums, int64_t* out_counts, int64_t cap, int64_t* n_rows);

/* ---- prepared plans and CUDA graphs (the native runtime around K1/K2) ----------------
 * PAPER.md:769-790 §4.1 (pipelines are generated and compiled once per query, then run),
 * PAPER.md:1043-1050 §4.3 (block arenas pre-allocated at initialisation: no allocation at
 * query time). A plan bundles one query's dimension builds (builds[j] builds the table
 * that shape->join_ht indexes: join_ht[j] is an index into builds[]), the fused pipeline
 * over `fact`, the union-router merge (NCCL allreduce of the partial group arrays when the
 * ctx has > 1 ranks) and the finalize step (a7: empty groups dropped, group codes decoded)
 * ON THE DEVICE, with the result copied into pinned host memory. hx_plan_create allocates
 * everything and runs the builds once, synchronously, to size the group arrays exactly;
 * hx_plan_enqueue is asynchronous, allocation-free and free of host synchronisation, so a
 * sequence of enqueues can be captured into a CUDA graph (hx_graph_*) and replayed. If the
 * dimensions change so that the group count differs from the plan's, the execution reports
 * HX_ECAPACITY (re-create the plan). The fact table and dims must outlive the plan. */
typedef struct {
  int32_t dim;                 /* index into the dims[] array of hx_plan_create   */
  int32_t key_col;
  int32_t n_preds;
  hx_pred preds[HX_MAX_PREDS];
  int32_t group_col;           /* -1: membership only                              */
  int32_t group_lo, group_hi;
} hx_build_spec;
typedef struct hx_plan hx_plan;
int hx_plan_create(hx_ctx* ctx, const hx_table* fact, hx_table* const* dims, int n_dims,
                   const hx_build_spec* builds, int n_builds, const hx_query_shape* shape,
                   hx_plan** out);
int hx_plan_enqueue(hx_ctx* ctx, hx_plan* plan);
/* Enqueue several plans as one step: every plan's builds first (on auxiliary streams, so
   they overlap the pipelines of the plans before them), then each plan's pipeline, merge and
   finalize in order, each waiting only for its own builds. Same results as n x
   hx_plan_enqueue; capturable. */
int hx_plans_enqueue(hx_ctx* ctx, hx_plan* const* plans, int n);
/* Waits for the last enqueued execution; rows as hx_merge_aggregates (group-index order). */
int hx_plan_result(hx_plan* plan, int64_t* sums, int64_t* counts, int32_t* keys, int64_t cap,
                   int64_t* n_rows);
/* K1 device time of the last execution (CUDA events around the launch) and its
   algorithmic bytes (rows x 4 B x distinct fact columns). Waits for the execution. */
int hx_plan_k1_time(hx_plan* plan, float* ms, int64_t* bytes);
/* Device time from the start of `first`'s K1 to the end of `last`'s K1 in their last
   executions (meaningful when both ran in one hx_plans_enqueue / graph launch, `first` before
   `last`): the span of the pipelines, including the gaps between them. Waits for `last`. */
int hx_plan_k1_span(hx_plan* first, hx_plan* last, float* ms);
int hx_plan_info(hx_plan* plan, int64_t* n_groups, int* n_gdims);
int hx_plan_free(hx_plan* plan);
typedef struct hx_graph hx_graph;
/* Capture every hx_plan_enqueue between begin and end on the ctx stream into a graph. */
int hx_graph_begin(hx_ctx* ctx);
int hx_graph_end(hx_ctx* ctx, hx_graph** out);
int hx_graph_launch(hx_ctx* ctx, hx_graph* graph);
int hx_graph_free(hx_graph* graph);

/* ---- measurement ------------------------------------------------------------------
 * When enabled, CUDA events bracket every K1 launch on the ctx stream. hx_profile_read
 * synchronises and returns the summed K1 device time (ms), launch count and algorithmic
 * bytes (rows x 4 B x distinct fact columns the shape references), then resets if asked. */
int hx_profile_enable(hx_ctx* ctx, int on);
int hx_profile_read(hx_ctx* ctx, double* k1_ms, int64_t* k1_launches, int64_t* k1_bytes,
                    int reset);
/* Counters since the last reset: kernels libhx launched, bytes it copied host->device
   (hx_load_columns from host memory) and device->host (hx_merge_aggregates, hx_ht_info). */
int hx_stats(hx_ctx* ctx, int64_t* launches, int64_t* h2d_bytes, int64_t* d2h_bytes, int reset);

#ifdef __cplusplus
}
#endif
#endif /* HX_H */

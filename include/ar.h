/*
 * ar.h -- C ABI of the B200-native Approximate & Refine (A&R) hot path over
 * bitwise-distributed (BWD) integer columns.
 *
 * Method: H. Pirk, S. Manegold, M. Kersten, "Waste Not... Efficient
 * Co-Processing of Relational Data", ICDE 2014.  Citations "PAPER.md:<line>"
 * refer to the text of that paper; "SURVEY s8" to /root/repo/SURVEY.md s8 (the
 * hot-path scope table), "DESIGN" to /root/repo/DESIGN.md.
 *
 * Conventions (all calls):
 *  - Plain pointers and sizes only.  A "device pointer" is CUDA device memory
 *    (e.g. a torch CUDA tensor's data_ptr); a "host-pinned pointer" is page-
 *    locked host memory (cudaHostAlloc / torch pin_memory) the GPU reads over
 *    the host link.  `stream` is a cudaStream_t passed as void*.
 *  - Every call that takes a stream is asynchronous on it, except
 *    ar_decompose_plan (documented below).  Results that live in device memory
 *    (counts, sums) are valid once the stream reaches that point.
 *  - The library never allocates device memory: the caller owns every buffer
 *    and workspace.  Handles (ar_column, ar_dist) are small host objects.
 *  - No call aborts or throws.  Each returns an ar_status; on failure
 *    ar_last_error() (thread-local) describes the cause.
 *  - Values are uint32 (signed callers map v -> v ^ 0x80000000).
 *    Positions are uint32 row indices local to the column (a shard), counts
 *    and sums are int64.  There is no floating point anywhere on the path.
 */
#ifndef AR_H
#define AR_H

#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef enum {
    AR_OK = 0,
    AR_ERR_INVALID = 1,      /* bad argument (null pointer, bad width, mismatched columns) */
    AR_ERR_RANGE = 2,        /* a buffer / workspace / capacity is too small, or overflow possible */
    AR_ERR_CUDA = 3,         /* CUDA runtime error (launch failure, bad pointer, no device) */
    AR_ERR_NCCL = 4,         /* NCCL error in an ar_dist_* call */
    AR_ERR_UNSUPPORTED = 5   /* valid but outside what this build implements (e.g. too many planes) */
} ar_status;

/* Where a part of a column lives. */
typedef enum {
    AR_LOC_DEVICE = 0,       /* HBM of the current device */
    AR_LOC_HOST_PINNED = 1   /* pinned host memory, read by kernels over the host link (zero-copy) */
} ar_loc;

/*
 * Physical layout of the major (approximation) part.  The paper leaves the
 * physical representation inside a bitwise partition open (PAPER.md:219-221,
 * s II-A); this build offers two (DESIGN "Data layout in HBM"):
 *  AR_LAYOUT_SLICED: rows are grouped in blocks of 32; block b stores w_major
 *    uint32 words, word j holding bit j of the majors of rows 32b..32b+31
 *    (bit l of the word = row 32b+l).  Scan-optimised: a range test costs a
 *    few bitwise ops per bit plane per 32 rows.  Required for ar_approx_select.
 *  AR_LAYOUT_PACKED: LSB-first bitstream, row i occupies bits [i*w, i*w+w) of
 *    the little-endian uint32 word stream.  Gather-optimised (one sector per
 *    value): use it for columns that are only aggregated (l_extendedprice).
 * Residuals (minor bits) use the same two layouts with width k: the plan picks
 * SLICED for k <= 8 (a block's k residual planes are k*4 <= 32 bytes, one
 * sector, so a gather costs the same as PACKED, and the one-pass kernel can
 * evaluate exact predicates on major + residual planes together) and PACKED
 * for wider residuals (a gather reads one sector instead of k*4 bytes).
 */
typedef enum {
    AR_LAYOUT_SLICED = 0,
    AR_LAYOUT_PACKED = 1
} ar_layout;

#define AR_MAX_PRED 8          /* predicates per conjunctive select            */
#define AR_MAX_AGG 2           /* factors of the SUM product    */
#define AR_MAX_GROUPS 4096     /* groups of ar_refine_group_sum (shared-memory group table) */
#define AR_MAX_PLANES 64       /* sum of w_major over the predicates of a scan */

/*
 * Decomposition descriptor, the "extended BAT" metadata of PAPER.md:908-916
 * (s V-C): number and significance of the bits on each device (which also
 * encodes the error of the approximation) and the prefix-compression base.
 * Filled by ar_decompose_plan; plain old data, caller-owned.
 */
typedef struct {
    int64_t n;                 /* rows                                                    */
    int32_t major_bits;        /* M of bwdecompose(A, M); k = 32 - M   */
    int32_t k;                 /* residual (minor) bits, 0..31                            */
    int32_t w_major;           /* stored major width after leading-zero removal, 0..M     */
    int32_t major_layout;      /* ar_layout of the major part                             */
    int32_t residual_loc;      /* ar_loc of the residual part                             */
    uint32_t base;             /* prefix base b: value = ((major << k) | residual) + b    */
    uint64_t major_bytes;      /* bytes the major buffer must provide                     */
    uint64_t residual_bytes;   /* bytes the residual buffer must provide (0 if k == 0)    */
    int32_t major_loc;         /* ar_loc of the major part: AR_LOC_DEVICE (set by the plan);
                                  a caller may set AR_LOC_HOST_PINNED before ar_decompose /
                                  ar_column_wrap for a column that is only gathered (an
                                  aggregate column): kernels then read it over the host link.
                                  Predicate columns must keep their majors on the device.  */
    int32_t residual_layout;   /* ar_layout of the residual part (set by the plan, see above) */
    int32_t value_signed;      /* 1: values are int32 (two's complement).  The column is
                                  decomposed in the order-preserving key domain
                                  d = v ^ 0x80000000: u = d - base, and
                                  predicate bounds of ar_pred are int32 bit patterns that
                                  the library maps the same way.  0: uint32 values, d = v. */
    int32_t residual_split;    /* h, 0 <= h < k: 0 = one SLICED / PACKED residual part.  h > 0
                                  (SLICED residuals, k <= 8) = the split layout: per
                                  8192-row super-group (256 blocks of 32 rows) first the h
                                  high residual planes of its 256 blocks (block-major, h
                                  words per block: planes k-h .. k-1), then the k - h low
                                  planes (k - h words per block: planes 0 .. k-h-1); so
                                  the high bits of a block can be read without its low
                                  bits (progressive refinement, DESIGN s6.3d).
                                  residual_bytes = ceil(n / 8192) * 1024 * k.            */
} ar_column_desc;

typedef struct ar_column ar_column;   /* opaque: desc + part pointers (host object) */

/* One conjunct lo <= value <= hi (inclusive, exact bounds; lo > hi selects nothing).
 * Operators normalise to this form: <x -> [0,x-1], >x -> [x+1,2^32-1],
 * ==x -> [x,x], between a and b -> [a,b].  On a signed column lo and hi are
 * int32 bit patterns compared in signed order. */
typedef struct {
    const ar_column* col;
    uint32_t lo;
    uint32_t hi;
} ar_pred;

/*
 * Candidate relation: the output of the approximate selection, a superset of
 * the exact result (Fig. 4 "sigma(Approx A <= 4)" yields
 * (ID, Approx A) pairs).  Entry j (0 <= j < *count) is
 *   pos[j]: the row position (ascending in j: the compaction is stable, so
 *           every refine join is a positional "invisible" join)
 *   aux[j]: bit 31 = definite (the row's whole bucket satisfies every
 *           predicate, so it needs no residual); bits 0..30 = the
 *           approximation tuple, i.e. the predicate columns' majors
 *           concatenated LSB-first in predicate order, present iff
 *           appr_bits > 0 (ar_approx_select flag AR_SELECT_CARRY_APPR).
 * pos, aux and count are caller-owned device buffers of `capacity` entries
 * (capacity >= n is always sufficient).
 */
typedef struct {
    uint32_t* pos;
    uint32_t* aux;
    int64_t* count;            /* device int64 */
    int64_t capacity;
    int32_t appr_bits;         /* set by ar_approx_select */
    int32_t reserved;
} ar_cands;

#define AR_AUX_DEFINITE 0x80000000u

/* Refined positions: ascending row positions of the exact result. Caller-owned device buffers. */
typedef struct {
    uint32_t* pos;
    int64_t* count;            /* device int64 */
    int64_t capacity;
} ar_positions;

/* ---------------------------------------------------------------- errors */

const char* ar_status_str(ar_status s);
const char* ar_last_error(void);     /* thread-local detail of the last failure */
const char* ar_version(void);
/* Name of the main kernel the calling thread's last ar_select_refine_sum,
 * ar_approx_select or ar_refine_sum launched: "fused_rl_kernel" (result-ring
 * one-pass kernel), "fused_kernel" (general one-pass kernel),
 * "select_rr_kernel" / "select_tile_kernel" (ordered select),
 * "refine_sum_sliced_kernel" /
 * "refine_sum_kernel" (refine + SUM), "" (none: empty input or an error).
 * Static storage; for tests and benchmarks that must know which path ran. */
const char* ar_last_scan_kernel(void);

/* --------------------------------------------------- a1: decomposition */

/* Workspace (device memory, >= this many bytes) for ar_decompose_plan. */
size_t ar_decompose_ws_bytes(void);

/*
 * Plan a BWD decomposition of column `col` (n uint32 values, device pointer or
 * host-pinned pointer) into `major_bits` major bits and k = 32 - major_bits
 * residual bits, the split of bwdecompose(A, bits) (s V-A).
 * Computes w_major = bit length of max((d - base) >> k) (leading zeros are
 * removed) with a min/max-reduction kernel, then the byte sizes
 * of both parts.  SYNCHRONISES `stream` once (the sizing pass).
 * flags: AR_DECOMPOSE_SIGNED   -- int32 values (desc->value_signed);
 *        AR_DECOMPOSE_BASE_MIN -- prefix compression with base = min(d) (the
 *          frame of reference; `base` is ignored);
 *        AR_DECOMPOSE_SPLIT(h) -- 1 <= h < k <= 8: the residual in the split
 *          layout (desc->residual_split = h; AR_ERR_INVALID otherwise).
 * `base` is in the key domain d (d = v ^ 0x80000000 for signed columns).
 * Errors: AR_ERR_INVALID if col == NULL && n > 0, n < 0, n >= 2^32,
 * major_bits outside [1,32], bad layout / location / flags, ws too small or
 * desc NULL; AR_ERR_RANGE if base > min(d) (a value below the base).
 */
#define AR_DECOMPOSE_SIGNED 1
#define AR_DECOMPOSE_BASE_MIN 2
#define AR_DECOMPOSE_SPLIT(h) (((h) & 31) << 8)
ar_status ar_decompose_plan(const uint32_t* col, int64_t n, int32_t major_bits,
                            int32_t major_layout, int32_t residual_loc, uint32_t base, int32_t flags,
                            void* ws, size_t ws_bytes, ar_column_desc* desc, void* stream);

/*
 * bwdecompose (the split of Fig. 2):
 * decompose and pack `col` per `desc`: the major part is written to
 * `major_buf` (device memory, desc->major_bytes bytes, padding zeroed) and the
 * residual part to `residual_buf` (device memory, or pinned host memory when
 * desc->residual_loc == AR_LOC_HOST_PINNED; desc->residual_bytes bytes).
 * The buffers must outlive the returned handle, which is freed with
 * ar_column_free.  Values larger than the plan's maximum are not detected:
 * plan and decompose the same column.
 * Errors: AR_ERR_INVALID (null pointers, bad desc), AR_ERR_RANGE (buffer too
 * small), AR_ERR_CUDA (launch failure or unmappable host pointer).
 */
ar_status ar_decompose(const uint32_t* col, const ar_column_desc* desc,
                       void* major_buf, uint64_t major_buf_bytes,
                       void* residual_buf, uint64_t residual_buf_bytes,
                       void* stream, ar_column** out);

/*
 * Widen a planned descriptor to a stored major width w_major >= desc->w_major
 * (<= major_bits) and recompute major_bytes.  Row shards of one table are
 * planned separately but must share one bucket geometry and layout: the
 * caller takes the global w_M = max over shards (an allreduce-MAX, SURVEY
 * s8(e)) and widens every shard's descriptor before ar_decompose.  Host only.
 * Errors: AR_ERR_INVALID (bad desc), AR_ERR_RANGE (w_major outside that range).
 */
ar_status ar_decompose_set_width(ar_column_desc* desc, int32_t w_major);

/* Wrap already-decomposed parts (e.g. a copy of the buffers ar_decompose wrote) in a new handle.
 * Both buffers must be 16-B aligned and hold at least the bytes the descriptor's
 * geometry needs (n, w_major, k and the layouts; ar_decompose_plan's sizes).
 * Errors: AR_ERR_INVALID (bad desc, null or misaligned buffer), AR_ERR_RANGE
 * (major_bytes / residual_bytes below that size), AR_ERR_CUDA (a host-resident
 * part that is not mapped pinned memory). */
ar_status ar_column_wrap(const ar_column_desc* desc, const void* major_buf, const void* residual_buf,
                         ar_column** out);
ar_status ar_column_get_desc(const ar_column* col, ar_column_desc* desc);
void ar_column_free(ar_column* col);

/* ------------------------------------- a2 + a3: approximate selection */

#define AR_SELECT_CARRY_APPR 1   /* write the approximation tuple into aux bits 0..30 */

/* Workspace (device memory) for ar_approx_select over n rows. */
size_t ar_select_ws_bytes(int64_t n);

/*
 * Approximate selection (s IV-B) of the conjunction of
 * `npred` predicates over columns of equal n (all major parts AR_LAYOUT_SLICED
 * in device memory).  Host side (a2): each exact [lo, hi] is relaxed to the
 * major ranges cand = [lo>>k, hi>>k] (bucket intersects [lo,hi]) and
 * def = [ceil(lo/2^k), floor((hi+1)/2^k) - 1] (bucket inside [lo,hi]), with
 * b = base subtracted first (DESIGN "Readings").  Device side
 * (a3): one pass over the packed majors with stable compaction into
 * out->pos / out->aux / *out->count: per tile a popc + block scan, and either
 * (select_rr_kernel, the default for wide sparse scans) the tile's entries
 * written once at the offset a decoupled look-back over the per-tile counts
 * gives, or (select_tile_kernel) tile slices in the workspace that one
 * compaction launch places at the prefix of the earlier tiles' counts.  The
 * workspace holds the per-tile counts / status words and the slices; the
 * one-kernel select launches cooperatively (AR_ERR_CUDA if its grid cannot be
 * co-resident).  At least one predicate is required (a
 * scan needs a column; [0, 2^32 - 1] keeps every row).  A predicate with
 * lo > hi makes the result empty (AR_OK).
 * Errors: AR_ERR_INVALID (npred < 1 or > AR_MAX_PRED, null / mismatched columns,
 * non-SLICED or host-resident majors), AR_ERR_RANGE (capacity < n, ws too
 * small, AR_SELECT_CARRY_APPR with sum of w_major > 31), AR_ERR_UNSUPPORTED
 * (sum of w_major > AR_MAX_PLANES).
 */
ar_status ar_approx_select(const ar_pred* preds, int32_t npred, int32_t flags, ar_cands* out,
                           void* ws, size_t ws_bytes, void* stream);

/* ----------------------------------------------------- a5: refinement */

/* Workspace (device memory) for ar_refine over up to `capacity` candidates. */
size_t ar_refine_ws_bytes(int64_t capacity);

/*
 * Selection refinement (Algorithm 2 SELECTREFINE):
 * for every candidate in `in` (ascending), definite candidates are kept
 * without touching residuals; the others are joined positionally with the
 * residual of every predicate column with k > 0 (device or host-pinned), the
 * exact value is rebuilt by bitwise concatenation ((major << k) | residual) +
 * base, and the exact predicate re-evaluated.  Output: ascending positions of
 * the exact result (stable compaction) and its count.  `preds` must be the
 * same list (same order) given to the ar_approx_select that produced `in`.
 * Errors: AR_ERR_INVALID (mismatch with in->appr_bits, null pointers),
 * AR_ERR_RANGE (out->capacity < in->capacity, ws too small).
 */
ar_status ar_refine(const ar_cands* in, const ar_pred* preds, int32_t npred, ar_positions* out,
                    void* ws, size_t ws_bytes, void* stream);

/* ----------------------------------------------------- a6: aggregation */

/*
 * SUM over the positions of `pos` of prod_c value_c(p), c < ncols (ncols in
 * {1, 2}), exact in int64 (SUM(refine), Fig. 3 / Fig. 7, PAPER.md:884-889;
 * destructive distributivity, is why the exact values are
 * rebuilt before multiplying).  Result written to *out_sum_dev (device int64).
 * Errors: AR_ERR_INVALID (ncols not in {1,2}, null pointers, column shorter
 * than a position), AR_ERR_RANGE if sum of (w_major + k) + ceil(log2 n) > 63
 * (the exact sum could overflow int64).
 */
ar_status ar_sum(const ar_positions* pos, const ar_column* const* cols, int32_t ncols,
                 int64_t* out_sum_dev, void* stream);

/*
 * Approximate SUM (bwd.sumapproximate of Fig. 7): the
 * approximate query answer from the approximation subplan alone, before any
 * residual is read, as strict error bounds
 * (PAPER.md:375-382).  `in` is the output of ar_approx_select; the exact
 * result R satisfies definite <= R <= candidates, and a value with major m
 * lies in its bucket [b + m 2^k, b + m 2^k + 2^k - 1] (clamped to 2^32 - 1).
 * Reads only the major parts of `cols`.  Writes device int64[4]:
 *   out4[0] = sum over definite candidates of prod_c bucket_min_c  (<= SUM(R))
 *   out4[1] = sum over all candidates of prod_c bucket_max_c       (>= SUM(R))
 *   out4[2] = |definite| (<= |R|),  out4[3] = |candidates| (>= |R|)
 * ncols in [0, 2] (0: COUNT bounds only, out4[0..1] = 0).
 * Errors: AR_ERR_INVALID (null pointers, ncols > 2), AR_ERR_RANGE as ar_sum.
 */
ar_status ar_sum_approximate(const ar_cands* in, const ar_column* const* cols, int32_t ncols,
                             int64_t* out4_dev, void* stream);

/*
 * MIN / MAX over the exact result (s IV-F, Fig. 6):
 * select min(Y) / max(Y) from R where <preds>, from the candidate relation
 * `in` of ar_approx_select over the same `preds`.  "The result of the
 * approximation of a minimum has to assuredly include the tuple ID of the
 * actual minimum.  To guarantee this, the error bounds of the applied
 * selections are propagated to the aggregation": with Y's
 * majors m (key domain), a definite candidate is certainly in R, so
 * only candidates with m <= min over definite candidates (MIN; m >= max over
 * definite candidates for MAX; every candidate when none is definite) can hold
 * the answer.  Those are refined -- the exact predicates (Alg. 2), then Y's
 * exact value from its residual ("a join of the candidate set with the input
 * residuals and the calculation of the minimum").
 * `col` is any column of the table (it may be a predicate column; its major
 * is then taken from the carried approximation).  Writes device int64[7]:
 *   out7[0] = the exact MIN / MAX (a signed column's value as int32; 0 if out7[1] == 0)
 *   out7[1] = refined rows that satisfy the predicates (>= 1 iff R is not empty)
 *   out7[2], out7[3] = approximate answer before refinement, lower / upper bound
 *             (bucket ends; 0, 0 without candidates):
 *             MIN in [bmin(min_C m), D ? bmax(min_D m) : bmax(max_C m)]
 *             MAX in [D ? bmin(max_D m) : bmin(min_C m), bmax(max_C m)]
 *   out7[4] = candidates refined, out7[5] = |definite|, out7[6] = |candidates|
 * `ws` is a caller-owned device workspace of ar_minmax_ws_bytes(in->capacity)
 * bytes (initialised by the call; it keeps each candidate's Y major between
 * the approximate and the refine pass).  Four kernel launches on `stream`.
 * Errors: AR_ERR_INVALID (null pointers, bad mode, predicates that do not
 * match the candidate relation), AR_ERR_RANGE (workspace too small).
 */
#define AR_MIN 0
#define AR_MAX 1
size_t ar_minmax_ws_bytes(int64_t capacity);
ar_status ar_minmax(const ar_cands* in, const ar_pred* preds, int32_t npred, const ar_column* col, int32_t mode,
                    int64_t* out7_dev, void* ws, size_t ws_bytes, void* stream);

/*
 * Grouped COUNT / SUM over the exact result (s IV-E/F):
 *   select key, count(*), sum(prod_c cols[c]) from R where <preds> group by key
 * e.g. Fig. 4 "select count(*) from R where A<5 groupby B".
 * The paper keeps low-cardinality group columns whole on the GPU
 * (PAPER.md:762-771), so `key` must be a k = 0 unsigned column: its values are
 * the group ids (no hashing), the approximate pre-grouping is exact, and only
 * the selection's false positives are eliminated (Alg. 2 on the candidate
 * relation `in` of ar_approx_select over the same `preds`).  Factors as in
 * ar_refine_sum (ncols in [0, 2]).  Writes device int64[2 * ngroups]:
 *   out[g] = SUM over R with key g (0 when ncols == 0), out[ngroups + g] = COUNT.
 * Errors: AR_ERR_INVALID (null pointers, ngroups outside [1, AR_MAX_GROUPS]),
 * AR_ERR_UNSUPPORTED (decomposed or signed key), AR_ERR_RANGE (the key's
 * descriptor admits values >= ngroups: base + 2^w_major - 1 must be < ngroups;
 * or a SUM that could overflow, as ar_sum).
 */
ar_status ar_refine_group_sum(const ar_cands* in, const ar_pred* preds, int32_t npred, const ar_column* key,
                              const ar_column* const* cols, int32_t ncols, int32_t ngroups, int64_t* out_dev,
                              void* stream);

/*
 * The approximation group operator (s IV-E): "hash-based
 * grouping to assign group IDs to unique values", the output positionally
 * aligned with the input.  For each row j < *rows->count at position
 * rows->pos[j] (e.g. the candidate relation: {cands.pos, cands.count,
 * cands.capacity}), the grouping value is
 *   AR_GROUP_APPROX: the approximate value base + (major << k) -- the bucket
 *                    minimum, a pre-grouping on approximate values (for a k = 0
 *                    key the exact value);
 *   AR_GROUP_EXACT : the exact value ((major << k) | residual) + base (reads the
 *                    residual, device or host-pinned).
 * Equal values get equal ids; ids are dense (0 .. #groups - 1) in order of
 * first insertion into a hash table (open addressing) in the caller's
 * `table` (ar_group_table_bytes(table_slots) bytes of device memory; table_slots
 * a power of two >= 2 * max_groups; cleared by the call), so the id of a value
 * depends on scheduling while the value of every id is written to
 * group_keys_out[id] (device, max_groups entries; a signed column's int32 bits).
 * gids_out (device, rows->capacity entries) receives the ids; *ngroups_dev
 * (device int64) the number of distinct values; *overflow_dev (device u32) bit 0
 * if there were more than max_groups values (ids are then clamped and the
 * grouping is invalid), bit 1 if the table filled up.  One launch + memsets.
 * Errors: AR_ERR_INVALID (null pointers, bad mode), AR_ERR_RANGE (table_slots).
 */
#define AR_GROUP_APPROX 0
#define AR_GROUP_EXACT 1
size_t ar_group_table_bytes(int64_t table_slots);
ar_status ar_group_ids(const ar_positions* rows, const ar_column* key, int32_t mode, void* table, int64_t table_slots,
                       int32_t max_groups, uint32_t* gids_out, uint32_t* group_keys_out, int64_t* ngroups_dev,
                       uint32_t* overflow_dev, void* stream);

/*
 * Grouped COUNT / SUM over the exact result by the ids of the approximation
 * group operator (s IV-E/F): as ar_refine_group_sum, but the group of
 * candidate j is gids[j] (device, aligned with the candidate relation `in`,
 * e.g. ar_group_ids over {in->pos, in->count}; values < ngroups).  The
 * refinement eliminates the selection's false positives
 * before anything is aggregated, so a group whose candidates were all false
 * positives ends with count 0.  Writes device int64[2 * ngroups]: out[g] = SUM
 * of prod_c cols[c] over R in group g, out[ngroups + g] = COUNT.
 * Errors: AR_ERR_INVALID (null pointers, ngroups outside [1, AR_MAX_GROUPS]),
 * otherwise as ar_refine_sum.
 */
ar_status ar_refine_group_sum_ids(const ar_cands* in, const ar_pred* preds, int32_t npred, const uint32_t* gids,
                                  int32_t ngroups, const ar_column* const* cols, int32_t ncols, int64_t* out_dev,
                                  void* stream);

/*
 * Positional projection of one column at the rows of `pos` (the invisible /
 * positional join of the A&R plan: bwd.leftjoinapproximate and
 * bwd.leftjoinrefine of Fig. 7; positional joins
 * PAPER.md:537-549).  out_values[j] (device, capacity >= pos->capacity) =
 *   AR_PROJECT_EXACT : the exact value ((major << k) | residual) + base
 *                      (reads the residual, device or host-pinned)
 *   AR_PROJECT_APPROX: the approximation base + (major << k), the bucket
 *                      minimum; the exact value lies in [out, out + 2^k - 1].
 * for j < *pos->count.  Candidate positions are projected by passing an
 * ar_positions {cands.pos, cands.count, cands.capacity}.
 * Errors: AR_ERR_INVALID (null pointers, bad mode).
 */
#define AR_PROJECT_APPROX 0
#define AR_PROJECT_EXACT 1
ar_status ar_project(const ar_positions* pos, const ar_column* col, int32_t mode, uint32_t* out_values,
                     void* stream);

/*
 * Fused refine + SUM (a5 + a6; SUM(refine) of Fig. 3 / Fig. 7, PAPER.md:333-359,
 * 884-889, over Alg. 2's refinement): the refinement of ar_refine without
 * materialising positions, then the product SUM of ar_sum over the refined
 * rows.  Aggregated columns that are also predicate columns reuse the carried
 * approximation (and residual) instead of re-gathering.  Writes
 * *out_sum_dev and *out_count_dev (refined row count); either may be NULL.
 * Errors: as ar_refine and ar_sum.
 */
ar_status ar_refine_sum(const ar_cands* in, const ar_pred* preds, int32_t npred,
                        const ar_column* const* cols, int32_t ncols,
                        int64_t* out_sum_dev, int64_t* out_count_dev, void* stream);

/*
 * One-pass A&R (a3 + a5 + a6 fused, SURVEY s8(a) "Fusion note"): scan the
 * majors, decide candidate / definite per row, refine the non-definite
 * candidates inline from the residuals and add the product SUM of `cols` over
 * the exact result.  No candidate list is materialised.  out_dev[0] = SUM,
 * out_dev[1] = |exact result|, out_dev[2] = |candidates|, out_dev[3] =
 * |definite| (device int64[4]; out_dev[2..3] give the approximate COUNT
 * interval [#definite, #candidates] before refinement).
 * Returns results identical to ar_approx_select -> ar_refine_sum.
 * Errors: as ar_approx_select and ar_sum (ncols may be 0: COUNT only).
 */
ar_status ar_select_refine_sum(const ar_pred* preds, int32_t npred,
                               const ar_column* const* cols, int32_t ncols,
                               int64_t* out_dev, void* stream);

/*
 * The same one-pass query for back-to-back query streams (and CUDA graphs):
 * with a workspace the call is a single kernel launch -- out_dev is written,
 * not accumulated, so no memset precedes it -- and may use programmatic
 * dependent launch so that its prologue and first tile loads overlap the tail
 * of the preceding kernel in the stream.
 *   ws        device memory of >= ar_select_refine_sum_ws_bytes() bytes whose
 *             first 4 bytes are zero before the first call (e.g. cudaMemset
 *             once); every call leaves them zero.  One workspace per stream:
 *             calls sharing it must be stream-ordered.  NULL = as
 *             ar_select_refine_sum (flags must be 0).
 *   flags     AR_SRS_PDL: launch as a programmatic dependent of the previous
 *             kernel; inputs are read after it completes, out_dev is written
 *             after it completes.
 *             AR_SRS_PDL_EARLY_READ: as AR_SRS_PDL, but the column parts are
 *             read while the previous kernel may still run -- the caller
 *             guarantees that kernel does not write them (e.g. the previous
 *             call of a query stream over immutable, already-decomposed columns).
 * Results are identical to ar_select_refine_sum.
 * Errors: as ar_select_refine_sum; AR_ERR_RANGE (ws_bytes too small);
 * AR_ERR_INVALID (unknown flags, or flags without a workspace).
 */
#define AR_SRS_PDL 1
#define AR_SRS_PDL_EARLY_READ 2
size_t ar_select_refine_sum_ws_bytes(void);
ar_status ar_select_refine_sum_ws(const ar_pred* preds, int32_t npred,
                                  const ar_column* const* cols, int32_t ncols, int32_t flags,
                                  int64_t* out_dev, void* ws, size_t ws_bytes, void* stream);

/* -------------------------------- a4: row-sharded multi-GPU exchange */
/* Not in the paper, which runs one query per GPU: the build
 * shards rows across GPUs; rows are independent, so only counts
 * (for global result offsets) and the SUM are exchanged. */

typedef struct ar_dist ar_dist;

/* Size of the opaque NCCL unique id blob (rank 0 creates it; the caller broadcasts it). */
size_t ar_dist_unique_id_bytes(void);
ar_status ar_dist_get_unique_id(void* id_out);

/* One communicator per rank over the current device (NCCL over NVLink / NVSwitch). */
ar_status ar_dist_init(ar_dist** d, const void* unique_id, int32_t rank, int32_t world);

/*
 * Count exchange: ncclAllGather of each rank's *local_count_dev into
 * all_counts_dev[world], then *global_offset_dev = sum of the counts of lower
 * ranks (the rank's slice of the concatenated, globally ordered result starts
 * there; global position = shard_row_base + local position).  Device pointers.
 */
ar_status ar_dist_offsets(ar_dist* d, const int64_t* local_count_dev, int64_t* all_counts_dev,
                          int64_t* global_offset_dev, void* stream);

/* In-place ncclAllReduce(int64, sum) of `n` device int64 values (the Q6 SUM and counts). */
ar_status ar_dist_sum(ar_dist* d, int64_t* values_dev, int32_t n, void* stream);

/*
 * Shard geometry (host only, no device work): rank `rank` of
 * `world` owns the contiguous rows [*row0, *row0 + *rows) of an n-row table.
 * Every shard but the last holds ceil(n / world) rounded up to a multiple of
 * AR_SHARD_ALIGN_ROWS rows, so each shard's SLICED / PACKED bitstreams start
 * 16-B aligned; the last shard is ragged and trailing shards may be empty.
 * Errors: AR_ERR_INVALID (n < 0, rank outside [0, world), null outputs).
 */
#define AR_SHARD_ALIGN_ROWS 128
ar_status ar_dist_shard_range(int64_t n, int32_t world, int32_t rank, int64_t* row0, int64_t* rows);

/*
 * The prefix step of ar_dist_offsets on its own (device, one launch on
 * `stream`): from the gathered counts all_counts_dev[world] of every rank,
 * *global_offset_dev = sum of the counts of ranks < rank and, if total_dev is
 * not NULL, *total_dev = sum of all counts.  ar_dist_offsets = ncclAllGather +
 * this kernel.  Errors: AR_ERR_INVALID (null pointers, rank outside [0, world)).
 */
ar_status ar_dist_exclusive_offsets(const int64_t* all_counts_dev, int32_t world, int32_t rank,
                                    int64_t* global_offset_dev, int64_t* total_dev, void* stream);

/*
 * Place a rank's refined positions in the concatenated, globally ordered
 * result (device, one launch): out_global[*global_offset_dev + j] =
 * row0 + local->pos[j] for j < *local->count (int64 global row positions;
 * row0 from ar_dist_shard_range).  out_global is a caller-owned device buffer
 * of out_capacity entries -- the whole result on one device, or a rank's view
 * of a distributed one.  If the slice does not fit, nothing is written and
 * *overflow_dev (device u32, caller-zeroed) gets bit 0 set.
 * Errors: AR_ERR_INVALID (null pointers, row0 < 0 or out_capacity < 0).
 */
ar_status ar_dist_concat_positions(const ar_positions* local, int64_t row0, const int64_t* global_offset_dev,
                                   int64_t* out_global, int64_t out_capacity, uint32_t* overflow_dev, void* stream);

void ar_dist_free(ar_dist* d);

#ifdef __cplusplus
}
#endif
#endif /* AR_H */

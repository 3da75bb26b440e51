// kernels.cuh -- parameter blocks and launchers shared by api.cu and the kernel files.
#pragma once
#include "common.cuh"

namespace ard {

// Approximate-select predicate, already relaxed to the major domain (step a2).
struct SelPred {
    const uint32_t* planes;   // SLICED major part (device)
    uint32_t w;               // planes per 32-row block (w_major)
    uint32_t mode;            // 0: k == 0 (def == cand); 1: approximate with a definite range; 2: no definite range
    uint32_t clo, chi;        // candidate major range
    uint32_t dlo, dhi;        // definite major range (mode 1)
    uint32_t soff;            // word offset of this predicate's planes inside one pipeline stage
    uint32_t ashift;          // bit offset of this major inside the approximation word
    // refine-side data, used by the fused kernel
    const uint32_t* residual; // PACKED width k (device or host-mapped), null if k == 0
    uint32_t k, base, lo, hi; // exact predicate on v = ((m << k) | r) + base
    uint32_t rlayout;         // residual layout (ar_layout)
    uint32_t res_stream;      // fused kernel: residual tile streamed into the stage (device-resident residuals)
    uint32_t res_soff;        // word offset of the streamed residual tile inside a stage
    uint32_t res_host;        // residual in pinned host memory (read over the host link)
    uint32_t res_hint;        // gathered-residual kernel: use the .L2::64B prefetch-size hint
    uint32_t rsplit;          // split residual layout: h high planes stored apart (0: not split)
    // split residual with its high planes streamed (result-ring kernel): the fine buckets
    // (u >> (k - h)) of the exact bounds and the low k - h bits of the bounds, u = v - base
    uint32_t sflo, sfhi, sllo, slhi;
    uint32_t scor;            // check-code bits forced on every undecided row (edge cases of the pmh encoding)
};

// Aggregate factor of the SUM product.
struct AggCol {
    const uint32_t* major;
    const uint32_t* residual;
    uint32_t w, k, layout, base, rlayout;
    uint32_t flip;            // 0x80000000 for a signed column (key domain d = v ^ flip)
    int32_t pred;             // index of the predicate over the same column, or -1
};

// Value of aggregate column a at row p.  Hot case inline (a bit-packed column
// without residual, e.g. l_extendedprice: one or two loads from one sector),
// everything else through the out-of-line generic path.
__device__ __forceinline__ uint32_t agg_gather(const AggCol& a, uint64_t p) {
    if (a.k == 0 && a.layout == AR_LAYOUT_PACKED && a.w > 0) return packed_get(a.major, p, (int)a.w) + a.base;
    return value_get(a.major, a.residual, p, (int)a.w, (int)a.k, (int)a.layout, a.base, (int)a.rlayout);
}

constexpr int kSelWarps = 4;                      // consumer warps per CTA
constexpr int kSelThreads = kSelWarps * 32;       // each consumer thread owns BPT consecutive 32-row blocks
constexpr int kSelMinTileRows = kSelThreads * 32; // tile rows = 4096 * BPT (BPT in {1, 2, 4})
constexpr int kStageEntries = 2048;
constexpr int kRrEntries = 512; 
constexpr int kRrMinPlanes = 12;      // ar_approx_select: select_rr_kernel for wider tiles (AR_SEL_RR=1)
constexpr int kRrSyncEntries = 2048;   // select_rr_kernel: denser tiles resolve at once and write directly
   // select_rr_kernel: staged entries per tile buffer (denser tiles resolve at once)
#ifndef AR_GROUP_SHIFT
#define AR_GROUP_SHIFT 8
#endif
constexpr int kGroupShift = AR_GROUP_SHIFT;       // select: 2^kGroupShift tiles per offset group

struct SelParams {
    SelPred p[AR_MAX_PRED];
    uint32_t pm[AR_MAX_PLANES][4];   // per global plane (ashift + j): cand lo/hi, def lo/hi bit as 0 / ~0
    int32_t npred;
    int32_t carry;            // write the approximation word into aux
    int64_t n;
    int64_t num_tiles;
    uint32_t stage_words;     // uint32 words per pipeline stage (all predicates)
    uint32_t nstages;
    uint32_t bpt;             // 32-row blocks per consumer thread (template parameter of the launch)
    uint32_t suspend_ns;      // mbarrier wait suspend hint (0 = spin)
    uint32_t prod_wait;       // producer's wait for a free stage: 0 = nanosleep back-off, 1 = try_wait,
                              // > 1 = try_wait with that suspend hint (ns)
    uint32_t debug;           // experiments only (AR_DEBUG): 1 = no look-back (provisional offsets), 2 = no copy-out
    uint32_t tile_rows;       // kSelMinTileRows * bpt
    uint32_t* out_pos;
    uint32_t* out_aux;
    long long* out_count;
    unsigned long long* status;   // [num_tiles] look-back words (unused by the select)
    unsigned int* ticket;         // dynamic tile counter (unused by the select)
    uint32_t* tile_count;         // select: [num_tiles] candidates per tile
    unsigned long long* group_sum; // select: candidates per group of 2^kGroupShift tiles (zeroed per call)
    uint32_t* tmp_pos;            // select: tile-local candidate slices (workspace, n entries)
    uint32_t* tmp_aux;
    // fused kernel only
    AggCol a[AR_MAX_AGG];
    int32_t nagg;
    int32_t exact_mode;           // fused: every decomposed predicate has its residual planes streamed, so
                                  // the exact predicate is evaluated on major + residual planes in place
    uint32_t pmx[AR_MAX_PRED][32][2];   // exact bounds, bit i of (lo - base) / (hi - base) as 0 / ~0
    uint32_t pmh[AR_MAX_PRED][32][4];   // split residuals: candidate lo / hi, definite lo / hi bits of the
                                        // relaxation at granularity k - h over (major << h | high planes)
    int32_t async_agg;            // fused: the one gathered aggregate column uses asynchronous gathers
    int32_t gidx;                 // index of that column in a[]
    unsigned long long* out4;     // sum, |result|, |cand|, |def|
    // result-ring kernel (fused.cu) only
    int32_t rl_list;              // 1: one gathered SUM factor, rows queued in the warp result ring
    int32_t rl_mpred;             // predicate whose exact value is the other SUM factor, or -1
    uint32_t rl_ring;             // result-ring entries per warp (power of two)
    uint32_t rl_depth;            // gather passes in flight per warp (4 or 8)
    int32_t rl_fin;               // 1: finalize out4 through rl_part / rl_ticket (no memset before the launch)
    int32_t rl_pdl;               // programmatic dependent launch: 1 = wait before reading inputs, 2 = read
                                  // inputs at once (caller: the previous kernel does not write them)
    unsigned long long* rl_part;  // [gridDim][4] CTA partials
    unsigned int* rl_ticket;      // CTAs done (zero between calls)
};

// Producer of the persistent scan kernels: one lane streams tiles (tile =
// blockIdx + i * gridDim) of every predicate's bit planes -- and, for streamed
// predicates, the tile's SLICED residual planes -- into a ring of nstages
// shared-memory stages with 1-D TMA bulk copies completing on full[s].  A tile
// index past the end is passed on as -1 and ends the stream.
__device__ __forceinline__ void produce_ring(const SelParams& P, uint64_t* full, uint64_t* empty, long long* slot,
                                             uint32_t* stages) {
    const uint64_t pol = policy_evict_first();
    const uint32_t blocks_per_tile = P.tile_rows / 32;
    uint32_t s = 0, ph = 0;   // ring slot and its phase parity (no integer division in the loop)
    for (uint32_t i = 0;; ++i) {
        if (i >= P.nstages) {
            if (P.prod_wait == 0)
                mbar_wait_sleep(empty + s, ph ^ 1u);   // back off with __nanosleep instead of spinning
            else
                mbar_wait(empty + s, ph ^ 1u, P.prod_wait == 1 ? 0u : P.prod_wait);   // hardware-suspended try_wait
        }
        const long long t = (long long)blockIdx.x + (long long)i * gridDim.x;
        if (t >= P.num_tiles) {
            slot[s] = -1;
            mbar_arrive(full + s);
            return;
        }
        slot[s] = t;
        const int64_t r0 = t * (int64_t)P.tile_rows;
        const int64_t rows = min((int64_t)P.tile_rows, P.n - r0);
        const uint32_t groups = (uint32_t)((rows + 127) / 128);   // 128-row groups, 16 B per plane
        uint32_t bytes = 0;
        for (int c = 0; c < P.npred; ++c) {
            bytes += groups * 16u * P.p[c].w;
            if (P.p[c].res_stream) bytes += groups * 16u * (P.p[c].rsplit ? P.p[c].rsplit : P.p[c].k);
        }
        mbar_arrive_expect_tx(full + s, bytes);
        uint32_t* stg = stages + (size_t)s * P.stage_words;
        for (int c = 0; c < P.npred; ++c) {
            const uint32_t w = P.p[c].w;
            if (w > 0)
                bulk_g2s(stg + P.p[c].soff, P.p[c].planes + (size_t)t * blocks_per_tile * w, groups * 16u * w,
                         full + s, pol);
            if (P.p[c].res_stream && P.p[c].rsplit) {
                // split residual: the tile's high planes, one chunk per super-group it covers
                const uint32_t k = P.p[c].k, h = P.p[c].rsplit, nb = groups * 4u;
                const uint64_t b0 = (uint64_t)t * blocks_per_tile;
                for (uint32_t done = 0; done < nb;) {
                    const uint64_t b = b0 + done;
                    const uint32_t bb = (uint32_t)(b % kSplitBlocks);
                    const uint32_t cnt = min(nb - done, (uint32_t)kSplitBlocks - bb);
                    bulk_g2s(stg + P.p[c].res_soff + done * h, P.p[c].residual + split_hi_word(b, (int)k, (int)h),
                             cnt * 4u * h, full + s, pol);
                    done += cnt;
                }
            } else if (P.p[c].res_stream) {   // the tile's SLICED residual planes
                const uint32_t k = P.p[c].k;
                bulk_g2s(stg + P.p[c].res_soff, P.p[c].residual + (size_t)t * blocks_per_tile * k,
                         groups * 16u * k, full + s, pol);
            }
        }
        if (++s == P.nstages) {
            s = 0;
            ph ^= 1u;
        }
    }
}

struct RefPred {
    const uint32_t* major;
    const uint32_t* residual;
    uint32_t w, k, layout, base, lo, hi, rlayout;
    uint32_t ashift;
    uint32_t carried;         // major available in aux
    uint32_t check;           // k > 0: must be re-evaluated on the exact value
};

constexpr int kRefThreads = 256;
constexpr int kRefPerThread = 8;
constexpr int kRefTile = kRefThreads * kRefPerThread;   // 2048 candidates per tile
constexpr int kRefWarpCopy = kRefTile;   // refine_kernel: a pending tile with more kept positions is copied out by the CTA (never: measured slower at C4)

struct RefParams {
    RefPred p[AR_MAX_PRED];
    int32_t npred;
    const uint32_t* in_pos;
    const uint32_t* in_aux;
    const long long* in_count;
    uint32_t* out_pos;
    long long* out_count;
    unsigned long long* status;
    unsigned int* ticket;
    AggCol a[AR_MAX_AGG];
    int32_t nagg;
    unsigned long long* out_sum;
    unsigned long long* out_cnt;
    // refine_sum_sliced_kernel (fast_k = 4 / 8, else 0): the one checked predicate and the gathered factor
    int32_t fast_k, fast_chk, fast_g;
};

struct SumParams {
    const uint32_t* pos;
    const long long* count;
    AggCol a[AR_MAX_AGG];
    int32_t nagg;
    unsigned long long* out_sum;
};

// sumapproximate over a candidate relation (bounds from the majors only)
struct ApproxSumParams {
    const uint32_t* pos;
    const uint32_t* aux;
    const long long* count;
    AggCol a[AR_MAX_AGG];
    int32_t nagg;
    unsigned long long* out4;   // [sum_lo, sum_hi, count_lo, count_hi]
};

// MIN / MAX with the selection's error bounds propagated (s IV-F, Fig. 6)
struct MinMaxParams {
    RefParams r;              // candidate relation + predicates (exact re-evaluation)
    AggCol y;                 // the aggregated column (pred >= 0: its major is in the aux word)
    int32_t mode;             // AR_MIN / AR_MAX
    unsigned int* ws;         // [0..3] min/max major over candidates / definite, [4] best exact key (xored)
    unsigned long long* wc;   // [0] |definite|, [1] rows refined, [2] survivors
    uint32_t* ymaj;           // [capacity] Y's major per candidate (approximate pass -> refine pass)
    long long* out7;
};

// grouped COUNT / SUM over the refined rows (s IV-E/F) by a GPU-resident key
struct GroupParams {
    RefParams r;              // candidates, predicates, aggregate factors (r.a, r.nagg)
    AggCol key;               // k == 0, unsigned; group id = key value (< ngroups, host-checked)
    const uint32_t* gids;     // or: group id per candidate (aligned with the candidate relation), < ngroups
    int32_t ngroups;
    unsigned long long* out;  // [ngroups] sums, then [ngroups] counts
};

// leftjoinapproximate / leftjoinrefine (positional projection)
struct ProjectParams {
    const uint32_t* pos;
    const long long* count;
    AggCol a;
    int32_t exact;
    uint32_t* out;
};

}  // namespace ard

namespace ar {
// launchers (return AR_OK or the CUDA failure)
size_t select_smem_bytes(uint32_t stage_words, uint32_t nstages, bool staging);
int kernel_warps(bool fused);
int kernel_bpt(bool fused);
const void* select_kernel_fn(const ard::SelParams& P, bool fused);
const void* select_rr_kernel_fn(const ard::SelParams& P);
size_t select_rr_smem_bytes(uint32_t stage_words, uint32_t nstages);
ar_status launch_select_rr(const void* fn, const ard::SelParams& P, int grid, size_t smem, cudaStream_t s);
int select_occupancy(const void* fn, size_t smem, bool fused);
ar_status launch_scan(const void* fn, const ard::SelParams& P, int grid, size_t smem, bool fused, cudaStream_t s);
ar_status launch_select_rest(const ard::SelParams& P, bool pdl, cudaStream_t s);
// ar_select_refine_sum_ws workspace: a ticket word (padded), then kSrsMaxGrid CTA partials of 4 x u64
constexpr size_t kSrsTicketBytes = 128;
constexpr int kSrsMaxGrid = 2048;
void retile(ard::SelParams& P, uint32_t tile_rows);   // fused.cu
ar_status launch_fused_rl(const ard::SelParams& P, const ar_column* const* cols, void* ws, int pdl, bool* launched,
                          bool* gathered_res, cudaStream_t s);
ar_status launch_refine(const ard::RefParams& P, int grid, bool wide, cudaStream_t s);
const void* refine_kernel_fn(bool wide);
ar_status launch_refine_sum(const ard::RefParams& P, int grid, cudaStream_t s);
ar_status launch_sum(const ard::SumParams& P, int grid, cudaStream_t s);
ar_status launch_approx_sum(const ard::ApproxSumParams& P, int grid, cudaStream_t s);
ar_status launch_project(const ard::ProjectParams& P, int grid, cudaStream_t s);
ar_status launch_minmax(const ard::MinMaxParams& P, int grid, cudaStream_t s);
ar_status launch_group_sum(const ard::GroupParams& P, int grid, cudaStream_t s);
ar_status launch_decompose_minmax(const uint32_t* col, int64_t n, uint32_t flip, uint32_t* out2, cudaStream_t s);
ar_status launch_pack_sliced(const uint32_t* col, int64_t n, int shift, uint32_t mask, uint32_t flip, uint32_t base,
                             int w, uint32_t* out, cudaStream_t s);
ar_status launch_pack_split(const uint32_t* col, int64_t n, int k, int h, uint32_t flip, uint32_t base, uint32_t* out,
                            cudaStream_t s);
ar_status launch_pack_packed(const uint32_t* col, int64_t n, int shift, uint32_t mask, uint32_t flip, uint32_t base,
                             int w, uint64_t out_words, uint32_t* out, cudaStream_t s);
ar_status launch_exclusive_offset(const long long* all_counts, int world, int rank, long long* out, long long* total,
                                  cudaStream_t s);
}  // namespace ar

// common.cuh -- shared internals of the A&R CUDA library (sm_100a).
// Column handle, host error plumbing, device bit-extraction / gather helpers,
// mbarrier + cp.async.bulk (TMA bulk copy) PTX wrappers, decoupled look-back.
#pragma once

#include <cuda_runtime.h>
#include <stdint.h>
#include <stdio.h>
#include <stdarg.h>
#include <string>
#include <algorithm>

#include "../../include/ar.h"

struct ar_column {
    ar_column_desc d;
    const uint32_t* major;      // device pointer (SLICED or PACKED, width d.w_major)
    const uint32_t* residual;   // device pointer, or device alias of pinned host memory (width d.k)
};

// Split SLICED residual: 32-row blocks per super-group (8192 rows, one default
// one-pass tile, so a tile's high planes are one contiguous chunk).
constexpr int kSplitBlocks = 256;

// ------------------------------------------------------------------ host side

namespace ar {

void set_error(const char* fmt, ...);
ar_status cuda_fail(cudaError_t e, const char* where);
int num_sms();
int current_device();
// Opt `fn` in to the largest dynamic shared memory it can have on the current
// device (the opt-in maximum minus its static shared memory), once per
// (device, kernel) and host thread: function attributes are per device.
void opt_in_max_smem(const void* fn);

inline uint64_t ceil_div_u64(uint64_t a, uint64_t b) { return (a + b - 1) / b; }

// Bytes of a SLICED major part: blocks of 32 rows, padded to 128-row groups so
// that every 4096-row tile (and every 128-row shard boundary) is 16-B aligned.
inline uint64_t sliced_bytes(int64_t n, int w) {
    return w == 0 ? 0 : ceil_div_u64((uint64_t)n, 128) * 16ull * (uint64_t)w;
}
// Split SLICED residual (k planes, h of them stored apart): super-groups of
// kSplitBlocks 32-row blocks, each kSplitBlocks x k words.
inline uint64_t split_bytes(int64_t n, int k) {
    return k == 0 ? 0 : ceil_div_u64((uint64_t)n, 32ull * kSplitBlocks) * 4ull * kSplitBlocks * (uint64_t)k;
}
// Residual layout code carried to the kernels: ar_layout | (residual_split << 8).
inline uint32_t rlayout_code(const ar_column_desc& d) {
    return (uint32_t)d.residual_layout | ((uint32_t)d.residual_split << 8);
}

// Bytes of a PACKED bitstream of width w: ceil(n*w/32) words + 1 guard word
// (a straddling value may read word i+1), rounded up to 16 B.
inline uint64_t packed_bytes(int64_t n, int w) {
    if (w == 0) return 0;
    uint64_t words = ceil_div_u64((uint64_t)n * (uint64_t)w, 32) + 1;
    return ceil_div_u64(words * 4, 16) * 16;
}

// Relaxation of one exact conjunct [lo, hi] to the major domain (step a2).
// Tight reading (DESIGN "Readings"):
//   u = v - base;  cand(m) <=> [m 2^k, m 2^k + 2^k - 1] meets [ulo, uhi]
//                  def(m)  <=> [m 2^k, m 2^k + 2^k - 1] inside [ulo, uhi]
struct Relaxed {
    bool empty;          // no row can qualify
    uint32_t clo, chi;   // candidate major range (inclusive, <= 2^w - 1)
    bool def_any;        // definite range non-empty
    uint32_t dlo, dhi;   // definite major range
};
Relaxed relax(uint32_t lo, uint32_t hi, uint32_t base, int k, int w);

}  // namespace ar

#define AR_TRY_CUDA(expr)                                         \
    do {                                                          \
        cudaError_t _e = (expr);                                  \
        if (_e != cudaSuccess) return ar::cuda_fail(_e, #expr);   \
    } while (0)

#define AR_CHECK_LAUNCH(name)                                     \
    do {                                                          \
        cudaError_t _e = cudaGetLastError();                      \
        if (_e != cudaSuccess) return ar::cuda_fail(_e, name);    \
    } while (0)

// ---------------------------------------------------------------- device side

namespace ard {

__device__ __forceinline__ uint32_t smem_u32(const void* p) {
    return static_cast<uint32_t>(__cvta_generic_to_shared(p));
}

// --- mbarrier (Hopper+) -------------------------------------------------------
__device__ __forceinline__ void mbar_init(uint64_t* bar, uint32_t count) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(count) : "memory");
}
__device__ __forceinline__ void fence_mbar_init() {
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
}
__device__ __forceinline__ void mbar_arrive_expect_tx(uint64_t* bar, uint32_t bytes) {
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes)
                 : "memory");
}
__device__ __forceinline__ void mbar_arrive(uint64_t* bar) {
    asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(smem_u32(bar)) : "memory");
}
// Blocking wait on an mbarrier phase.  With a suspend-time hint (ns) the
// hardware may park the thread until the phase completes instead of returning
// after its short default window (a spinning warp steals issue slots);
// hint == 0 is a plain try_wait loop.  The hint is a kernel parameter
// (AR_SUSPEND_NS) so it can be tuned without recompiling.
__device__ __forceinline__ void mbar_wait(uint64_t* bar, uint32_t parity, uint32_t hint_ns) {
    if (hint_ns) {
        asm volatile(
            "{\n\t.reg .pred p;\n"
            "AR_WAIT_%=:\n\t"
            "mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1, %2;\n\t"
            "@!p bra AR_WAIT_%=;\n}" ::"r"(smem_u32(bar)),
            "r"(parity), "r"(hint_ns)
            : "memory");
    } else {
        asm volatile(
            "{\n\t.reg .pred p;\n"
            "AR_WAIT_%=:\n\t"
            "mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n\t"
            "@!p bra AR_WAIT_%=;\n}" ::"r"(smem_u32(bar)),
            "r"(parity)
            : "memory");
    }
}

// The same on a shared-window address (smem_u32 of the barrier computed once by
// the caller: the generic -> shared conversion is several instructions).
__device__ __forceinline__ void mbar_wait_a(uint32_t bar, uint32_t parity, uint32_t hint_ns) {
    if (hint_ns) {
        asm volatile(
            "{\n\t.reg .pred p;\n"
            "AR_WAIT_%=:\n\t"
            "mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1, %2;\n\t"
            "@!p bra AR_WAIT_%=;\n}" ::"r"(bar),
            "r"(parity), "r"(hint_ns)
            : "memory");
    } else {
        asm volatile(
            "{\n\t.reg .pred p;\n"
            "AR_WAIT_%=:\n\t"
            "mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n\t"
            "@!p bra AR_WAIT_%=;\n}" ::"r"(bar),
            "r"(parity)
            : "memory");
    }
}
__device__ __forceinline__ void mbar_arrive_a(uint32_t bar) {
    asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(bar) : "memory");
}

// Wait with an exponential __nanosleep back-off between probes: for a lone
// producer lane, whose spinning would otherwise take issue slots from the
// consumer warps of its SM.
__device__ __forceinline__ void mbar_wait_sleep(uint64_t* bar, uint32_t parity) {
    uint32_t ns = 256;
    while (true) {
        uint32_t done;
        asm volatile(
            "{\n\t.reg .pred p;\n\t"
            "mbarrier.test_wait.parity.shared::cta.b64 p, [%1], %2;\n\t"
            "selp.u32 %0, 1, 0, p;\n}"
            : "=r"(done)
            : "r"(smem_u32(bar)), "r"(parity)
            : "memory");
        if (done) return;
        __nanosleep(ns);
        if (ns < 2048) ns <<= 1;
    }
}

// --- TMA bulk copy global -> shared (1-D, no tensor map), completes on an mbarrier
__device__ __forceinline__ void bulk_g2s(void* dst, const void* src, uint32_t bytes, uint64_t* bar,
                                         uint64_t policy) {
    asm volatile(
        "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes.L2::cache_hint [%0], [%1], %2, [%3], %4;" ::
            "r"(smem_u32(dst)),
        "l"(src), "r"(bytes), "r"(smem_u32(bar)), "l"(policy)
        : "memory");
}
__device__ __forceinline__ uint64_t policy_evict_first() {
    uint64_t p;
    asm volatile("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(p));
    return p;
}

// --- named barrier among the consumer warps only (id 1; id 0 is __syncthreads)
__device__ __forceinline__ void bar_sync(uint32_t id, uint32_t nthreads) {
    asm volatile("bar.sync %0, %1;" ::"r"(id), "r"(nthreads) : "memory");
}

// --- 64-bit per-tile status words (rr_prefix below).  Each word carries its own
// flag and value, and no other data is published through it, so relaxed
// gpu-scope single-copy-atomic accesses are sufficient.
__device__ __forceinline__ void st_relaxed(unsigned long long* p, unsigned long long v) {
    asm volatile("st.relaxed.gpu.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ unsigned long long ld_relaxed(const unsigned long long* p) {
    unsigned long long v;
    asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}

constexpr unsigned long long kFlagAgg = 1ull << 62;
constexpr unsigned long long kFlagInc = 1ull << 63;   // inclusive prefix (select_rr_kernel)
constexpr unsigned long long kValueMask = (1ull << 62) - 1;

// Round-robin persistent kernels (tile t = blockIdx + i * gridDim, every CTA
// resident, tiles walked in order): each tile publishes kFlagAgg | count in
// status[t] at once; warp 0 of the owner then obtains the exclusive prefix as
// its CTA's previous inclusive prefix + the aggregates of the gridDim - 1 tiles
// in between -- no chain of inclusive prefixes.  gridDim <= 32 * kAggPerLane.
constexpr int kAggPerLane = 20;
// Warp 0: exclusive prefix of tile t = this CTA's previous tile's inclusive
// prefix + the aggregates of the tiles in between (t - G, t).
__device__ __forceinline__ unsigned long long rr_prefix(const unsigned long long* status, long long t, unsigned lane,
                                                        unsigned long long prev_incl) {
    const long long lo = t - (long long)gridDim.x + 1 > 0 ? t - (long long)gridDim.x + 1 : 0;
    unsigned long long v[kAggPerLane];
#pragma unroll
    for (int q = 0; q < kAggPerLane; ++q) {
        const long long idx = lo + lane + 32 * q;
        v[q] = idx < t ? ld_relaxed(status + idx) : kFlagAgg;
    }
    while (true) {
        bool ready = true;
#pragma unroll
        for (int q = 0; q < kAggPerLane; ++q) ready &= (v[q] >> 62) != 0;
        if (__all_sync(0xffffffffu, ready)) break;
        __nanosleep(32);
#pragma unroll
        for (int q = 0; q < kAggPerLane; ++q) {
            const long long idx = lo + lane + 32 * q;
            if ((v[q] >> 62) == 0) v[q] = ld_relaxed(status + idx);
        }
    }
    unsigned long long sum = 0;
#pragma unroll
    for (int q = 0; q < kAggPerLane; ++q) sum += v[q] & kValueMask;
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) sum += __shfl_xor_sync(0xffffffffu, sum, o);
    return prev_incl + sum;
}

// Warp-wide decoupled look-back (Merrill & Garland) over per-tile status words:
// exclusive prefix of tile t from the windows of the 32 preceding words, each
// either a count (kFlagAgg, published right after the tile is decided) or an
// inclusive prefix (kFlagInc, published when the tile is resolved); the walk
// ends at the first inclusive prefix.  Lane 0 publishes t's inclusive prefix.
// Every lane returns the exclusive prefix.  Waits only for counts.
__device__ __forceinline__ unsigned long long lookback_inclusive(unsigned long long* status, long long t,
                                                                 unsigned long long total, unsigned lane) {
    unsigned long long excl = 0;
    long long idx = t - 1;
    while (idx >= 0) {
        const long long j = idx - (long long)lane;
        unsigned long long v = j >= 0 ? ld_relaxed(status + j) : kFlagInc;
        while (!__all_sync(0xffffffffu, (v >> 62) != 0)) {
            __nanosleep(32);
            if ((v >> 62) == 0) v = ld_relaxed(status + j);
        }
        const unsigned inc = __ballot_sync(0xffffffffu, (v >> 63) != 0);
        const unsigned upto = inc ? (__ffs(inc) - 1) : 31u;   // lanes 0..upto contribute
        unsigned long long x = lane <= upto ? (v & kValueMask) : 0ull;
#pragma unroll
        for (int o = 16; o > 0; o >>= 1) x += __shfl_xor_sync(0xffffffffu, x, o);
        excl += x;
        if (inc) break;
        idx -= 32;
    }
    if (lane == 0) st_relaxed(status + t, kFlagInc | (excl + total));
    return excl;
}

// --- value extraction ----------------------------------------------------------

#ifndef AR_GHINT
#define AR_GHINT ".L2::64B"
#endif
// Gather load of one word.  On B200 a plain scalar load makes L2 fetch a whole
// 128-B line from HBM; the .L2::64B prefetch-size hint halves that, which is the
// smallest gather granularity measured (tools/gather_probe.cu, DESIGN "Gathers").
__device__ __forceinline__ uint32_t ld_gather(const uint32_t* p) {
    uint32_t v;
    asm volatile("ld.global.nc" AR_GHINT ".u32 %0, [%1];" : "=r"(v) : "l"(p));   // volatile: never speculated past its guard
    return v;
}

// Predicated, non-volatile gathers for kernels that issue a batch of gathers
// before using any of them: the compiler may reorder and overlap them, and the
// predicate (not a branch the compiler could if-convert) keeps an unneeded
// gather from touching memory.  A skipped load returns 0.
__device__ __forceinline__ uint32_t ld_gather_if(const uint32_t* p, bool pred) {
    uint32_t v = 0;
    asm("{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %2, 0;\n\t@q ld.global.nc" AR_GHINT ".u32 %0, [%1];\n\t}"
        : "+r"(v) : "l"(p), "r"((uint32_t)pred));
    return v;
}
__device__ __forceinline__ uint4 ld_gather_if4(const uint32_t* p, bool pred) {   // 16-B aligned
    uint4 v = make_uint4(0, 0, 0, 0);
    asm("{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %5, 0;\n\t@q ld.global.nc" AR_GHINT ".v4.u32 {%0,%1,%2,%3}, [%4];\n\t}"
        : "+r"(v.x), "+r"(v.y), "+r"(v.z), "+r"(v.w) : "l"(p), "r"((uint32_t)pred));
    return v;
}
// The same gathers without the L2 prefetch-size hint: for pinned host memory
// read over the host link, where the request size is the transfer size
// (AR_HOST_HINT selects, DESIGN s6.3c).
__device__ __forceinline__ uint32_t ld_gather_if_nh(const uint32_t* p, bool pred) {
    uint32_t v = 0;
    asm("{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %2, 0;\n\t@q ld.global.nc.u32 %0, [%1];\n\t}"
        : "+r"(v) : "l"(p), "r"((uint32_t)pred));
    return v;
}
__device__ __forceinline__ uint4 ld_gather_if4_nh(const uint32_t* p, bool pred) {   // 16-B aligned
    uint4 v = make_uint4(0, 0, 0, 0);
    asm("{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %5, 0;\n\t@q ld.global.nc.v4.u32 {%0,%1,%2,%3}, [%4];\n\t}"
        : "+r"(v.x), "+r"(v.y), "+r"(v.z), "+r"(v.w) : "l"(p), "r"((uint32_t)pred));
    return v;
}
__device__ __forceinline__ uint32_t packed_get_if(const uint32_t* __restrict__ s, uint64_t p, int w, bool pred) {
    const uint64_t bit = p * (uint64_t)w;
    const uint32_t sh = (uint32_t)(bit & 31);
    const uint32_t lo = ld_gather_if(s + (bit >> 5), pred);
    const uint32_t hi = ld_gather_if(s + (bit >> 5) + 1, pred && sh + (uint32_t)w > 32u);
    const uint32_t v = __funnelshift_r(lo, hi, sh);
    return w == 32 ? v : (v & ((1u << w) - 1u));
}
// Split SLICED residual (layout code AR_LAYOUT_SLICED | h << 8).  Per
// super-group of kSplitBlocks blocks: the h high planes of its blocks (h words
// per block, planes k-h .. k-1), then the k - h low planes (k - h words per
// block, planes 0 .. k-h-1).  So a tile's high planes are one contiguous chunk
// (streamed) and a block's low planes are k - h consecutive words (gathered).
__device__ __forceinline__ uint64_t split_hi_word(uint64_t blk, int k, int h) {   // plane k - h of block blk
    return (blk / kSplitBlocks) * ((uint64_t)kSplitBlocks * k) + (blk % kSplitBlocks) * (uint64_t)h;
}
__device__ __forceinline__ uint64_t split_lo_word(uint64_t blk, int k, int h) {   // plane 0 of block blk
    return (blk / kSplitBlocks) * ((uint64_t)kSplitBlocks * k) + (uint64_t)kSplitBlocks * h +
           (blk % kSplitBlocks) * (uint64_t)(k - h);
}
// word of plane j (bit j of the residual, j < k) of 32-row block blk
__device__ __forceinline__ uint64_t split_word(uint64_t blk, int k, int h, int j) {
    return j >= k - h ? split_hi_word(blk, k, h) + (uint64_t)(j - (k - h)) : split_lo_word(blk, k, h) + (uint64_t)j;
}

// Residual of row p: SLICED blocks of k = 4 / 8 planes (16-B aligned) in one or
// two vector loads of the block's sector, other widths (and the split layout)
// word by word.
__device__ __forceinline__ uint32_t residual_get_if(const uint32_t* s, uint64_t p, int k, int layout, bool pred) {
    if ((layout & 0xff) != AR_LAYOUT_SLICED) return packed_get_if(s, p, k, pred);
    const uint32_t l = (uint32_t)(p & 31);
    uint32_t r = 0;
    const int h = layout >> 8;
    if (h) {
        for (int j = 0; j < k; ++j) r |= ((ld_gather_if(s + split_word(p >> 5, k, h, j), pred) >> l) & 1u) << j;
        return r;
    }
    const uint32_t* blk = s + (p >> 5) * (uint64_t)k;
    if (k == 8 || k == 4) {
        const uint4 a = ld_gather_if4(blk, pred);
        r = ((a.x >> l) & 1u) | (((a.y >> l) & 1u) << 1) | (((a.z >> l) & 1u) << 2) | (((a.w >> l) & 1u) << 3);
        if (k == 8) {
            const uint4 b = ld_gather_if4(blk + 4, pred);
            r |= (((b.x >> l) & 1u) << 4) | (((b.y >> l) & 1u) << 5) | (((b.z >> l) & 1u) << 6) |
                 (((b.w >> l) & 1u) << 7);
        }
        return r;
    }
    for (int j = 0; j < k; ++j) r |= ((ld_gather_if(blk + j, pred) >> l) & 1u) << j;
    return r;
}

// Value of row p from a PACKED LSB-first bitstream of width w (1..32) in global memory.
__device__ __forceinline__ uint32_t packed_get(const uint32_t* __restrict__ s, uint64_t p, int w) {
    uint64_t bit = p * (uint64_t)w;
    uint64_t wi = bit >> 5;
    uint32_t sh = (uint32_t)(bit & 31);
    uint32_t lo = ld_gather(s + wi);
    uint32_t v = lo >> sh;
    if (sh + (uint32_t)w > 32u) v = __funnelshift_r(lo, ld_gather(s + wi + 1), sh);
    return w == 32 ? v : (v & ((1u << w) - 1u));
}
// Residual of row p (width k) in any layout, from device memory or from
// pinned host memory through a mapped pointer.  SLICED (k <= 8): the block's k
// planes sit in one 32-B sector; split: its high and low planes in two places.
__device__ __forceinline__ uint32_t residual_get(const uint32_t* s, uint64_t p, int k, int layout) {
    if ((layout & 0xff) == AR_LAYOUT_SLICED) {
        const uint32_t l = (uint32_t)(p & 31);
        const int h = layout >> 8;
        uint32_t r = 0;
        if (h) {
            for (int j = 0; j < k; ++j) r |= ((ld_gather(s + split_word(p >> 5, k, h, j)) >> l) & 1u) << j;
            return r;
        }
        const uint32_t* blk = s + (p >> 5) * (uint64_t)k;
        for (int j = 0; j < k; ++j) r |= ((ld_gather(blk + j) >> l) & 1u) << j;
        return r;
    }
    return packed_get(s, p, k);
}

// Same extraction from a PACKED stream staged in shared memory (bit offset `bit`).
__device__ __forceinline__ uint32_t packed_get_smem(const uint32_t* s, uint32_t bit, int w) {
    const uint32_t wi = bit >> 5, sh = bit & 31;
    const uint32_t lo = s[wi];
    uint32_t v = lo >> sh;
    if (sh + (uint32_t)w > 32u) v = __funnelshift_r(lo, s[wi + 1], sh);
    return w == 32 ? v : (v & ((1u << w) - 1u));
}

// Major of row p from a SLICED part of width w (w words per 32-row block).
// Off the hot path (majors of predicate columns travel in the aux word), so
// kept out of line to keep the kernels' instruction footprint small.
static __device__ __noinline__ uint32_t sliced_get(const uint32_t* __restrict__ s, uint64_t p, int w) {
    const uint32_t* blk = s + (p >> 5) * (uint64_t)w;
    uint32_t l = (uint32_t)(p & 31);
    uint32_t m = 0;
    for (int j = 0; j < w; ++j) m |= ((__ldg(blk + j) >> l) & 1u) << j;
    return m;
}

__device__ __forceinline__ uint32_t major_get(const uint32_t* __restrict__ s, uint64_t p, int w, int layout) {
    if (w == 0) return 0;
    return layout == AR_LAYOUT_SLICED ? sliced_get(s, p, w) : packed_get(s, p, w);
}

// Exact value of row p of a column (major and residual joined).
// Generic (any layout, any k): out of line; kernels inline only their hot case.
static __device__ __noinline__ uint32_t value_get(const uint32_t* major, const uint32_t* residual, uint64_t p,
                                              int w, int k, int layout, uint32_t base, int rlayout) {
    uint32_t m = major_get(major, p, w, layout);
    uint32_t r = k ? residual_get(residual, p, k, rlayout) : 0u;
    uint32_t u = k == 32 ? r : ((m << k) | r);
    return u + base;
}

// Valid-row mask of the 32-row block starting at row r0 of an n-row column.
__device__ __forceinline__ uint32_t valid_mask(int64_t r0, int64_t n) {
    int64_t rem = n - r0;
    return rem >= 32 ? 0xffffffffu : (rem <= 0 ? 0u : ((1u << rem) - 1u));
}

// Block-wide exclusive scan of one uint32 per thread over NT threads (consumer
// warps only, named barrier `bar`).  `warp_tot` is smem of NT/32 words.
template <int NT>
__device__ __forceinline__ uint32_t block_excl_scan(uint32_t x, uint32_t* warp_tot, uint32_t& total, uint32_t bar) {
    const unsigned lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    uint32_t incl = x;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
        uint32_t y = __shfl_up_sync(0xffffffffu, incl, o);
        if (lane >= (unsigned)o) incl += y;
    }
    if (lane == 31) warp_tot[warp] = incl;
    bar_sync(bar, NT);
    uint32_t before = 0, all = 0;
#pragma unroll
    for (int i = 0; i < NT / 32; ++i) {
        uint32_t t = warp_tot[i];
        before += (i < (int)warp) ? t : 0u;
        all += t;
    }
    total = all;
    return before + incl - x;
}

}  // namespace ard

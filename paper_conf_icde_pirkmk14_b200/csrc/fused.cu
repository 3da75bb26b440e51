// fused.cu -- one-pass A&R with a per-warp result ring: a3 approximate select,
// a5 refine and a6 SUM in one persistent kernel (SURVEY s8(a) "Fusion note").
//
// Applies when every decomposed predicate has its SLICED residual planes
// (k <= 8) streamed with the majors (SelParams.exact_mode), so the exact
// predicate of Alg. 2 is decided on the planes in the scan
// itself: the bitwise concatenation of residual and major planes (the "+bw"
// join of PAPER.md:637-638) runs through one borrow chain against the exact
// bounds.  Candidate and definite masks (definite = SURVEY
// A6) are still evaluated for the |cand| / |def| counts of out4.
//
// Per tile the work is then:
//   1. every consumer thread decides BPT 32-row blocks (blocks interleaved over
//      the CTA, so the 16-B plane loads of a warp are contiguous in smem);
//   2. the warp appends its result rows to a ring in shared memory -- (row,
//      other SUM factor), the factor read from the stage while it is held --
//      and releases the stage;
//   3. whenever the ring holds 32 entries, one lane-parallel pass issues the
//      gathers of the aggregate column (l_extendedprice) as asynchronous
//      cp.async copies into a per-warp slot ring; a slot is summed kDepth - 1
//      passes later, so no warp ever waits on a gather.
// Compared with fused_kernel (select.cu) the per-tile bookkeeping runs once
// per BPT blocks, the list holds results only, and its passes are always full.
#include <type_traits>

#include "rl_common.cuh"

namespace ard {
namespace rl {

constexpr int kRingDefault = 128;         // result entries (row, factor) per warp (power of two)
constexpr int kDepth = 4;                 // gather passes in flight per warp
constexpr int kSlotWords = 4 * 32;        // per pass: lo[32], hi[32], info[32], factor[32]
// + with a split residual, the KL gathered low-plane words of each lane's row
__host__ __device__ constexpr int slot_words(int kl) { return kSlotWords + 32 * kl; }

// Exact value of predicate C's column at row l of block blk, from the stage.
template <class S, int C>
__device__ __forceinline__ uint32_t stage_value(const SelParams& P, const uint32_t* stg, uint32_t blk, uint32_t l) {
    constexpr int W = S::w(C), K = S::k(C);
    uint32_t m = 0, r = 0;
#pragma unroll
    for (int j = 0; j < W; ++j) m |= ((stg[P.p[C].soff + blk * W + j] >> l) & 1u) << j;
    if constexpr (K > 0) {
#pragma unroll
        for (int j = 0; j < K; ++j) r |= ((stg[P.p[C].res_soff + blk * K + j] >> l) & 1u) << j;
        return ((m << K) | r) + P.p[C].base;
    }
    return m + P.p[C].base;
}

__device__ __forceinline__ void cp_async4(uint32_t* dst, const uint32_t* src) {
    asm volatile("cp.async.ca.shared.global" AR_GHINT " [%0], [%1], 4;" ::"r"(smem_u32(dst)), "l"(src) : "memory");
}
__device__ __forceinline__ void cp_async4_a(uint32_t dst, const uint32_t* src) {   // dst: shared-window address
    asm volatile("cp.async.ca.shared.global" AR_GHINT " [%0], [%1], 4;" ::"r"(dst), "l"(src) : "memory");
}
__device__ __forceinline__ void cp_async16_a(uint32_t dst, const uint32_t* src) {
    asm volatile("cp.async.cg.shared.global" AR_GHINT " [%0], [%1], 16;" ::"r"(dst), "l"(src) : "memory");
}
__device__ __forceinline__ void cp_async16(uint32_t* dst, const uint32_t* src) {
    asm volatile("cp.async.cg.shared.global" AR_GHINT " [%0], [%1], 16;" ::"r"(smem_u32(dst)), "l"(src) : "memory");
}
__device__ __forceinline__ void cp_async_commit() { asm volatile("cp.async.commit_group;" ::: "memory"); }
template <int N>
__device__ __forceinline__ void cp_async_wait() { asm volatile("cp.async.wait_group %0;" ::"n"(N) : "memory"); }

// Low-plane word j of lane `lane` in a slot (KL = 4: one 16-B copy per lane).
template <int KL>
__device__ __forceinline__ uint32_t* low_word(uint32_t* sl, uint32_t lane, int j) {
    return KL == 4 ? sl + kSlotWords + lane * 4 + j : sl + kSlotWords + j * 32 + lane;
}

// Sum one landed gather slot: this lane's entry (a lane only reads what it copied).
// KL > 0: an entry with a check code (info bits 8-9; bit 0: the row lies in the
// fine bucket of lo, bit 1: in that of hi) is a row the high residual planes
// left undecided; its KL low planes (landed with the aggregate) decide it
// against the low bits of the exact bounds, and a row that qualifies counts
// in `nchk`.
// KP > 0 (gathered-residual kernel): the check entries are the non-definite
// candidates of a predicate with a bit-packed KP-bit residual; its two landed
// words and bit offset (info bits 10-14) give the residual, tested the same
// way (the candidate's bucket is that of lo or of hi).  has_g = false (COUNT):
// the ring holds check entries only and nothing is summed.
template <int KL = 0, int KP = 0>
__device__ __forceinline__ unsigned long long drain(uint32_t* sl, uint32_t lane, uint32_t gmask, uint32_t gbase,
                                                    const SelPred* sp = nullptr, uint32_t* nchk = nullptr,
                                                    bool has_g = true) {
    const uint32_t info = sl[64 + lane];
    if (!(info >> 31)) return 0ull;
    if constexpr (KL > 0) {
        const uint32_t code = (info >> 8) & 3u;
        if (code) {
            const uint32_t l = (info >> 10) & 31u;
            uint32_t low = 0;
#pragma unroll
            for (int j = 0; j < KL; ++j) low |= ((*low_word<KL>(sl, lane, j) >> l) & 1u) << j;
            if (((code & 1u) && low < sp->sllo) || ((code & 2u) && low > sp->slhi)) return 0ull;
            ++*nchk;
        }
    }
    if constexpr (KP > 0) {
        const uint32_t code = (info >> 8) & 3u;
        if (code) {
            const uint32_t r = __funnelshift_r(*low_word<2>(sl, lane, 0), *low_word<2>(sl, lane, 1), (info >> 10) & 31u) &
                               (KP >= 32 ? 0xffffffffu : ((1u << KP) - 1u));
            if (((code & 1u) && r < sp->sllo) || ((code & 2u) && r > sp->slhi)) return 0ull;
            ++*nchk;
        }
        if (!has_g) return 0ull;
    }
    // bits of the hi word past the value's width are masked off, so a slot whose
    // value did not straddle (hi word not copied) reads harmless stale data
    const uint32_t v = (__funnelshift_r(sl[lane], sl[32 + lane], info & 31u) & gmask) + gbase;
    return (unsigned long long)v * sl[96 + lane];
}

// out4 = {SUM, |result|, |candidates|, |definite|} from every consumer warp's
// totals.  Without a workspace (rl_fin == 0) out4 was zeroed by the caller and
// each warp adds atomically; with one, each CTA writes its partials to
// rl_part[blockIdx] and the last CTA to arrive (ticket) sums them into out4
// and re-arms the ticket -- no memset before the launch.  Consumer warps only
// (the producer warp has exited): they meet at named barrier 1.
template <int NW>
__device__ __forceinline__ void finalize_out4(const SelParams& P, unsigned warp, unsigned lane,
                                              unsigned long long sum, unsigned long long c2, unsigned long long c0,
                                              unsigned long long c1) {
    constexpr int NT = NW * 32;
    if (!P.rl_fin) {   // out4 zeroed by the caller: one atomic per counter and warp
        if (lane == 0) {
            atomicAdd(P.out4 + 0, sum);
            atomicAdd(P.out4 + 1, c2);
            atomicAdd(P.out4 + 2, c0);
            atomicAdd(P.out4 + 3, c1);
        }
        return;
    }
    __shared__ unsigned long long red[NW][4];
    __shared__ uint32_t last;
    if (lane == 0) {
        red[warp][0] = sum;
        red[warp][1] = c2;
        red[warp][2] = c0;
        red[warp][3] = c1;
    }
    bar_sync(1, NT);
    if (threadIdx.x == 0) {
        unsigned long long t4[4] = {0, 0, 0, 0};
        for (int w = 0; w < NW; ++w)
            for (int i = 0; i < 4; ++i) t4[i] += red[w][i];
        if (P.rl_pdl) asm volatile("griddepcontrol.wait;" ::: "memory");   // the previous call is done with out4
        unsigned long long* part = P.rl_part + 4ull * blockIdx.x;
        for (int i = 0; i < 4; ++i) __stcg(part + i, t4[i]);
        __threadfence();
        last = atomicAdd(P.rl_ticket, 1u) == gridDim.x - 1 ? 1u : 0u;
    }
    bar_sync(1, NT);
    if (!last) return;
    __threadfence();
    unsigned long long t4[4] = {0, 0, 0, 0};
    for (uint32_t b = threadIdx.x; b < gridDim.x; b += NT)
        for (int i = 0; i < 4; ++i) t4[i] += __ldcg(P.rl_part + 4ull * b + i);
#pragma unroll
    for (int o = 16; o > 0; o >>= 1)
        for (int i = 0; i < 4; ++i) t4[i] += __shfl_xor_sync(0xffffffffu, t4[i], o);
    bar_sync(1, NT);
    if (lane == 0)
        for (int i = 0; i < 4; ++i) red[warp][i] = t4[i];
    bar_sync(1, NT);
    if (threadIdx.x == 0) {
        unsigned long long o4[4] = {0, 0, 0, 0};
        for (int w = 0; w < NW; ++w)
            for (int i = 0; i < 4; ++i) o4[i] += red[w][i];
        for (int i = 0; i < 4; ++i) P.out4[i] = o4[i];
        *P.rl_ticket = 0u;
    }
}

template <int NW, int BPT, int... WK>
__global__ void __launch_bounds__((NW + 1) * 32, 2) fused_rl_kernel(const __grid_constant__ SelParams P) {
    using S = typename ShapeOf<WK...>::type;
    constexpr int NT = NW * 32;
    // a split residual (one predicate SP): its high planes are in the stage, its KL low planes are
    // gathered with the aggregate for the rows they decide
    constexpr int SP = S::split(), KL = S::kl(), SPi = SP < 0 ? 0 : SP, SW = slot_words(KL);
    extern __shared__ __align__(128) unsigned char smem[];
    uint64_t* full = reinterpret_cast<uint64_t*>(smem);
    uint64_t* empty = full + P.nstages;
    long long* slot = reinterpret_cast<long long*>(empty + P.nstages);
    const size_t head_bytes = ((size_t)P.nstages * 24 + 127) & ~size_t(127);
    uint32_t* stages = reinterpret_cast<uint32_t*>(smem + head_bytes);
    const unsigned warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const uint32_t kRing = P.rl_ring, rmask = kRing - 1;
    uint2* ring = reinterpret_cast<uint2*>(stages + (size_t)P.nstages * P.stage_words) + warp * kRing;
    uint32_t* gs0 = reinterpret_cast<uint32_t*>(reinterpret_cast<uint2*>(stages + (size_t)P.nstages * P.stage_words) +
                                                NW * kRing);
    const uint32_t depth = P.rl_depth, dmask = depth - 1;   // gather passes in flight per warp (4 or 8)
    uint32_t* gs = gs0 + warp * (depth * SW);
    // shared-window addresses, converted once (the conversion is several instructions)
    const uint32_t gs_a = smem_u32(gs), full_a = smem_u32(full), empty_a = smem_u32(empty);
    if (threadIdx.x == 0) {
        for (uint32_t s = 0; s < P.nstages; ++s) {
            mbar_init(full + s, 1);
            mbar_init(empty + s, NW);
        }
        fence_mbar_init();
    }
    __syncthreads();
    if (warp == NW) {
        if (lane == 0) {
            if (P.rl_pdl == 1) asm volatile("griddepcontrol.wait;" ::: "memory");   // inputs may be in flight
            produce_ring(P, full, empty, slot, stages);
            // every tile of this CTA is loading: the next call in the stream may start its prologue
            if (P.rl_pdl) asm volatile("griddepcontrol.launch_dependents;" ::: "memory");
        }
        return;
    }

    const bool list = P.rl_list != 0;
    const bool direct = !list && P.nagg > 0;
    const AggCol& G = P.a[P.gidx];
    const uint32_t gmask = G.w >= 32 ? 0xffffffffu : ((1u << G.w) - 1u);
    uint32_t ncand = 0, ndef = 0, nres = 0, nchk = 0;
    unsigned long long sum = 0;
    uint32_t rhead = 0, rcnt = 0, gseq = 0;   // warp-uniform ring head / fill and gather passes issued

    // One gather pass over the `take` oldest ring entries (take <= 32).
    auto pass = [&](uint32_t take) {
        uint32_t* sl = gs + (gseq & dmask) * SW;
        const uint32_t sl_a = gs_a + (gseq & dmask) * (SW * 4);
        uint32_t info = 0u, f = 0u;
        if (lane < take) {
            const uint32_t ri = (rhead + lane) & rmask;
            const uint2 e = ring[ri];
            const uint64_t bit = (uint64_t)e.x * G.w;
            const uint32_t* src = G.major + (bit >> 5);
            const uint32_t sh = (uint32_t)(bit & 31);
            cp_async4_a(sl_a + lane * 4, src);
            if (sh + G.w > 32u) cp_async4_a(sl_a + (32 + lane) * 4, src + 1);
            info = 0x80000000u | sh;
            f = e.y;
            if constexpr (KL > 0) {
                // the check code rides in the top two bits of the factor (host: factors < 2^30)
                const uint32_t code = e.y >> 30;
                f = e.y & 0x3fffffffu;
                if (code) {   // an undecided row: its low residual planes travel with the aggregate
                    const uint32_t* lp = P.p[SPi].residual + split_lo_word(e.x >> 5, S::k(SPi), S::h(SPi));
                    if constexpr (KL == 4) {
                        cp_async16_a(sl_a + (kSlotWords + lane * 4) * 4, lp);
                    } else {
#pragma unroll
                        for (int j = 0; j < KL; ++j) cp_async4_a(sl_a + (kSlotWords + j * 32 + lane) * 4, lp + j);
                    }
                    info |= (code << 8) | ((e.x & 31u) << 10);
                }
            }
        }
        sl[64 + lane] = info;
        sl[96 + lane] = f;
        cp_async_commit();
        ++gseq;
        rhead += take;
        rcnt -= take;
        if (gseq >= depth) {   // sum the pass issued depth - 1 passes ago
            if (depth == 8)
                cp_async_wait<7>();
            else
                cp_async_wait<kDepth - 1>();
            sum += drain<KL>(gs + (gseq & dmask) * SW, lane, gmask, G.base, &P.p[SPi], &nchk);
        }
    };

    uint32_t s = 0, ph = 0;
    for (;; s = (s + 1 == P.nstages) ? (ph ^= 1u, 0u) : s + 1) {
        mbar_wait_a(full_a + 8 * s, ph, P.suspend_ns);
        const long long t = slot[s];
        if (t < 0) break;
        const uint32_t* stg = stages + (size_t)s * P.stage_words;
        if (P.debug == 7) {   // experiment: the TMA stream alone (no evaluation)
            __syncwarp();
            if (lane == 0) mbar_arrive_a(empty_a + 8 * s);
            continue;
        }
        const int64_t tile_r0 = t * (int64_t)P.tile_rows;
        const bool full_tile = tile_r0 + (int64_t)P.tile_rows <= P.n;

        // a3 + a5: candidate, definite and exact masks of this thread's blocks
        // result rows (incl. undecided ones); split residual: the undecided rows in the fine bucket
        // of the lower bound (k0) / of the upper bound (k1) -- the check code, bits 30 / 31 of the entry
        uint32_t xm[BPT], k0[BPT], k1[BPT];
#pragma unroll
        for (int b = 0; b < BPT; ++b) {
            const uint32_t blk = b * NT + threadIdx.x;
            const uint32_t vm = full_tile ? 0xffffffffu : valid_mask(tile_r0 + 32 * (int64_t)blk, P.n);
            uint32_t cm, dm, em, ul = 0u, uh = 0u;
            if constexpr (S::kDynamic)
                eval_block_dyn(P, stg, blk, vm, cm, dm, em);
            else
                eval_block<S, true>(P, stg, blk, vm, cm, dm, em, ul, uh);
            ncand += __popc(cm);
            ndef += __popc(dm);
            const uint32_t xk = em & (ul | uh);
            nres += __popc(em & ~xk);
            xm[b] = em;
            if constexpr (KL > 0) {
                k0[b] = xk & (ul | (0u - (P.p[SPi].scor & 1u)));
                k1[b] = xk & (uh | (0u - ((P.p[SPi].scor >> 1) & 1u)));
            } else {
                k0[b] = k1[b] = 0u;
            }
        }
        auto code_at = [&](int b, uint32_t l) -> uint32_t {   // check code << 30 of row l of block b
            if constexpr (KL > 0)
                return (((k0[b] >> l) & 1u) << 30) | (((k1[b] >> l) & 1u) << 31);
            else
                return 0u;
        };

        if (direct) {
            // a6 without gathers: every factor is a predicate column, its value is in the stage
#pragma unroll
            for (int b = 0; b < BPT; ++b) {
                const uint32_t blk = b * NT + threadIdx.x;
                for (uint32_t m = xm[b]; m; m &= m - 1) {
                    const uint32_t l = __ffs(m) - 1;
                    unsigned long long prod = 1;
                    for (int a = 0; a < P.nagg; ++a) {
                        uint32_t v = 0;
                        if constexpr (S::kDynamic) {
                            v = stage_value_dyn(P, stg, P.a[a].pred, blk, l);
                        } else {
                            static_for<S::N>([&](auto cc) {
                                constexpr int C = decltype(cc)::value;
                                if (C == P.a[a].pred) v = stage_value<S, C>(P, stg, blk, l);
                            });
                        }
                        prod *= v;
                    }
                    sum += prod;
                }
            }
        } else if (list) {
            // a6: queue (row, other factor) of every result row in the warp ring
            uint32_t my = 0;
#pragma unroll
            for (int b = 0; b < BPT; ++b) my += __popc(xm[b]);
            uint32_t incl = my;
#pragma unroll
            for (int o = 1; o < 32; o <<= 1) {
                const uint32_t y = __shfl_up_sync(0xffffffffu, incl, o);
                if (lane >= (unsigned)o) incl += y;
            }
            const uint32_t total = __shfl_sync(0xffffffffu, incl, 31);
            uint32_t e = incl - my;   // this thread's next entry, warp-relative
            for (uint32_t rb = 0; rb < total;) {
                // rounds only when the tile's results overflow the free part of the ring
                const uint32_t lim = min(total, rb + kRing - rcnt);
                const uint32_t wbase = rhead + rcnt - rb;
#pragma unroll
                for (int b = 0; b < BPT; ++b) {
                    if (xm[b] && e < lim) {
                        const uint32_t blk = b * NT + threadIdx.x;
                        const uint32_t row0 = (uint32_t)tile_r0 + blk * 32;
                        uint32_t m = xm[b];
                        if (P.rl_mpred < 0) {
                            do {
                                const uint32_t l = __ffs(m) - 1;
                                m &= m - 1;
                                ring[(wbase + e) & rmask] = make_uint2(row0 + l, 1u | code_at(b, l));
                                ++e;
                            } while (m && e < lim);
                        } else if constexpr (S::kDynamic) {
                            do {
                                const uint32_t l = __ffs(m) - 1;
                                m &= m - 1;
                                ring[(wbase + e) & rmask] = make_uint2(row0 + l, stage_value_dyn(P, stg, P.rl_mpred, blk, l));
                                ++e;
                            } while (m && e < lim);
                        } else {
                            static_for<S::N>([&](auto cc) {
                                constexpr int C = decltype(cc)::value;
                                constexpr int W = S::w(C), K = S::k(C);
                                if (C != P.rl_mpred) return;
                                uint32_t x[W];
                                lds_words<W>(x, stg + P.p[C].soff + blk * W);
                                if constexpr (S::h(C) > 0) return;   // never the split column (host-checked)
                                uint32_t r[K > 0 ? K : 1];
                                if constexpr (K > 0) lds_words<K>(r, stg + P.p[C].res_soff + blk * K);
                                do {
                                    const uint32_t l = __ffs(m) - 1;
                                    m &= m - 1;
                                    uint32_t v = row_bits<W>(x, l);
                                    if constexpr (K > 0) v = (v << K) | row_bits<K>(r, l);
                                    ring[(wbase + e) & rmask] = make_uint2(row0 + l, (v + P.p[C].base) | code_at(b, l));
                                    ++e;
                                } while (m && e < lim);
                            });
                        }
                        xm[b] = m;
                    }
                }
                __syncwarp();
                rcnt += lim - rb;
                rb = lim;
                if (rb < total) {   // ring full: make room before the next round
                    while (rcnt >= 32) pass(32);
                    __syncwarp();
                }
            }
        }
        __syncwarp();
        if (lane == 0) mbar_arrive_a(empty_a + 8 * s);   // the stage is no longer read
        if (list) {
            while (rcnt >= 32) pass(32);
            __syncwarp();
        }
    }
    if (list) {   // the ring's tail, then every pass still in flight
        while (rcnt > 0) pass(min(rcnt, 32u));
        cp_async_wait<0>();
        for (uint32_t g = gseq >= depth ? gseq - depth + 1 : 0; g < gseq; ++g)
            sum += drain<KL>(gs + (g & dmask) * SW, lane, gmask, G.base, &P.p[SPi], &nchk);
    }

    unsigned long long c0 = ncand, c1 = ndef, c2 = nres + nchk;
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) {
        sum += __shfl_xor_sync(0xffffffffu, sum, o);
        c0 += __shfl_xor_sync(0xffffffffu, c0, o);
        c1 += __shfl_xor_sync(0xffffffffu, c1, o);
        c2 += __shfl_xor_sync(0xffffffffu, c2, o);
    }
    finalize_out4<NW>(P, warp, lane, sum, c2, c0, c1);
}

// Two-phase one-pass kernel with gathered residuals ("rg"): the residual of a
// decomposed predicate is never streamed.  Phase A of tile t decides candidate
// and definite rows on the majors alone; definite rows are
// results at once (their whole bucket qualifies) and go to the
// result ring, and for every 32-row block that holds a non-definite candidate
// the block's K residual planes (K * 4 bytes of one sector, HBM or pinned host
// memory) are gathered into registers.  Phase B of tile t runs one tile later,
// when those loads have landed: the exact predicate on residual + major planes
// (the "+bw" concatenation; Alg. 2) keeps
// the non-definite candidates that qualify, and they join the ring.  A stage is
// released after its phase B, so the producer streams only major planes (Q6:
// 14 of the old 22 KB per 8192-row tile) and the residual traffic is the
// touched sectors only.  Factors of the SUM: one gathered bit-packed column
// times at most one k = 0 predicate column (ring), k = 0 predicate columns only
// (direct), or none (COUNT).
template <int NW, int BPT, int... WK>
__global__ void __launch_bounds__((NW + 1) * 32, 2) fused_rg_kernel(const __grid_constant__ SelParams P) {
    using S = Shape<WK...>;
    constexpr int NT = NW * 32;
    constexpr int KS = S::ksum();
    // a compiled split residual (predicate SP): rows its high planes leave undecided go to the ring as check
    // entries and their KL low planes are gathered with the aggregate (no synchronous gather)
    constexpr int SP = S::split(), KL = S::kl(), SPi = SP < 0 ? 0 : SP;
    // a bit-packed residual (predicate PC, k > 8, the query's only decomposed predicate): its non-definite
    // candidates go to the ring as check entries, their residual (1-2 words) gathered with the aggregate
    constexpr int PC = S::pk(), PCi = PC < 0 ? 0 : PC, KP = PC < 0 ? 0 : S::k(PCi);
    constexpr int CKi = SP >= 0 ? SPi : PCi;                  // the predicate whose check entries the ring holds
    constexpr bool kChk = KL > 0 || KP > 0;
    constexpr int SW = slot_words(KL > 0 ? KL : (KP > 0 ? 2 : 0));
    extern __shared__ __align__(128) unsigned char smem[];
    uint64_t* full = reinterpret_cast<uint64_t*>(smem);
    uint64_t* empty = full + P.nstages;
    long long* slot = reinterpret_cast<long long*>(empty + P.nstages);
    const size_t head_bytes = ((size_t)P.nstages * 24 + 127) & ~size_t(127);
    uint32_t* stages = reinterpret_cast<uint32_t*>(smem + head_bytes);
    const unsigned warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const uint32_t kRing = P.rl_ring, rmask = kRing - 1;
    uint2* ring = reinterpret_cast<uint2*>(stages + (size_t)P.nstages * P.stage_words) + warp * kRing;
    uint32_t* gs = reinterpret_cast<uint32_t*>(reinterpret_cast<uint2*>(stages + (size_t)P.nstages * P.stage_words) +
                                               NW * kRing) + warp * (kDepth * SW);
    if (threadIdx.x == 0) {
        for (uint32_t s = 0; s < P.nstages; ++s) {
            mbar_init(full + s, 1);
            mbar_init(empty + s, NW);
        }
        fence_mbar_init();
    }
    __syncthreads();
    if (warp == NW) {
        if (lane == 0) {
            if (P.rl_pdl == 1) asm volatile("griddepcontrol.wait;" ::: "memory");
            produce_ring(P, full, empty, slot, stages);
            if (P.rl_pdl) asm volatile("griddepcontrol.launch_dependents;" ::: "memory");
        }
        return;
    }

    const bool list = P.rl_list != 0;
    const bool direct = !list && P.nagg > 0;
    const bool cring = KP > 0 && P.nagg == 0;   // COUNT with packed check entries: a ring of check entries only
    const bool ring_on = list || cring;
    const AggCol& G = P.a[P.gidx];
    const uint32_t gmask = G.w >= 32 ? 0xffffffffu : ((1u << G.w) - 1u);
    uint32_t ncand = 0, ndef = 0, nres = 0, nchk = 0;
    unsigned long long sum = 0;
    uint32_t rhead = 0, rcnt = 0, gseq = 0;

    auto pass = [&](uint32_t take) {
        uint32_t* sl = gs + (gseq % kDepth) * SW;
        uint32_t info = 0u, f = 0u;
        if (lane < take) {
            const uint2 e = ring[(rhead + lane) & rmask];
            info = 0x80000000u;
            if (list) {
                const uint64_t bit = (uint64_t)e.x * G.w;
                const uint32_t* src = G.major + (bit >> 5);
                const uint32_t sh = (uint32_t)(bit & 31);
                cp_async4(sl + lane, src);
                if (sh + G.w > 32u) cp_async4(sl + 32 + lane, src + 1);
                info |= sh;
            }
            f = e.y;
            if constexpr (KP > 0) {
                const uint32_t code = e.y >> 30;   // check code (host: factors < 2^30)
                f = e.y & 0x3fffffffu;
                if (code) {   // the candidate's bit-packed residual: bits [row * KP, row * KP + KP)
                    const uint64_t rb = (uint64_t)e.x * KP;
                    const uint32_t* rp = P.p[PCi].residual + (rb >> 5);
                    const uint32_t rsh = (uint32_t)(rb & 31);
                    cp_async4(low_word<2>(sl, lane, 0), rp);
                    if (rsh + KP > 32u) cp_async4(low_word<2>(sl, lane, 1), rp + 1);
                    info |= (code << 8) | (rsh << 10);
                }
            }
            if constexpr (KL > 0) {
                const uint32_t code = e.y >> 30;   // check code (host: factors < 2^30)
                f = e.y & 0x3fffffffu;
                if (code) {
                    const uint32_t* lp = P.p[SPi].residual + split_lo_word(e.x >> 5, S::k(SPi), S::h(SPi));
                    if constexpr (KL == 4) {
                        cp_async16(low_word<KL>(sl, lane, 0), lp);
                    } else {
#pragma unroll
                        for (int j = 0; j < KL; ++j) cp_async4(low_word<KL>(sl, lane, j), lp + j);
                    }
                    info |= (code << 8) | ((e.x & 31u) << 10);
                }
            }
        }
        sl[64 + lane] = info;
        sl[96 + lane] = f;
        cp_async_commit();
        ++gseq;
        rhead += take;
        rcnt -= take;
        if (gseq >= (uint32_t)kDepth) {
            cp_async_wait<kDepth - 1>();
            sum += drain<KL, KP>(gs + (gseq % kDepth) * SW, lane, gmask, G.base, &P.p[CKi], &nchk, list);
        }
    };

    // a6 for the result rows xm[] of a tile held in stage `stg`; ck0 / ck1: rows of xm that are check
    // entries (split residual, list mode) in the fine bucket of the lower / upper bound
    auto consume = [&](const uint32_t* stg, int64_t tile_r0, uint32_t (&xm)[BPT], const uint32_t (&ck0)[BPT],
                       const uint32_t (&ck1)[BPT]) {
#pragma unroll
        for (int b = 0; b < BPT; ++b) nres += __popc(xm[b] & ~(ck0[b] | ck1[b]));   // check rows count when drained
        auto code_at = [&](int b, uint32_t l) -> uint32_t {   // check code << 30 of row l of block b
            if constexpr (kChk)
                return (((ck0[b] >> l) & 1u) << 30) | (((ck1[b] >> l) & 1u) << 31);
            else
                return 0u;
        };
        if (direct) {
#pragma unroll
            for (int b = 0; b < BPT; ++b) {
                const uint32_t blk = b * NT + threadIdx.x;
                for (uint32_t m = xm[b]; m; m &= m - 1) {
                    const uint32_t l = __ffs(m) - 1;
                    unsigned long long prod = 1;
                    for (int a = 0; a < P.nagg; ++a) {
                        uint32_t v = 0;
                        static_for<S::N>([&](auto cc) {
                            constexpr int C = decltype(cc)::value;
                            constexpr int W = S::w(C);
                            if constexpr (S::k(C) == 0) {
                                if (C == P.a[a].pred) {
                                    uint32_t x[W];
                                    lds_words<W>(x, stg + P.p[C].soff + blk * W);
                                    v = row_of<W>(x, l) + P.p[C].base;
                                }
                            }
                        });
                        prod *= v;
                    }
                    sum += prod;
                }
            }
            return;
        }
        if (!ring_on) return;
        uint32_t my = 0;
#pragma unroll
        for (int b = 0; b < BPT; ++b) my += __popc(xm[b]);
        uint32_t incl = my;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            const uint32_t y = __shfl_up_sync(0xffffffffu, incl, o);
            if (lane >= (unsigned)o) incl += y;
        }
        const uint32_t total = __shfl_sync(0xffffffffu, incl, 31);
        uint32_t e = incl - my;
        for (uint32_t rb = 0; rb < total;) {
            const uint32_t lim = min(total, rb + kRing - rcnt);
            const uint32_t wbase = rhead + rcnt - rb;
#pragma unroll
            for (int b = 0; b < BPT; ++b) {
                if (xm[b] && e < lim) {
                    const uint32_t blk = b * NT + threadIdx.x;
                    const uint32_t row0 = (uint32_t)tile_r0 + blk * 32;
                    uint32_t m = xm[b];
                    if (P.rl_mpred < 0) {
                        do {
                            const uint32_t l = __ffs(m) - 1;
                            m &= m - 1;
                            ring[(wbase + e) & rmask] = make_uint2(row0 + l, 1u | code_at(b, l));
                            ++e;
                        } while (m && e < lim);
                    } else {
                        static_for<S::N>([&](auto cc) {
                            constexpr int C = decltype(cc)::value;
                            constexpr int W = S::w(C);
                            if constexpr (S::k(C) == 0) {
                                if (C != P.rl_mpred) return;
                                uint32_t x[W];
                                lds_words<W>(x, stg + P.p[C].soff + blk * W);
                                do {
                                    const uint32_t l = __ffs(m) - 1;
                                    m &= m - 1;
                                    ring[(wbase + e) & rmask] =
                                        make_uint2(row0 + l, (row_bits<W>(x, l) + P.p[C].base) | code_at(b, l));
                                    ++e;
                                } while (m && e < lim);
                            }
                        });
                    }
                    xm[b] = m;
                }
            }
            __syncwarp();
            rcnt += lim - rb;
            rb = lim;
            if (rb < total) {
                while (rcnt >= 32) pass(32);
                __syncwarp();
            }
        }
    };

    uint32_t rres[BPT][KS > 0 ? KS : 1];   // residual words of the pending tile's blocks (in flight)
    uint32_t pnd[BPT];                      // its non-definite candidate masks
#pragma unroll
    for (int b = 0; b < BPT; ++b) pnd[b] = 0u;
    long long pt = -1;                      // pending tile (phase B not yet run), its stage
    uint32_t pst = 0;

    // Phase B of the pending tile: exact predicate on its non-definite candidates, results to the ring,
    // then its stage is released.
    auto phase_b = [&]() {
        const uint32_t* stg = stages + (size_t)pst * P.stage_words;
        const int64_t r0 = pt * (int64_t)P.tile_rows;
        uint32_t xm[BPT], xk0[BPT], xk1[BPT];
#pragma unroll
        for (int b = 0; b < BPT; ++b) {
            const uint32_t blk = b * NT + threadIdx.x;
            uint32_t em = pnd[b], u0 = 0u, u1 = 0u;
            if (em) {
                static_for<S::N>([&](auto cc) {
                    constexpr int C = decltype(cc)::value;
                    constexpr int W = S::w(C), K = S::k(C), KO = S::kofs(C);
                    if constexpr (K > 0 && S::h(C) > 0) {
                        // compiled split residual: the high planes (gathered in phase A) give the relaxation at
                        // granularity 2^(K-H); its definite rows are results, its undecided ones check entries
                        // whose code (fine bucket of lo / of hi) the pass turns into a low-plane gather
                        constexpr int H = S::h(C);
                        uint32_t x[W];
                        lds_words<W>(x, stg + P.p[C].soff + blk * W);
                        uint32_t fl = 0, fh = 0, gl = 0, gh = 0;
#pragma unroll
                        for (int j = K - H; j < K; ++j) {
                            fl = bsub(rres[b][KO + j], P.pmh[C][j - (K - H)][0], fl);
                            fh = brsub(rres[b][KO + j], P.pmh[C][j - (K - H)][1], fh);
                            gl = bsub(rres[b][KO + j], P.pmh[C][j - (K - H)][2], gl);
                            gh = brsub(rres[b][KO + j], P.pmh[C][j - (K - H)][3], gh);
                        }
#pragma unroll
                        for (int j = 0; j < W; ++j) {
                            fl = bsub(x[j], P.pmh[C][H + j][0], fl);
                            fh = brsub(x[j], P.pmh[C][H + j][1], fh);
                            gl = bsub(x[j], P.pmh[C][H + j][2], gl);
                            gh = brsub(x[j], P.pmh[C][H + j][3], gh);
                        }
                        em &= ~(fl | fh);
                        u0 = gl | (0u - (P.p[C].scor & 1u));
                        u1 = gh | (0u - ((P.p[C].scor >> 1) & 1u));
                        const uint32_t und = gl | gh;
                        u0 &= und;
                        u1 &= und;
                    } else if constexpr (K > 0 && K <= 8) {
                        uint32_t x[W];
                        lds_words<W>(x, stg + P.p[C].soff + blk * W);
                        const uint32_t H = P.p[C].rsplit;
                        uint32_t dp = 0u;
                        if (H) {
                            // split layout: the high planes (gathered in phase A) refine the bucket to 2^(k-h)
                            // values; rows decided there need no low planes, the rest gather them now
                            uint32_t cl = 0, ch = 0, dl = 0, dh = 0;
#pragma unroll
                            for (int j = 0; j < K; ++j) {
                                if (j < K - (int)H) continue;
                                const uint32_t i = j - (K - H);
                                cl = bsub(rres[b][KO + j], P.pmh[C][i][0], cl);
                                ch = brsub(rres[b][KO + j], P.pmh[C][i][1], ch);
                                dl = bsub(rres[b][KO + j], P.pmh[C][i][2], dl);
                                dh = brsub(rres[b][KO + j], P.pmh[C][i][3], dh);
                            }
#pragma unroll
                            for (int j = 0; j < W; ++j) {
                                cl = bsub(x[j], P.pmh[C][H + j][0], cl);
                                ch = brsub(x[j], P.pmh[C][H + j][1], ch);
                                dl = bsub(x[j], P.pmh[C][H + j][2], dl);
                                dh = brsub(x[j], P.pmh[C][H + j][3], dh);
                            }
                            dp = em & ~(dl | dh);
                            em &= ~(cl | ch) & (dl | dh);   // still undecided
                            const uint64_t gblk = (uint64_t)(r0 >> 5) + blk;
                            const uint32_t* lo = P.p[C].residual + split_lo_word(gblk, K, (int)H);
#pragma unroll
                            for (int j = 0; j < K; ++j) {
                                if (j >= K - (int)H) continue;
                                rres[b][KO + j] = P.p[C].res_hint ? ld_gather_if(lo + j, em != 0u)
                                                                  : ld_gather_if_nh(lo + j, em != 0u);
                            }
                        }
                        uint32_t el = 0, eh = 0;
#pragma unroll
                        for (int j = 0; j < K; ++j) {
                            el = bsub(rres[b][KO + j], P.pmx[C][j][0], el);
                            eh = brsub(rres[b][KO + j], P.pmx[C][j][1], eh);
                        }
#pragma unroll
                        for (int j = 0; j < W; ++j) {
                            el = bsub(x[j], P.pmx[C][K + j][0], el);
                            eh = brsub(x[j], P.pmx[C][K + j][1], eh);
                        }
                        em = dp | (em & ~(el | eh));
                    }
                });
            }
            xm[b] = em;
            xk0[b] = em & u0;
            xk1[b] = em & u1;
        }
        consume(stg, r0, xm, xk0, xk1);
        __syncwarp();
        if (lane == 0) mbar_arrive(empty + pst);
    };

    uint32_t zero[BPT];
#pragma unroll
    for (int b = 0; b < BPT; ++b) zero[b] = 0u;
    uint32_t s = 0, ph = 0;
    for (;; s = (s + 1 == P.nstages) ? (ph ^= 1u, 0u) : s + 1) {
        mbar_wait(full + s, ph, P.suspend_ns);
        const long long t = slot[s];
        if (t < 0) break;
        const uint32_t* stg = stages + (size_t)s * P.stage_words;
        const int64_t tile_r0 = t * (int64_t)P.tile_rows;
        const bool full_tile = tile_r0 + (int64_t)P.tile_rows <= P.n;

        // phase A (tile t): candidate / definite masks on the majors
        uint32_t dmk[BPT], ndm[BPT], ul_[BPT], uh_[BPT];
#pragma unroll
        for (int b = 0; b < BPT; ++b) {
            const uint32_t blk = b * NT + threadIdx.x;
            const uint32_t vm = full_tile ? 0xffffffffu : valid_mask(tile_r0 + 32 * (int64_t)blk, P.n);
            uint32_t cm, dm, em;
            uint32_t ul, uh;
            eval_block<S, false>(P, stg, blk, vm, cm, dm, em, ul, uh);
            ul_[b] = ul;
            uh_[b] = uh;
            ncand += __popc(cm);
            ndef += __popc(dm);
            dmk[b] = dm;
            ndm[b] = cm & ~dm;
        }
        if constexpr (KP > 0) {
            // bit-packed residual: definite rows are results, non-definite candidates check entries whose
            // code (bucket of lo / of hi) the pass turns into a residual gather (Alg. 2 on those rows only)
            uint32_t xm[BPT], k0[BPT], k1[BPT];
#pragma unroll
            for (int b = 0; b < BPT; ++b) {
                const uint32_t nd = ndm[b];
                k0[b] = nd & (ul_[b] | (0u - (P.p[PCi].scor & 1u)));
                k1[b] = nd & (uh_[b] | (0u - ((P.p[PCi].scor >> 1) & 1u)));
                xm[b] = cring ? nd : (dmk[b] | nd);
                if (cring) nres += __popc(dmk[b]);   // COUNT: definite rows never enter the ring
            }
            consume(stg, tile_r0, xm, k0, k1);
            __syncwarp();
            if (lane == 0) mbar_arrive(empty + s);
        } else if constexpr (KS > 0) {
            if (pt >= 0) phase_b();          // the previous tile's residual gathers have had a tile to land
            // gather the residual sectors of this tile's blocks with a non-definite candidate
#pragma unroll
            for (int b = 0; b < BPT; ++b) {
                const uint64_t gblk = (uint64_t)(tile_r0 >> 5) + b * NT + threadIdx.x;
                static_for<S::N>([&](auto cc) {
                    constexpr int C = decltype(cc)::value;
                    constexpr int K = S::k(C), KO = S::kofs(C);
                    if constexpr (K > 0 && K <= 8) {
                        const uint32_t H = P.p[C].rsplit;
                        if (H == 0) {
                            res_issue<K>(&rres[b][KO], P.p[C].residual, gblk, ndm[b] != 0u, P.p[C].res_hint != 0u);
                        } else {   // split layout: only the block's h high planes now
                            const uint32_t* hp = P.p[C].residual + split_hi_word(gblk, K, (int)H);
                            const bool hint = P.p[C].res_hint != 0u;
#pragma unroll
                            for (int j = 0; j < K; ++j) {
                                if (j < K - (int)H) continue;
                                const uint32_t* q = hp + (j - (K - H));
                                rres[b][KO + j] = hint ? ld_gather_if(q, ndm[b] != 0u) : ld_gather_if_nh(q, ndm[b] != 0u);
                            }
                        }
                    }
                });
                pnd[b] = ndm[b];
            }
            pt = t;
            pst = s;
            consume(stg, tile_r0, dmk, zero, zero);   // definite rows are results now
        } else {
            consume(stg, tile_r0, dmk, zero, zero);   // k = 0 everywhere: candidate = definite = exact
            __syncwarp();
            if (lane == 0) mbar_arrive(empty + s);
        }
        if (ring_on) {
            while (rcnt >= 32) pass(32);
            __syncwarp();
        }
    }
    if constexpr (KS > 0) {
        if (pt >= 0) phase_b();
    }
    if (ring_on) {
        while (rcnt > 0) pass(min(rcnt, 32u));
        cp_async_wait<0>();
        for (uint32_t g = gseq >= (uint32_t)kDepth ? gseq - kDepth + 1 : 0; g < gseq; ++g)
            sum += drain<KL, KP>(gs + (g % kDepth) * SW, lane, gmask, G.base, &P.p[CKi], &nchk, list);
    }

    unsigned long long c0 = ncand, c1 = ndef, c2 = nres + nchk;
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) {
        sum += __shfl_xor_sync(0xffffffffu, sum, o);
        c0 += __shfl_xor_sync(0xffffffffu, c0, o);
        c1 += __shfl_xor_sync(0xffffffffu, c1, o);
        c2 += __shfl_xor_sync(0xffffffffu, c2, o);
    }
    finalize_out4<NW>(P, warp, lane, sum, c2, c0, c1);
}

}  // namespace rl
}  // namespace ard

// ------------------------------------------------------------------------ host

namespace ar {

// Re-lay the stage for another tile size (setup_scan sized it for 8192 rows):
// each predicate's planes, then its streamed residual planes, tile_rows / 32
// words per plane.
void retile(ard::SelParams& P, uint32_t tile_rows) {
    if (P.tile_rows == tile_rows) return;
    P.tile_rows = tile_rows;
    uint32_t words = 0;
    for (int c = 0; c < P.npred; ++c) {
        P.p[c].soff = words;
        words += (tile_rows / 32) * P.p[c].w;
        if (P.p[c].res_stream) {   // residual planes (a split residual: its high planes)
            P.p[c].res_soff = words;
            words += (tile_rows / 32) * (P.p[c].rsplit ? P.p[c].rsplit : P.p[c].k);
        }
    }
    P.stage_words = std::max<uint32_t>(words, 4);
    P.num_tiles = (int64_t)ceil_div_u64((uint64_t)P.n, tile_rows);
}

namespace {

constexpr int WK(int w, int k) { return (w << 6) | k; }
constexpr int WKH(int w, int k, int h) { return (h << 12) | (w << 6) | k; }   // split residual, h planes streamed

// shape key of predicate c as the result-ring kernel sees it
inline int rl_key(const ard::SelPred& p) {
    if (!p.res_stream) return (int)(p.w << 6);
    return (int)((p.rsplit << 12) | (p.w << 6) | p.k);
}
// the predicate whose split residual is streamed (at most one), or -1; its low planes per row
inline int rl_split(const ard::SelParams& P, uint32_t* kl) {
    int sp = -1;
    *kl = 0;
    for (int c = 0; c < P.npred; ++c)
        if (P.p[c].res_stream && P.p[c].rsplit) {
            if (sp >= 0) return -2;
            sp = c;
            *kl = P.p[c].k - P.p[c].rsplit;
        }
    return sp;
}

struct RlFn {
    const void* fn;
    int nw;
    uint32_t tile_rows;
};


// (consumer warps, blocks per thread): AR_RL_CFG = 0/1/2/3/4/5 picks (8,1), (4,2),
// (2,4), (16,1), (4,1), (8,2); tile rows = NW * BPT * 1024.
template <int... Ws>
RlFn rl_pick(int cfg) {
    switch (cfg) {
        case 1: return {(const void*)ard::rl::fused_rl_kernel<4, 2, Ws...>, 4, 8192};
        case 2: return {(const void*)ard::rl::fused_rl_kernel<2, 4, Ws...>, 2, 8192};
        case 3: return {(const void*)ard::rl::fused_rl_kernel<16, 1, Ws...>, 16, 16384};
        case 4: return {(const void*)ard::rl::fused_rl_kernel<4, 1, Ws...>, 4, 4096};
        case 5: return {(const void*)ard::rl::fused_rl_kernel<8, 2, Ws...>, 8, 16384};
        default: return {(const void*)ard::rl::fused_rl_kernel<8, 1, Ws...>, 8, 8192};
    }
}

template <int... Ws>
RlFn rg_pick(int cfg) {
    switch (cfg) {
        case 1: return {(const void*)ard::rl::fused_rg_kernel<4, 2, Ws...>, 4, 8192};
        case 3: return {(const void*)ard::rl::fused_rg_kernel<16, 1, Ws...>, 16, 16384};
        case 4: return {(const void*)ard::rl::fused_rg_kernel<4, 1, Ws...>, 4, 4096};
        default: return {(const void*)ard::rl::fused_rg_kernel<8, 1, Ws...>, 8, 8192};
    }
}

template <int... Ws>
bool rl_match(const ard::SelParams& P) {
    constexpr int n = sizeof...(Ws);
    constexpr int wk[] = {Ws..., 0};
    if (P.npred != n) return false;
    for (int c = 0; c < n; ++c)
        if (rl_key(P.p[c]) != wk[c]) return false;
    return true;
}

// rg shapes: (w_major << 6) | k of every predicate, the residual gathered (SLICED, k <= 8); a split
// residual carries its h (<< 12) when its undecided rows can be check entries of the result ring (list
// mode, the other factor below 2^30; rg_split_ok), otherwise it is matched as unsplit (runtime h,
// synchronous low-plane gathers)
template <int... Ws>
bool rg_match(const ard::SelParams& P, bool split_ok) {
    constexpr int n = sizeof...(Ws);
    constexpr int wk[] = {Ws..., 0};
    if (P.npred != n) return false;
    for (int c = 0; c < n; ++c) {
        const uint32_t h = split_ok ? P.p[c].rsplit : 0u;
        if ((int)((h << 12) | (P.p[c].w << 6) | P.p[c].k) != wk[c]) return false;
    }
    return true;
}
// a bit-packed residual (k > 8) as check entries of the gathered-residual kernel: the query's only
// decomposed predicate, SUM through the result ring with the other factor below 2^30, or COUNT
inline bool rg_packed_ok(const ard::SelParams& P) {
    int nk = 0, np = 0;
    for (int c = 0; c < P.npred; ++c) {
        nk += P.p[c].k > 0 ? 1 : 0;
        np += (P.p[c].k > 8 && P.p[c].residual != nullptr) ? 1 : 0;
    }
    const bool mp_small =
        P.rl_mpred < 0 || (P.p[P.rl_mpred].base == 0 && P.p[P.rl_mpred].w + P.p[P.rl_mpred].k <= 30);
    return nk == 1 && np == 1 && ((P.rl_list && mp_small) || P.nagg == 0);
}
inline bool rg_split_ok(const ard::SelParams& P) {
    int ns = 0;
    for (int c = 0; c < P.npred; ++c) ns += P.p[c].rsplit ? 1 : 0;
    const bool mp_small =
        P.rl_mpred < 0 || (P.p[P.rl_mpred].base == 0 && P.p[P.rl_mpred].w + P.p[P.rl_mpred].k <= 30);
    return ns == 1 && P.rl_list && mp_small;
}

RlFn rg_find(const ard::SelParams& P, int cfg) {
    const bool sok = rg_split_ok(P);
#define AR_RG_TRY(...) \
    if (rg_match<__VA_ARGS__>(P, sok)) return rg_pick<__VA_ARGS__>(cfg);
    AR_RG_TRY(WKH(4, 8, 4), WK(4, 0), WK(6, 0))
    AR_RG_TRY(WKH(4, 8, 3), WK(4, 0), WK(6, 0))
    AR_RG_TRY(WKH(4, 8, 2), WK(4, 0), WK(6, 0))
#undef AR_RG_TRY
#define AR_RG_TRY(...) \
    if (rg_match<__VA_ARGS__>(P, false)) return rg_pick<__VA_ARGS__>(cfg);
    AR_RG_TRY(WK(4, 8), WK(4, 0), WK(6, 0))
    AR_RG_TRY(WK(24, 8))
    AR_RG_TRY(WK(24, 8), WK(24, 8))
#undef AR_RG_TRY
    // bit-packed residuals (C3 at M = 8 / 16 / 12, BASELINE configs[2]) as check entries
#define AR_RG_TRY(...) \
    if (pok && rg_match<__VA_ARGS__>(P, false)) return rg_pick<__VA_ARGS__>(cfg);
    const bool pok = rg_packed_ok(P);
    AR_RG_TRY(WK(8, 24))
    AR_RG_TRY(WK(16, 16))
    AR_RG_TRY(WK(12, 20))
#undef AR_RG_TRY
    return {nullptr, 0, 0};
}

// Decomposition shapes with a result-ring kernel: Q6 (l_shipdate 4 major + 8
// residual planes, l_discount 4, l_quantity 6), single 24/8 columns (C1, C3
// at M = 24), k = 0 single columns, and the two-column 24/8 spatial query.
RlFn rl_find(const ard::SelParams& P, int cfg) {
#define AR_RL_TRY(...) \
    if (rl_match<__VA_ARGS__>(P)) return rl_pick<__VA_ARGS__>(cfg);
    AR_RL_TRY(WK(4, 8), WK(4, 0), WK(6, 0))
    AR_RL_TRY(WKH(4, 8, 4), WK(4, 0), WK(6, 0))
    AR_RL_TRY(WKH(4, 8, 3), WK(4, 0), WK(6, 0))
    AR_RL_TRY(WKH(4, 8, 2), WK(4, 0), WK(6, 0))
    AR_RL_TRY(WK(24, 8))
    AR_RL_TRY(WK(8, 0))
    AR_RL_TRY(WK(16, 0))
    AR_RL_TRY(WK(24, 0))
    AR_RL_TRY(WK(32, 0))
    AR_RL_TRY(WK(24, 8), WK(24, 8))
#undef AR_RL_TRY
    // any other decomposition: the runtime-shape kernel (widths and bounds from the parameters;
    // not for streamed split residuals)
    static const bool no_dyn = getenv("AR_RL_NODYN") && atoi(getenv("AR_RL_NODYN"));
    uint32_t kl;
    if (!no_dyn && rl_split(P, &kl) == -1) return rl_pick<-1>(cfg);
    return {nullptr, 0, 0};
}

int env_cfg() {
    static const int v = [] {
        const char* e = getenv("AR_RL_CFG");
        return e ? atoi(e) : 0;
    }();
    return v;
}

int env_ring() {
    static const int v = [] {
        const char* e = getenv("AR_RL_RING");
        int r = e ? atoi(e) : ard::rl::kRingDefault;
        int p = 64;   // power of two in [64, 1024]
        while (p < r && p < 1024) p <<= 1;
        return p;
    }();
    return v;
}

size_t rl_smem_bytes(const ard::SelParams& P, uint32_t nstages, int nw, bool rg) {
    const size_t head = ((size_t)nstages * 24 + 127) & ~size_t(127);
    uint32_t kl = 0;
    if (!rg) {
        rl_split(P, &kl);
    } else if (rg_split_ok(P)) {   // a compiled split shape uses KL low-plane words per slot lane
        for (int c = 0; c < P.npred; ++c)
            if (P.p[c].rsplit) kl = P.p[c].k - P.p[c].rsplit;
    } else if (rg_packed_ok(P)) {   // packed check entries: two residual words per slot lane
        kl = 2;
    }
    return head + (size_t)nstages * P.stage_words * 4 + (size_t)nw * P.rl_ring * 8 +
           (size_t)nw * (rg ? ard::rl::kDepth : P.rl_depth) * ard::rl::slot_words((int)kl) * 4;
}

}  // namespace

// Launch the result-ring kernel if it applies (returns AR_OK and *launched);
// otherwise *launched = false and the caller takes fused_kernel.
ar_status launch_fused_rl(const ard::SelParams& P0, const ar_column* const* cols, void* ws, int pdl, bool* launched,
                          bool* gathered_res, cudaStream_t s) {
    *launched = false;
    *gathered_res = false;
    ard::SelParams P = P0;   // the caller's copy stays valid for fused_kernel
    P.rl_fin = ws ? 1 : 0;
    P.rl_pdl = ws ? pdl : 0;
    P.rl_ticket = ws ? (unsigned int*)ws : nullptr;
    P.rl_part = ws ? (unsigned long long*)((char*)ws + kSrsTicketBytes) : nullptr;
    static const bool off = getenv("AR_FUSED_LEGACY") && atoi(getenv("AR_FUSED_LEGACY"));
    // AR_RL_RESMODE: 0 (default) streamed-residual kernel where it applies, else the two-phase kernel
    // with gathered residuals; 2 gathered only
    static const int resmode = getenv("AR_RL_RESMODE") ? atoi(getenv("AR_RL_RESMODE")) : 0;
    if (off || P.n >= (int64_t)1 << 32) return AR_OK;
    // factors: none (COUNT), all predicate columns (direct), or one gathered bit-packed column
    // in device memory times at most one predicate column (result ring)
    int gathered = 0, g = -1, mp = -1;
    bool fac_k0 = true;   // every predicate-column factor has k = 0 (its value is in the major planes)
    for (int i = 0; i < P.nagg; ++i) {
        if (P.a[i].pred < 0) {
            ++gathered;
            g = i;
        } else {
            mp = P.a[i].pred;
            fac_k0 = fac_k0 && P.p[mp].k == 0;
        }
    }
    if (gathered > 1) return AR_OK;
    if (gathered == 1) {
        const ard::AggCol& a = P.a[g];
        if (a.k != 0 || a.layout != AR_LAYOUT_PACKED || a.w == 0 || cols[g]->d.major_loc != AR_LOC_DEVICE) return AR_OK;
        P.rl_list = 1;
        P.gidx = g;
        P.rl_mpred = P.nagg == 2 ? mp : -1;
    } else {
        P.rl_list = 0;
        P.rl_mpred = -1;
    }
    // the gathered-residual kernel: every decomposed predicate has a SLICED residual (k <= 8, HBM or
    // pinned host memory); factors as above with k = 0 predicate columns
    bool rg_ok = fac_k0;
    for (int c = 0; c < P.npred && rg_ok; ++c)
        if (P.p[c].k > 0)
            rg_ok = (P.p[c].rlayout & 0xffu) == AR_LAYOUT_SLICED && P.p[c].residual != nullptr && P.p[c].k <= 8;
    if (!rg_ok && fac_k0 && rg_packed_ok(P)) rg_ok = true;   // bit-packed residual: check entries
    RlFn k{nullptr, 0, 0};
    bool rg = false;
    // streamed residual planes first (device residuals: a stream of every block's planes beats
    // gathering the touched sectors, DESIGN s6.3c), the gathered-residual kernel otherwise (residuals
    // in pinned host memory, or the stream heuristic said no)
    // a streamed split residual needs the result ring (its undecided rows travel with the gathered
    // aggregate) and must not be the other SUM factor
    uint32_t kl = 0;
    const int sp = rl_split(P, &kl);
    // (the check code rides in the top bits of the other factor, so that factor must stay below 2^30)
    const bool mp_small = P.rl_mpred < 0 || (P.p[P.rl_mpred].base == 0 && P.p[P.rl_mpred].w + P.p[P.rl_mpred].k <= 30);
    const bool rl_ok = P.exact_mode != 0 && sp != -2 && (sp < 0 || (P.rl_list && P.rl_mpred != sp && mp_small));
    if (rl_ok && resmode != 2) k = rl_find(P, env_cfg());
    if (!k.fn && rg_ok) {
        ard::SelParams Q = P;
        // the .L2::64B prefetch-size hint on HBM residuals; over the host link AR_HOST_HINT (default 0)
        static const int host_hint = getenv("AR_HOST_HINT") ? atoi(getenv("AR_HOST_HINT")) : 0;
        for (int c = 0; c < Q.npred; ++c) {
            Q.p[c].res_stream = 0;
            Q.p[c].res_hint = (Q.p[c].res_host ? host_hint : 1) ? 1u : 0u;
        }
        k = rg_find(Q, env_cfg());
        if (k.fn) {
            P = Q;
            P.tile_rows = 0;   // force retile without residual planes
            rg = true;
        }
    }
    if (!k.fn) return AR_OK;
    retile(P, k.tile_rows);
    P.rl_ring = (uint32_t)env_ring();
    static const int depth_env = getenv("AR_RL_DEPTH") ? atoi(getenv("AR_RL_DEPTH")) : 4;
    P.rl_depth = depth_env == 8 ? 8u : 4u;

    // deepest stage ring (<= max_st) that keeps `want` CTAs per SM, else fewer CTAs with >= 2 stages
    static const int force_st = getenv("AR_STAGES") ? atoi(getenv("AR_STAGES")) : 0;
    static const int want_ctas = getenv("AR_RL_CTAS") ? atoi(getenv("AR_RL_CTAS")) : 2;
    // the result-ring kernel runs 3 stages (deeper rings measured slower at C4 / C2: the stream's extra
    // TMA requests delay the aggregate gathers, DESIGN s6.3); the two-phase kernel up to 8
    const uint32_t max_st = rg ? 8u : 3u;
    auto fit = [&](const RlFn& kk, const ard::SelParams& PP, int want, uint32_t* st_out, int* occ_out) {
        opt_in_max_smem(kk.fn);
        const int thr = (kk.nw + 1) * 32;
        *st_out = 0;
        *occ_out = 0;
        for (int target = std::max(want, 1); target >= 1 && !*st_out; --target)
            for (uint32_t st = force_st > 0 ? 8u : max_st; st >= 2; --st) {
                if (force_st > 0 && (int)st != force_st) continue;
                // the two-phase kernel holds two stages (phase B of tile t - 1 while tile t is decided)
                if (target >= 2 && st < (rg ? 4u : 3u) && force_st <= 0) break;
                int o = 0;
                cudaOccupancyMaxActiveBlocksPerMultiprocessor(&o, kk.fn, thr, rl_smem_bytes(PP, st, kk.nw, rg));
                if (o >= target) {
                    *st_out = st;
                    *occ_out = std::min(o, std::max(want, 1));
                    break;
                }
            }
        cudaGetLastError();
    };
    uint32_t stages = 0;
    int occ = 0;
    fit(k, P, want_ctas, &stages, &occ);
    // wide stages (e.g. a 24/8 column: 32 planes = 32 KB per 8192-row tile) leave one 8-warp CTA per SM:
    // then 4-warp CTAs on 4096-row tiles, as many as fit (C3 at M = 24: 0.495 vs 0.562 ms), unless
    // AR_RL_CFG chose the configuration
    if (!getenv("AR_RL_CFG") && occ < 2) {
        ard::SelParams P4 = P;
        const RlFn k4 = rg ? rg_find(P4, 4) : rl_find(P4, 4);
        if (k4.fn) {
            retile(P4, k4.tile_rows);
            uint32_t st4 = 0;
            int occ4 = 0;
            fit(k4, P4, 3, &st4, &occ4);
            // at equal resident warps the smaller tiles win too (two pipelines per SM, finer tail)
            if (st4 && occ4 * k4.nw >= occ * k.nw) {
                k = k4;
                P = P4;
                stages = st4;
                occ = occ4;
            }
        }
    }
    const int threads = (k.nw + 1) * 32;
    static const bool dbg = getenv("AR_DEBUG_LAUNCH") != nullptr;
    if (dbg)
        fprintf(stderr, "launch_fused_rl: %s nw=%d tile=%u stages=%u ctas/SM=%d smem=%zu\n", rg ? "rg" : "rl", k.nw,
                k.tile_rows, stages, occ, rl_smem_bytes(P, stages ? stages : 1, k.nw, rg));
    if (!stages) return AR_OK;
    P.nstages = stages;
    const int grid = (int)std::min<int64_t>(P.num_tiles, (int64_t)num_sms() * occ);
    if (ws && grid > kSrsMaxGrid) return AR_OK;
    void* args[] = {&P};
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = dim3(grid);
    cfg.blockDim = dim3(threads);
    cfg.dynamicSmemBytes = rl_smem_bytes(P, stages, k.nw, rg);
    cfg.stream = s;
    cudaLaunchAttribute attr[1];
    attr[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
    attr[0].val.programmaticStreamSerializationAllowed = P.rl_pdl ? 1 : 0;
    cfg.attrs = attr;
    cfg.numAttrs = 1;
    AR_TRY_CUDA(cudaLaunchKernelExC(&cfg, k.fn, args));
    *launched = true;
    *gathered_res = rg;
    return AR_OK;
}

}  // namespace ar

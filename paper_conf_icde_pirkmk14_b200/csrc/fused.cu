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
__device__ __forceinline__ void cp_async_commit() { asm volatile("cp.async.commit_group;" ::: "memory"); }
template <int N>
__device__ __forceinline__ void cp_async_wait() { asm volatile("cp.async.wait_group %0;" ::"n"(N) : "memory"); }

// Sum one landed gather slot: this lane's entry (a lane only reads what it copied).
__device__ __forceinline__ unsigned long long drain(const uint32_t* sl, uint32_t lane, uint32_t gmask,
                                                    uint32_t gbase) {
    const uint32_t info = sl[64 + lane];
    if (!(info >> 31)) return 0ull;
    // bits of the hi word past the value's width are masked off, so a slot whose
    // value did not straddle (hi word not copied) reads harmless stale data
    const uint32_t v = (__funnelshift_r(sl[lane], sl[32 + lane], info & 31u) & gmask) + gbase;
    return (unsigned long long)v * sl[96 + lane];
}

template <int NW, int BPT, int... WK>
__global__ void __launch_bounds__((NW + 1) * 32, 2) fused_rl_kernel(const __grid_constant__ SelParams P) {
    using S = Shape<WK...>;
    constexpr int NT = NW * 32;
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
                                               NW * kRing) + warp * (kDepth * kSlotWords);
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
    uint32_t ncand = 0, ndef = 0, nres = 0;
    unsigned long long sum = 0;
    uint32_t rhead = 0, rcnt = 0, gseq = 0;   // warp-uniform ring head / fill and gather passes issued

    // One gather pass over the `take` oldest ring entries (take <= 32).
    auto pass = [&](uint32_t take) {
        uint32_t* sl = gs + (gseq % kDepth) * kSlotWords;
        uint32_t info = 0u, f = 0u;
        if (lane < take) {
            const uint2 e = ring[(rhead + lane) & rmask];
            const uint64_t bit = (uint64_t)e.x * G.w;
            const uint32_t* src = G.major + (bit >> 5);
            const uint32_t sh = (uint32_t)(bit & 31);
            cp_async4(sl + lane, src);
            if (sh + G.w > 32u) cp_async4(sl + 32 + lane, src + 1);
            info = 0x80000000u | sh;
            f = e.y;
        }
        sl[64 + lane] = info;
        sl[96 + lane] = f;
        cp_async_commit();
        ++gseq;
        rhead += take;
        rcnt -= take;
        if (gseq >= (uint32_t)kDepth) {   // sum the pass issued kDepth - 1 passes ago
            cp_async_wait<kDepth - 1>();
            sum += drain(gs + (gseq % kDepth) * kSlotWords, lane, gmask, G.base);
        }
    };

    uint32_t s = 0, ph = 0;
    for (;; s = (s + 1 == P.nstages) ? (ph ^= 1u, 0u) : s + 1) {
        mbar_wait(full + s, ph, P.suspend_ns);
        const long long t = slot[s];
        if (t < 0) break;
        const uint32_t* stg = stages + (size_t)s * P.stage_words;
        if (P.debug == 7) {   // experiment: the TMA stream alone (no evaluation)
            __syncwarp();
            if (lane == 0) mbar_arrive(empty + s);
            continue;
        }
        const int64_t tile_r0 = t * (int64_t)P.tile_rows;
        const bool full_tile = tile_r0 + (int64_t)P.tile_rows <= P.n;

        // a3 + a5: candidate, definite and exact masks of this thread's blocks
        uint32_t xm[BPT];
#pragma unroll
        for (int b = 0; b < BPT; ++b) {
            const uint32_t blk = b * NT + threadIdx.x;
            const uint32_t vm = full_tile ? 0xffffffffu : valid_mask(tile_r0 + 32 * (int64_t)blk, P.n);
            uint32_t cm, dm, em;
            eval_block<S, true>(P, stg, blk, vm, cm, dm, em);
            ncand += __popc(cm);
            ndef += __popc(dm);
            nres += __popc(em);
            xm[b] = em;
        }

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
                        static_for<S::N>([&](auto cc) {
                            constexpr int C = decltype(cc)::value;
                            if (C == P.a[a].pred) v = stage_value<S, C>(P, stg, blk, l);
                        });
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
                                ring[(wbase + e) & rmask] = make_uint2(row0 + l, 1u);
                                ++e;
                            } while (m && e < lim);
                        } else {
                            static_for<S::N>([&](auto cc) {
                                constexpr int C = decltype(cc)::value;
                                constexpr int W = S::w(C), K = S::k(C);
                                if (C != P.rl_mpred) return;
                                uint32_t x[W];
                                lds_words<W>(x, stg + P.p[C].soff + blk * W);
                                uint32_t r[K > 0 ? K : 1];
                                if constexpr (K > 0) lds_words<K>(r, stg + P.p[C].res_soff + blk * K);
                                do {
                                    const uint32_t l = __ffs(m) - 1;
                                    m &= m - 1;
                                    uint32_t v = row_of<W>(x, l);
                                    if constexpr (K > 0) v = (v << K) | row_of<K>(r, l);
                                    ring[(wbase + e) & rmask] = make_uint2(row0 + l, v + P.p[C].base);
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
        if (lane == 0) mbar_arrive(empty + s);   // the stage is no longer read
        if (list) {
            while (rcnt >= 32) pass(32);
            __syncwarp();
        }
    }
    if (list) {   // the ring's tail, then every pass still in flight
        while (rcnt > 0) pass(min(rcnt, 32u));
        cp_async_wait<0>();
        for (uint32_t g = gseq >= (uint32_t)kDepth ? gseq - kDepth + 1 : 0; g < gseq; ++g)
            sum += drain(gs + (g % kDepth) * kSlotWords, lane, gmask, G.base);
    }

    unsigned long long c0 = ncand, c1 = ndef, c2 = nres;
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) {
        sum += __shfl_xor_sync(0xffffffffu, sum, o);
        c0 += __shfl_xor_sync(0xffffffffu, c0, o);
        c1 += __shfl_xor_sync(0xffffffffu, c1, o);
        c2 += __shfl_xor_sync(0xffffffffu, c2, o);
    }
    if (!P.rl_fin) {   // out4 zeroed by the caller: one atomic per counter and warp
        if (lane == 0) {
            atomicAdd(P.out4 + 0, sum);
            atomicAdd(P.out4 + 1, c2);
            atomicAdd(P.out4 + 2, c0);
            atomicAdd(P.out4 + 3, c1);
        }
        return;
    }
    // Workspace finalize (no memset before the launch): CTA partial -> rl_part[blockIdx]; the last
    // CTA to arrive (ticket) sums all partials into out4 and re-arms the ticket.  Consumer warps
    // only: the producer warp has exited, so they meet at named barrier 1.
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
        if (P.p[c].res_stream) {
            P.p[c].res_soff = words;
            words += (tile_rows / 32) * P.p[c].k;
        }
    }
    P.stage_words = std::max<uint32_t>(words, 4);
    P.num_tiles = (int64_t)ceil_div_u64((uint64_t)P.n, tile_rows);
}

namespace {

constexpr int WK(int w, int k) { return (w << 6) | k; }

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
bool rl_match(const ard::SelParams& P) {
    constexpr int n = sizeof...(Ws);
    constexpr int wk[] = {Ws..., 0};
    if (P.npred != n) return false;
    for (int c = 0; c < n; ++c) {
        const uint32_t k = P.p[c].res_stream ? P.p[c].k : 0u;
        if ((int)((P.p[c].w << 6) | k) != wk[c]) return false;
    }
    return true;
}

// Decomposition shapes with a result-ring kernel: Q6 (l_shipdate 4 major + 8
// residual planes, l_discount 4, l_quantity 6), single 24/8 columns (C1, C3
// at M = 24), k = 0 single columns, and the two-column 24/8 spatial query.
RlFn rl_find(const ard::SelParams& P, int cfg) {
#define AR_RL_TRY(...) \
    if (rl_match<__VA_ARGS__>(P)) return rl_pick<__VA_ARGS__>(cfg);
    AR_RL_TRY(WK(4, 8), WK(4, 0), WK(6, 0))
    AR_RL_TRY(WK(24, 8))
    AR_RL_TRY(WK(8, 0))
    AR_RL_TRY(WK(16, 0))
    AR_RL_TRY(WK(24, 0))
    AR_RL_TRY(WK(32, 0))
    AR_RL_TRY(WK(24, 8), WK(24, 8))
#undef AR_RL_TRY
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

size_t rl_smem_bytes(const ard::SelParams& P, uint32_t nstages, int nw) {
    const size_t head = ((size_t)nstages * 24 + 127) & ~size_t(127);
    return head + (size_t)nstages * P.stage_words * 4 + (size_t)nw * P.rl_ring * 8 +
           (size_t)nw * ard::rl::kDepth * ard::rl::kSlotWords * 4;
}

}  // namespace

// Launch the result-ring kernel if it applies (returns AR_OK and *launched);
// otherwise *launched = false and the caller takes fused_kernel.
ar_status launch_fused_rl(const ard::SelParams& P0, const ar_column* const* cols, void* ws, int pdl, bool* launched,
                          cudaStream_t s) {
    *launched = false;
    ard::SelParams P = P0;   // the caller's copy stays valid for fused_kernel
    P.rl_fin = ws ? 1 : 0;
    P.rl_pdl = ws ? pdl : 0;
    P.rl_ticket = ws ? (unsigned int*)ws : nullptr;
    P.rl_part = ws ? (unsigned long long*)((char*)ws + kSrsTicketBytes) : nullptr;
    static const bool off = getenv("AR_FUSED_LEGACY") && atoi(getenv("AR_FUSED_LEGACY"));
    if (off || !P.exact_mode || P.n >= (int64_t)1 << 32) return AR_OK;
    // factors: none (COUNT), all predicate columns (direct), or one gathered bit-packed column
    // in device memory times at most one predicate column (result ring)
    int gathered = 0, g = -1, mp = -1;
    for (int i = 0; i < P.nagg; ++i) {
        if (P.a[i].pred < 0) {
            ++gathered;
            g = i;
        } else {
            mp = P.a[i].pred;
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
    const RlFn k = rl_find(P, env_cfg());
    if (!k.fn) return AR_OK;
    retile(P, k.tile_rows);
    P.rl_ring = (uint32_t)env_ring();

    // deepest stage ring (<= 8, >= 3) that keeps 2 CTAs per SM, else 1 CTA with >= 2 stages
    opt_in_max_smem(k.fn);
    const int threads = (k.nw + 1) * 32;
    uint32_t stages = 0;
    int occ = 0;
    static const int force_st = getenv("AR_STAGES") ? atoi(getenv("AR_STAGES")) : 0;
    static const int want_ctas = getenv("AR_RL_CTAS") ? atoi(getenv("AR_RL_CTAS")) : 2;
    for (int target = std::max(want_ctas, 1); target >= 1 && !stages; --target)
        for (uint32_t st = 8; st >= 2; --st) {
            if (force_st > 0 && (int)st != force_st) continue;
            if (target >= 2 && st < 3 && force_st <= 0) break;
            int o = 0;
            cudaOccupancyMaxActiveBlocksPerMultiprocessor(&o, k.fn, threads, rl_smem_bytes(P, st, k.nw));
            if (o >= target) {
                stages = st;
                occ = o;
                break;
            }
        }
    cudaGetLastError();
    if (!stages) return AR_OK;
    P.nstages = stages;
    const int grid = (int)std::min<int64_t>(P.num_tiles, (int64_t)num_sms() * std::min(occ, std::max(want_ctas, 1)));
    if (ws && grid > kSrsMaxGrid) return AR_OK;
    void* args[] = {&P};
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = dim3(grid);
    cfg.blockDim = dim3(threads);
    cfg.dynamicSmemBytes = rl_smem_bytes(P, stages, k.nw);
    cfg.stream = s;
    cudaLaunchAttribute attr[1];
    attr[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
    attr[0].val.programmaticStreamSerializationAllowed = P.rl_pdl ? 1 : 0;
    cfg.attrs = attr;
    cfg.numAttrs = 1;
    AR_TRY_CUDA(cudaLaunchKernelExC(&cfg, k.fn, args));
    *launched = true;
    return AR_OK;
}

}  // namespace ar

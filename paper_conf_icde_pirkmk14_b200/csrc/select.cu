// select.cu -- step a3: approximate selection + stable compaction over SLICED
// majors (s IV-B), and the general one-pass A&R kernel
// (a3 + a5 + a6) for shapes the result-ring kernel (fused.cu) does not cover.
//
// Every range predicate is evaluated on the bit planes with borrow chains: per
// plane and per bound one 3-input logic op decides 32 rows at once (DESIGN
// s6.2).  Like the paper's operators, which are JIT-generated per data type and
// decomposition, the kernels are specialised on the
// decomposition: FixedPlanes<BPT, W...> holds the thread's planes in registers
// with compile-time widths (tight, unrolled code); DynPlanes<BPT> is the
// generic runtime-width path for any other shape.
//
// select_tile_kernel + compact_kernel: one 8192-row tile per CTA (one TMA bulk
// copy per predicate), stable compaction into the tile's workspace slice, then
// one warp per tile moves the slice to its final offset (no CTA waits on
// another CTA; DESIGN s6.2 lists the measured alternatives).
//
// fused_kernel: persistent CTAs, one producer warp streaming tiles into a ring
// of shared-memory stages (produce_ring), consumer warps compacting candidates
// into per-warp lists in shared memory; non-definite candidates are refined in
// place, the SUM factors of the exact rows gathered asynchronously.
#include <type_traits>

#include "rl_common.cuh"

namespace ard {

// ------------------------------------------------------------ bit-plane tests

// For one 32-row block with W planes x[0..W) (x[j] = bit j of the 32 values,
// LSB first), lo <= v <= hi is decided by two borrow chains run from the LSB:
// v < lo iff v - lo borrows out of the top bit, v > hi iff hi - v does.  Per
// plane and bound the borrow update is one 3-input logic op (LOP3); the bound's
// bit j is a warp-uniform all-0 / all-1 mask.
// Written as explicit lop3 (immLut = F(0xF0, 0xCC, 0xAA)): left to itself the
// compiler splits each into three LOP3s.
__device__ __forceinline__ uint32_t borrow_sub(uint32_t x, uint32_t cbit, uint32_t b) {   // borrow of x - c
    uint32_t d;   // (~x & (c | b)) | (x & c & b)
    asm("lop3.b32 %0, %1, %2, %3, 0x8E;" : "=r"(d) : "r"(x), "r"(cbit), "r"(b));
    return d;
}
__device__ __forceinline__ uint32_t borrow_rsub(uint32_t x, uint32_t cbit, uint32_t b) {  // borrow of c - x
    uint32_t d;   // (~c & (x | b)) | (c & x & b)
    asm("lop3.b32 %0, %1, %2, %3, 0xB2;" : "=r"(d) : "r"(x), "r"(cbit), "r"(b));
    return d;
}
__device__ __forceinline__ uint32_t bitmask(uint32_t v, uint32_t j) { return 0u - ((v >> j) & 1u); }

// Bound bits come as precomputed all-0 / all-1 words from the kernel parameters
// (pm[plane][0..3] = candidate lo / hi, definite lo / hi), so with compile-time
// plane indices each LOP3 takes its bound straight from the constant bank.
template <int W, int O, int LO, int HI>
__device__ __forceinline__ uint32_t range_mask_pm(const uint32_t* x, const SelParams& P) {
    uint32_t bl = 0, bh = 0;
#pragma unroll
    for (int j = 0; j < W; ++j) {
        bl = borrow_sub(x[j], P.pm[O + j][LO], bl);
        bh = borrow_rsub(x[j], P.pm[O + j][HI], bh);
    }
    return ~(bl | bh);
}

// Major of row l (0..31) of a block from its bit planes in shared memory.
__device__ __forceinline__ uint32_t plane_value(const uint32_t* pl, uint32_t w, uint32_t l) {
    uint32_t m = 0;
    for (uint32_t j = 0; j < w; ++j) m |= ((pl[j] >> l) & 1u) << j;
    return m;
}

// ------------------------------------------------------------ plane sources

template <int I>
using ic = std::integral_constant<int, I>;
template <int N, int I = 0, class F>
__device__ __forceinline__ void static_for(F&& f) {
    if constexpr (I < N) {
        f(ic<I>{});
        static_for<N, I + 1>(f);
    }
}


template <int... Ws>
__host__ __device__ constexpr int wid(int c) {
    constexpr int a[] = {Ws..., 0};
    return a[c];
}
template <int... Ws>
__host__ __device__ constexpr int woff(int c) {
    constexpr int a[] = {Ws..., 0};
    int o = 0;
    for (int i = 0; i < c; ++i) o += a[i];
    return o;
}

// Compile-time decomposition shape: the thread's planes live in registers.
template <int BPT, int... Ws>
struct FixedPlanes {
    static constexpr int N = sizeof...(Ws);
    static constexpr int TOTAL = (0 + ... + Ws);
    // shape ops: compile-time predicate loop and widths
    template <class F>
    __device__ __forceinline__ static void for_pred(const SelParams&, F&& f) {
        static_for<N>(f);
    }
    template <int C>
    __device__ __forceinline__ static constexpr uint32_t pw(const SelParams&, std::integral_constant<int, C>) {
        return (uint32_t)wid<Ws...>(C);
    }
    uint32_t x[BPT][TOTAL > 0 ? TOTAL : 1];

    template <int C>
    __device__ __forceinline__ void load_c(const SelParams& P, const uint32_t* stg) {
        if constexpr (C < N) {
            constexpr int w = wid<Ws...>(C), o = woff<Ws...>(C);
            const uint32_t* pl = stg + P.p[C].soff + threadIdx.x * (BPT * w);
            if constexpr ((BPT * w) % 4 == 0) {
#pragma unroll
                for (int q = 0; q < BPT * w / 4; ++q) {
                    const uint4 v = reinterpret_cast<const uint4*>(pl)[q];
                    const uint32_t vv[4] = {v.x, v.y, v.z, v.w};
#pragma unroll
                    for (int e = 0; e < 4; ++e) x[(4 * q + e) / w][o + (4 * q + e) % w] = vv[e];
                }
            } else {
#pragma unroll
                for (int b = 0; b < BPT; ++b)
#pragma unroll
                    for (int j = 0; j < w; ++j) x[b][o + j] = pl[b * w + j];
            }
            load_c<C + 1>(P, stg);
        }
    }
    __device__ __forceinline__ void load(const SelParams& P, const uint32_t* stg) { load_c<0>(P, stg); }

    template <int C>
    __device__ __forceinline__ void eval_c(const SelParams& P, uint32_t (&cm)[BPT], uint32_t (&dm)[BPT]) const {
        if constexpr (C < N) {
            constexpr int w = wid<Ws...>(C), o = woff<Ws...>(C);
            const SelPred& p = P.p[C];
#pragma unroll
            for (int b = 0; b < BPT; ++b) {
                const uint32_t c = range_mask_pm<w, o, 0, 1>(&x[b][o], P);
                cm[b] &= c;
                if (p.mode == 0)
                    dm[b] &= c;
                else if (p.mode == 1)
                    dm[b] &= range_mask_pm<w, o, 2, 3>(&x[b][o], P);
                else
                    dm[b] = 0;
            }
            eval_c<C + 1>(P, cm, dm);
        }
    }
    __device__ __forceinline__ void eval(const SelParams& P, uint32_t (&cm)[BPT], uint32_t (&dm)[BPT]) const {
        eval_c<0>(P, cm, dm);
    }

    // Exact predicate (Alg. 2 on the planes): for each decomposed predicate whose
    // residual planes are in the stage, one borrow chain over the k residual
    // planes then the w major planes -- the bitwise concatenation "+bw" of the
    // approximation and the residual -- against the exact bounds.  xm &= result.
    template <int C, int K>
    __device__ __forceinline__ void exact_k(const SelParams& P, const uint32_t* stg, uint32_t (&xm)[BPT]) const {
        constexpr int w = wid<Ws...>(C), o = woff<Ws...>(C);
        const SelPred& p = P.p[C];
#pragma unroll
        for (int b = 0; b < BPT; ++b) {
            const uint32_t* rp = stg + p.res_soff + (threadIdx.x * BPT + b) * K;
            uint32_t r[K];
            if constexpr (K % 4 == 0) {   // 16-B aligned: k = 4, 8
#pragma unroll
                for (int q = 0; q < K / 4; ++q) {
                    const uint4 v = reinterpret_cast<const uint4*>(rp)[q];
                    r[4 * q] = v.x; r[4 * q + 1] = v.y; r[4 * q + 2] = v.z; r[4 * q + 3] = v.w;
                }
            } else {
#pragma unroll
                for (int j = 0; j < K; ++j) r[j] = rp[j];
            }
            uint32_t bl = 0, bh = 0;
#pragma unroll
            for (int j = 0; j < K; ++j) {
                bl = borrow_sub(r[j], P.pmx[C][j][0], bl);
                bh = borrow_rsub(r[j], P.pmx[C][j][1], bh);
            }
#pragma unroll
            for (int j = 0; j < w; ++j) {
                bl = borrow_sub(x[b][o + j], P.pmx[C][K + j][0], bl);
                bh = borrow_rsub(x[b][o + j], P.pmx[C][K + j][1], bh);
            }
            xm[b] &= ~(bl | bh);
        }
    }
    // Exact predicate (Alg. 2 on the planes): for each decomposed predicate whose
    // residual planes are in the stage, one borrow chain over the k residual
    // planes then the w major planes -- the bitwise concatenation "+bw" of the
    // approximation and the residual -- against the exact bounds.  xm &= result.
    template <int C = 0>
    __device__ __forceinline__ void exact(const SelParams& P, const uint32_t* stg, uint32_t (&xm)[BPT]) const {
        if constexpr (C < N) {
            if (P.p[C].res_stream) {
                switch (P.p[C].k) {   // residual planes are only streamed for k <= 8
                    case 1: exact_k<C, 1>(P, stg, xm); break;
                    case 2: exact_k<C, 2>(P, stg, xm); break;
                    case 3: exact_k<C, 3>(P, stg, xm); break;
                    case 4: exact_k<C, 4>(P, stg, xm); break;
                    case 5: exact_k<C, 5>(P, stg, xm); break;
                    case 6: exact_k<C, 6>(P, stg, xm); break;
                    case 7: exact_k<C, 7>(P, stg, xm); break;
                    default: exact_k<C, 8>(P, stg, xm); break;
                }
            }
            exact<C + 1>(P, stg, xm);
        }
    }

    // major of predicate C at row l of block B
    template <int B, int C>
    __device__ __forceinline__ uint32_t value(uint32_t l) const {
        constexpr int w = wid<Ws...>(C), o = woff<Ws...>(C);
        uint32_t m = 0;
#pragma unroll
        for (int j = 0; j < w; ++j) m |= ((x[B][o + j] >> l) & 1u) << j;
        return m;
    }
    template <int B, int C = 0>
    __device__ __forceinline__ uint32_t value_rt(int c, uint32_t l) const {
        if constexpr (C < N) {
            if (c == C) return value<B, C>(l);
            return value_rt<B, C + 1>(c, l);
        } else {
            return 0u;
        }
    }
    // approximation tuple of row l of tile-block blk, read from the stage (lane-parallel pass)
    template <int C = 0>
    __device__ __forceinline__ static uint32_t appr_smem(const SelParams& P, const uint32_t* stg, uint32_t blk,
                                                         uint32_t l) {
        if constexpr (C < N) {
            constexpr int w = wid<Ws...>(C), o = woff<Ws...>(C);
            uint32_t x[w];   // the block's planes: vector loads (a block starts at a multiple of w words)
            rl::lds_words<w>(x, stg + P.p[C].soff + blk * w);
            return (rl::row_bits<w>(x, l) << o) | appr_smem<C + 1>(P, stg, blk, l);
        } else {
            return 0u;
        }
    }
    // approximation tuple: all majors concatenated LSB-first in predicate order
    template <int B>
    __device__ __forceinline__ uint32_t appr(const SelParams&, uint32_t l) const {
        return rl::row_bits<TOTAL>(x[B], l);
    }
};

// Runtime decomposition shape: planes stay in shared memory.
template <int BPT>
struct DynPlanes {
    const uint32_t* stg;
    template <class F>
    __device__ __forceinline__ static void for_pred(const SelParams& P, F&& f) {
        for (int c = 0; c < P.npred; ++c) f(c);
    }
    __device__ __forceinline__ static uint32_t pw(const SelParams& P, int c) { return P.p[c].w; }

    __device__ __forceinline__ void load(const SelParams&, const uint32_t* s) { stg = s; }

    __device__ __forceinline__ void eval(const SelParams& P, uint32_t (&cm)[BPT], uint32_t (&dm)[BPT]) const {
        for (int c = 0; c < P.npred; ++c) {
            const SelPred& p = P.p[c];
            const uint32_t w = p.w;
            const uint32_t* pl = stg + p.soff + threadIdx.x * BPT * w;
            uint32_t cl[BPT], ch[BPT], dl[BPT], dh[BPT];
#pragma unroll
            for (int b = 0; b < BPT; ++b) cl[b] = ch[b] = dl[b] = dh[b] = 0;
            for (uint32_t j = 0; j < w; ++j) {
                const uint32_t L = bitmask(p.clo, j), H = bitmask(p.chi, j);
                const uint32_t DL = bitmask(p.dlo, j), DH = bitmask(p.dhi, j);
#pragma unroll
                for (int b = 0; b < BPT; ++b) {
                    const uint32_t x = pl[b * w + j];
                    cl[b] = borrow_sub(x, L, cl[b]);
                    ch[b] = borrow_rsub(x, H, ch[b]);
                    dl[b] = borrow_sub(x, DL, dl[b]);
                    dh[b] = borrow_rsub(x, DH, dh[b]);
                }
            }
#pragma unroll
            for (int b = 0; b < BPT; ++b) {
                const uint32_t c0 = ~(cl[b] | ch[b]);
                cm[b] &= c0;
                dm[b] = p.mode == 0 ? (dm[b] & c0) : (p.mode == 1 ? (dm[b] & ~(dl[b] | dh[b])) : 0u);
            }
        }
    }
    __device__ __forceinline__ void exact(const SelParams& P, const uint32_t* s, uint32_t (&xm)[BPT]) const {
        for (int c = 0; c < P.npred; ++c) {
            const SelPred& p = P.p[c];
            if (!p.res_stream) continue;
            const uint32_t k = p.k, w = p.w;
#pragma unroll
            for (int b = 0; b < BPT; ++b) {
                const uint32_t* rp = s + p.res_soff + (threadIdx.x * BPT + b) * k;
                const uint32_t* mp = s + p.soff + (threadIdx.x * BPT + b) * w;
                uint32_t bl = 0, bh = 0;
                for (uint32_t j = 0; j < k + w; ++j) {
                    const uint32_t x = j < k ? rp[j] : mp[j - k];
                    bl = borrow_sub(x, P.pmx[c][j][0], bl);
                    bh = borrow_rsub(x, P.pmx[c][j][1], bh);
                }
                xm[b] &= ~(bl | bh);
            }
        }
    }
    template <int B>
    __device__ __forceinline__ uint32_t value_rt(const SelParams& P, int c, uint32_t l) const {
        const uint32_t w = P.p[c].w;
        return plane_value(stg + P.p[c].soff + (threadIdx.x * BPT + B) * w, w, l);
    }
    template <int B>
    __device__ __forceinline__ uint32_t appr(const SelParams& P, uint32_t l) const {
        uint32_t a = 0;
        for (int c = 0; c < P.npred; ++c) a |= value_rt<B>(P, c, l) << P.p[c].ashift;
        return a;
    }
    __device__ __forceinline__ static uint32_t appr_smem(const SelParams& P, const uint32_t* stg, uint32_t blk,
                                                         uint32_t l) {
        uint32_t a = 0;
        for (int c = 0; c < P.npred; ++c) a |= plane_value(stg + P.p[c].soff + blk * P.p[c].w, P.p[c].w, l) << P.p[c].ashift;
        return a;
    }
};


// ------------------------------------------------------------ pipeline

struct SmemLayout {
    uint64_t* full;
    uint64_t* empty;
    long long* slot;
    uint32_t* warp_tot;
    unsigned long long* misc;
    uint32_t* st_pos;
    uint32_t* st_aux;
    uint32_t* stages;
};

__device__ __forceinline__ SmemLayout carve(unsigned char* smem, uint32_t nstages, bool staging) {
    SmemLayout L;
    L.full = reinterpret_cast<uint64_t*>(smem);
    L.empty = L.full + nstages;
    L.slot = reinterpret_cast<long long*>(L.empty + nstages);
    L.warp_tot = reinterpret_cast<uint32_t*>(L.slot + nstages);
    L.misc = reinterpret_cast<unsigned long long*>(L.warp_tot + 32);
    unsigned char* p = reinterpret_cast<unsigned char*>(L.misc + 8);
    if (staging) {
        L.st_pos = reinterpret_cast<uint32_t*>(p);
        L.st_aux = L.st_pos + kStageEntries;
        p = reinterpret_cast<unsigned char*>(L.st_aux + kStageEntries);
    } else {
        L.st_pos = L.st_aux = nullptr;
    }
    // align by offset from the smem base (an integer round trip would lose the
    // shared address space and turn every stage access into a generic load)
    const size_t off = (size_t)(p - smem);
    L.stages = reinterpret_cast<uint32_t*>(smem + ((off + 127) & ~size_t(127)));
    return L;
}

// Producer: produce_ring (kernels.cuh) over this kernel's shared-memory carve-up.
__device__ __forceinline__ void produce(const SelParams& P, const SmemLayout& L) {
    produce_ring(P, L.full, L.empty, L.slot, L.stages);
}

template <int NW>
__device__ __forceinline__ void init_barriers(const SelParams& P, const SmemLayout& L) {
    if (threadIdx.x == 0) {
        for (uint32_t s = 0; s < P.nstages; ++s) {
            mbar_init(L.full + s, 1);
            mbar_init(L.empty + s, NW);
        }
        fence_mbar_init();
    }
    __syncthreads();
}

// ------------------------------------------------------------ ordered select

// Ordered select in three short, dependency-free kernels:
//   1. select_tile_kernel: persistent CTAs, tiles round-robin; nstages tile
//      buffers per CTA, so the TMA bulk copies of the CTA's next tiles are in
//      flight while it decides one (no CTA ever waits on another).  Per tile:
//      evaluate the planes, compact the candidates (stable: per-thread popc,
//      block scan) and write them with coalesced stores to the tile's own
//      slice of a workspace buffer, plus its count.
//   2. scan_counts_kernel: one CTA turns the per-tile counts into exclusive
//      offsets and the total.
//   3. compact_kernel: each CTA moves a chunk of tiles' slices to their final
//      offsets.
// No CTA ever waits for another: on this GPU a decoupled look-back spent most
// of the select kernel's time at its barrier (DESIGN s6.2).  The workspace
// round trip is 8 B per candidate written and read back (L2-resident at low
// selectivity).
template <class PS, int NW, int BPT, bool kCarry>
__global__ void __launch_bounds__(NW * 32) select_tile_kernel(const __grid_constant__ SelParams P) {
    constexpr int NT = NW * 32;
    constexpr uint32_t kMaxBufs = 4;
    extern __shared__ __align__(128) unsigned char smem[];
    __shared__ __align__(8) uint64_t bar[kMaxBufs];
    __shared__ uint32_t warp_tot[32];
    uint32_t* st_pos = reinterpret_cast<uint32_t*>(smem);
    uint32_t* stg0 = st_pos + kStageEntries;          // 16-B aligned (kStageEntries * 4 bytes above)
    const uint32_t nb = P.nstages;                    // tile buffers: the next tiles load while one is decided
    const long long G = gridDim.x;

    // thread 0: one TMA bulk copy per predicate brings tile t's planes into buffer b
    auto issue = [&](long long t, uint32_t b) {
        const int64_t r0 = t * (int64_t)P.tile_rows;
        const int64_t rows = min((int64_t)P.tile_rows, P.n - r0);
        const uint32_t groups = (uint32_t)((rows + 127) / 128);
        uint32_t bytes = 0;
        for (int c = 0; c < P.npred; ++c) bytes += groups * 16u * P.p[c].w;
        mbar_arrive_expect_tx(&bar[b], bytes);
        const uint64_t pol = policy_evict_first();
        uint32_t* stg = stg0 + (size_t)b * P.stage_words;
        for (int c = 0; c < P.npred; ++c) {
            const uint32_t w = P.p[c].w;
            if (w)
                bulk_g2s(stg + P.p[c].soff, P.p[c].planes + (size_t)t * (P.tile_rows / 32) * w, groups * 16u * w,
                         &bar[b], pol);
        }
    };
    if (threadIdx.x == 0) {
        for (uint32_t b = 0; b < nb; ++b) mbar_init(&bar[b], 1);
        fence_mbar_init();
        for (uint32_t b = 0; b < nb; ++b)
            if (blockIdx.x + (long long)b * G < P.num_tiles) issue(blockIdx.x + (long long)b * G, b);
    }
    __syncthreads();

    uint32_t i = 0;
    for (long long t = blockIdx.x; t < P.num_tiles; t += G, ++i) {
        // one tile per CTA (nb == 1, the default): no buffer rotation
        const uint32_t b = nb == 1 ? 0u : i % nb;
        const uint32_t* stg = stg0 + (size_t)b * P.stage_words;
        mbar_wait(&bar[b], nb == 1 ? (i & 1u) : ((i / nb) & 1u), 0);
        // compact_kernel (a programmatic dependent) may be scheduled once this CTA's last tile is loaded
        if (G == P.num_tiles || t + G >= P.num_tiles) asm volatile("griddepcontrol.launch_dependents;" ::: "memory");

        PS ps;
        ps.load(P, stg);
        uint32_t cm[BPT], dm[BPT];
        if ((t + 1) * (int64_t)P.tile_rows <= P.n) {   // a full tile: every row valid
#pragma unroll
            for (int q = 0; q < BPT; ++q) cm[q] = dm[q] = 0xffffffffu;
        } else {
            const int64_t r0 = t * (int64_t)P.tile_rows + (int64_t)threadIdx.x * (32 * BPT);
#pragma unroll
            for (int q = 0; q < BPT; ++q) cm[q] = dm[q] = valid_mask(r0 + 32 * q, P.n);
        }
        ps.eval(P, cm, dm);
        uint32_t cnt = 0;
#pragma unroll
        for (int q = 0; q < BPT; ++q) cnt += __popc(cm[q]);
        uint32_t total;
        const uint32_t excl = block_excl_scan<NT>(cnt, warp_tot, total, 1);
        if (threadIdx.x == 0) {
            P.tile_count[t] = total;
            if (total) atomicAdd(P.group_sum + (t >> kGroupShift), (unsigned long long)total);
        }

        // entries in rounds of kStageEntries: per-thread positions, lane-parallel aux, coalesced stores
        const uint32_t tile_r0 = (uint32_t)(t * (int64_t)P.tile_rows);
        uint32_t* tmp_pos = P.tmp_pos + (size_t)t * P.tile_rows;
        uint32_t* tmp_aux = P.tmp_aux + (size_t)t * P.tile_rows;
        uint32_t e = excl;
        for (uint32_t base = 0; base < total; base += kStageEntries) {
            const uint32_t lim = min(base + (uint32_t)kStageEntries, excl + cnt);
            static_for<BPT>([&](auto bc) {
                constexpr int q = decltype(bc)::value;
                const uint32_t rbase = (threadIdx.x * BPT + q) << 5;
                while (cm[q] && e < lim) {
                    const uint32_t l = __ffs(cm[q]) - 1;
                    cm[q] &= cm[q] - 1;
                    st_pos[e - base] = (rbase | l) | (((dm[q] >> l) & 1u) << 31);
                    ++e;
                }
            });
            __syncthreads();
            const uint32_t nround = min((uint32_t)kStageEntries, total - base);
            for (uint32_t j = threadIdx.x; j < nround; j += NT) {
                const uint32_t v = st_pos[j];
                const uint32_t o = v & 0x7fffffffu;
                uint32_t aux = v & 0x80000000u;
                if (kCarry) aux |= PS::appr_smem(P, stg, o >> 5, o & 31u);
                tmp_pos[base + j] = tile_r0 + o;
                tmp_aux[base + j] = aux;
            }
            __syncthreads();
        }
        __syncthreads();   // buffer b and warp_tot are free
        if (threadIdx.x == 0 && t + (long long)nb * G < P.num_tiles) issue(t + (long long)nb * G, b);
    }
}

#ifndef AR_RR_MINB
#define AR_RR_MINB 10   // CTAs per SM the register budget must allow (occupancy is what the kernel needs)
#endif
// Ordered select in ONE kernel, no workspace round trip: persistent CTAs (all
// co-resident: cooperative launch), tiles round-robin, nb TMA tile buffers per
// CTA.  Per tile the CTA evaluates the planes, publishes its candidate count
// (status[t] = kFlagAgg | count) at once and stages the tile's (position, aux)
// entries in shared memory; the entries then wait there while the CTA decides
// its next tile, and go out at their final offset, found by a decoupled
// look-back (Merrill & Garland) that normally ends at an already resolved
// neighbour (kFlagInc | inclusive prefix).  A tile with more than kRrEntries
// candidates resolves its offset at once and writes in rounds.
template <class PS, int NW, int BPT, bool kCarry>
__global__ void __launch_bounds__(NW * 32, AR_RR_MINB) select_rr_kernel(const __grid_constant__ SelParams P) {
    constexpr int NT = NW * 32;
    constexpr uint32_t kMaxBufs = 4;
    extern __shared__ __align__(128) unsigned char smem[];
    __shared__ __align__(8) uint64_t bar[kMaxBufs];
    __shared__ uint32_t warp_tot[32];
    __shared__ unsigned long long s_off;
    // staged entries: the row inside the tile (15 bits) | definite << 15, and the aux word
    uint32_t* st_aux = reinterpret_cast<uint32_t*>(smem);                 // [2][kRrEntries]
    uint16_t* st_row = reinterpret_cast<uint16_t*>(st_aux + 2 * kRrEntries);   // [2][kRrEntries]
    uint32_t* stg0 = reinterpret_cast<uint32_t*>(st_row + 2 * kRrEntries);     // nb tile buffers
    const uint32_t nb = P.nstages;
    const long long G = gridDim.x;
    const unsigned warp = threadIdx.x >> 5, lane = threadIdx.x & 31;

    auto issue = [&](long long t, uint32_t b) {
        const int64_t r0 = t * (int64_t)P.tile_rows;
        const int64_t rows = min((int64_t)P.tile_rows, P.n - r0);
        const uint32_t groups = (uint32_t)((rows + 127) / 128);
        uint32_t bytes = 0;
        for (int c = 0; c < P.npred; ++c) bytes += groups * 16u * P.p[c].w;
        mbar_arrive_expect_tx(&bar[b], bytes);
        const uint64_t pol = policy_evict_first();
        uint32_t* stg = stg0 + (size_t)b * P.stage_words;
        for (int c = 0; c < P.npred; ++c) {
            const uint32_t w = P.p[c].w;
            if (w)
                bulk_g2s(stg + P.p[c].soff, P.p[c].planes + (size_t)t * (P.tile_rows / 32) * w, groups * 16u * w,
                         &bar[b], pol);
        }
    };
    if (threadIdx.x == 0) {
        for (uint32_t b = 0; b < nb; ++b) mbar_init(&bar[b], 1);
        fence_mbar_init();
        for (uint32_t b = 0; b < nb; ++b)
            if (blockIdx.x + (long long)b * G < P.num_tiles) issue(blockIdx.x + (long long)b * G, b);
    }
    __syncthreads();

    long long pend = -1;                // tile whose entries wait in st_*[pbuf] for their offset
    uint32_t pend_total = 0, pbuf = 0;
    bool pend_dense = false;            // its entries are in its workspace slice, not in shared memory
    // Exclusive prefix of tile t by decoupled look-back (warp 0): one window of the 32 preceding
    // status words per step; a tile that is already resolved carries its inclusive prefix
    // (kFlagInc) and ends the walk, otherwise its count is added and the walk goes on.  Counts
    // are published right after each tile's evaluation, a round before its entries are
    // resolved, so the window is normally complete and ends at a resolved neighbour.
    auto lookback = [&](long long t, uint32_t total) {   // warp 0 only; every lane gets the prefix
        const unsigned long long excl = lookback_inclusive(P.status, t, total, lane);
        if (lane == 0 && t == P.num_tiles - 1) *P.out_count = (long long)(excl + total);
        return excl;
    };
    // Warp 0 writes out the pending tile while the other warps go on to the next tile (their
    // next block-scan barrier waits for it, so the buffer is free before it is restaged).
    auto resolve_w0 = [&]() {
        const unsigned long long off = lookback(pend, pend_total);
        const uint16_t* sp = st_row + pbuf * kRrEntries;
        const uint32_t* sa = st_aux + pbuf * kRrEntries;
        const uint32_t r0 = (uint32_t)(pend * (int64_t)P.tile_rows);
        for (uint32_t j = lane; j < pend_total; j += 32) {
            P.out_pos[off + j] = r0 + (sp[j] & 0x7fffu);
            P.out_aux[off + j] = sa[j];
        }
    };

    uint32_t i = 0, cb = 0;   // cb: staging buffer of the current tile
    for (long long t = blockIdx.x; t < P.num_tiles; t += G, ++i) {
        const uint32_t b = nb == 1 ? 0u : i % nb;
        const uint32_t* stg = stg0 + (size_t)b * P.stage_words;
        mbar_wait(&bar[b], nb == 1 ? (i & 1u) : ((i / nb) & 1u), 0);

        PS ps;
        ps.load(P, stg);
        uint32_t cm[BPT], dm[BPT];
        if ((t + 1) * (int64_t)P.tile_rows <= P.n) {
#pragma unroll
            for (int q = 0; q < BPT; ++q) cm[q] = dm[q] = 0xffffffffu;
        } else {
            const int64_t r0 = t * (int64_t)P.tile_rows + (int64_t)threadIdx.x * (32 * BPT);
#pragma unroll
            for (int q = 0; q < BPT; ++q) cm[q] = dm[q] = valid_mask(r0 + 32 * q, P.n);
        }
        ps.eval(P, cm, dm);
        uint32_t cnt = 0;
#pragma unroll
        for (int q = 0; q < BPT; ++q) cnt += __popc(cm[q]);
        uint32_t total;
        const uint32_t excl = block_excl_scan<NT>(cnt, warp_tot, total, 1);
        if (threadIdx.x == 0) st_relaxed(P.status + t, kFlagAgg | total);   // publish the count at once
        const uint32_t tile_r0 = (uint32_t)(t * (int64_t)P.tile_rows);

        const bool dense = total > (uint32_t)kRrEntries;
        if (total > (uint32_t)kRrSyncEntries) {
            // a very dense tile: resolve the pending one and this one's offset now, write in rounds
            // straight to the output (the writes dwarf the look-back; a workspace round trip would not)
            if (pend >= 0 && !pend_dense) {
                if (warp == 0) resolve_w0();
            } else if (pend >= 0) {
                if (warp == 0) {
                    const unsigned long long o = lookback(pend, pend_total);
                    if (lane == 0) s_off = o;
                }
                __syncthreads();
                const unsigned long long off = s_off;
                const uint32_t* tp = P.tmp_pos + (size_t)pend * P.tile_rows;
                const uint32_t* ta = P.tmp_aux + (size_t)pend * P.tile_rows;
                for (uint32_t j = threadIdx.x; j < pend_total; j += NT) {
                    P.out_pos[off + j] = __ldcs(tp + j);
                    P.out_aux[off + j] = __ldcs(ta + j);
                }
                __syncthreads();   // every thread has read s_off
            }
            if (warp == 0) {
                const unsigned long long o = lookback(t, total);
                if (lane == 0) s_off = o;
            }
            pend = -1;
            __syncthreads();
            const unsigned long long off = s_off;
            uint16_t* sp = st_row + cb * kRrEntries;
            uint32_t e = excl;
            for (uint32_t base = 0; base < total; base += kRrEntries) {
                const uint32_t lim = min(base + (uint32_t)kRrEntries, excl + cnt);
                static_for<BPT>([&](auto bc) {
                    constexpr int q = decltype(bc)::value;
                    const uint32_t rbase = (threadIdx.x * BPT + q) << 5;
                    while (cm[q] && e < lim) {
                        const uint32_t l = __ffs(cm[q]) - 1;
                        cm[q] &= cm[q] - 1;
                        sp[e - base] = (uint16_t)((rbase | l) | (((dm[q] >> l) & 1u) << 15));
                        ++e;
                    }
                });
                __syncthreads();
                const uint32_t nround = min((uint32_t)kRrEntries, total - base);
                for (uint32_t j = threadIdx.x; j < nround; j += NT) {
                    const uint32_t v = sp[j];
                    const uint32_t o = v & 0x7fffu;
                    uint32_t aux = (v >> 15) << 31;
                    if (kCarry) aux |= PS::appr_smem(P, stg, o >> 5, o & 31u);
                    P.out_pos[off + base + j] = tile_r0 + o;
                    P.out_aux[off + base + j] = aux;
                }
                __syncthreads();
            }
            if (threadIdx.x == 0 && t + (long long)nb * G < P.num_tiles) issue(t + (long long)nb * G, b);
            continue;
        }
        if (!dense) {
            // stage this tile's entries in buffer cb (the pending tile holds the other one)
            uint16_t* sp = st_row + cb * kRrEntries;
            uint32_t* sa = st_aux + cb * kRrEntries;
            uint32_t e = excl;
            static_for<BPT>([&](auto bc) {
                constexpr int q = decltype(bc)::value;
                const uint32_t rbase = (threadIdx.x * BPT + q) << 5;
                for (uint32_t m = cm[q]; m; m &= m - 1) {
                    const uint32_t l = __ffs(m) - 1;
                    sp[e++] = (uint16_t)((rbase | l) | (((dm[q] >> l) & 1u) << 15));
                }
            });
            __syncthreads();
            for (uint32_t j = threadIdx.x; j < total; j += NT) {
                const uint32_t v = sp[j];
                const uint32_t o = v & 0x7fffu;
                uint32_t aux = (v >> 15) << 31;
                if (kCarry) aux |= PS::appr_smem(P, stg, o >> 5, o & 31u);
                sa[j] = aux;
            }
        } else {
            // a dense tile: its entries go, in rounds through buffer cb, to the tile's own workspace
            // slice (tile-local order); they are copied to their final offset when resolved
            uint16_t* sp = st_row + cb * kRrEntries;
            uint32_t* tp = P.tmp_pos + (size_t)t * P.tile_rows;
            uint32_t* ta = P.tmp_aux + (size_t)t * P.tile_rows;
            uint32_t e = excl;
            for (uint32_t base = 0; base < total; base += kRrEntries) {
                const uint32_t lim = min(base + (uint32_t)kRrEntries, excl + cnt);
                static_for<BPT>([&](auto bc) {
                    constexpr int q = decltype(bc)::value;
                    const uint32_t rbase = (threadIdx.x * BPT + q) << 5;
                    while (cm[q] && e < lim) {
                        const uint32_t l = __ffs(cm[q]) - 1;
                        cm[q] &= cm[q] - 1;
                        sp[e - base] = (uint16_t)((rbase | l) | (((dm[q] >> l) & 1u) << 15));
                        ++e;
                    }
                });
                __syncthreads();
                const uint32_t nround = min((uint32_t)kRrEntries, total - base);
                for (uint32_t j = threadIdx.x; j < nround; j += NT) {
                    const uint32_t v = sp[j];
                    const uint32_t o = v & 0x7fffu;
                    uint32_t aux = (v >> 15) << 31;
                    if (kCarry) aux |= PS::appr_smem(P, stg, o >> 5, o & 31u);
                    tp[base + j] = tile_r0 + o;
                    ta[base + j] = aux;
                }
                if (base + kRrEntries < total) __syncthreads();   // sp is refilled by the next round
            }
        }
        __syncthreads();   // stage b is free; entries staged
        if (threadIdx.x == 0 && t + (long long)nb * G < P.num_tiles) issue(t + (long long)nb * G, b);
        // resolve the pending tile (a round after its count was published: the look-back is short)
        if (pend >= 0) {
            if (!pend_dense) {
                if (warp == 0) resolve_w0();
            } else {   // a dense pending tile: warp 0 finds the offset, the whole CTA copies its slice
                if (warp == 0) {
                    const unsigned long long o = lookback(pend, pend_total);
                    if (lane == 0) s_off = o;
                }
                __syncthreads();
                const unsigned long long off = s_off;
                const uint32_t* tp = P.tmp_pos + (size_t)pend * P.tile_rows;
                const uint32_t* ta = P.tmp_aux + (size_t)pend * P.tile_rows;
                for (uint32_t j = threadIdx.x; j < pend_total; j += NT) {
                    P.out_pos[off + j] = __ldcs(tp + j);
                    P.out_aux[off + j] = __ldcs(ta + j);
                }
            }
        }
        pend = t;
        pend_total = total;
        pend_dense = dense;
        if (!dense) {
            pbuf = cb;
            cb ^= 1u;
        }
    }
    if (pend >= 0) {   // the last tile
        if (!pend_dense) {
            if (warp == 0) resolve_w0();
        } else {
            if (warp == 0) {
                const unsigned long long o = lookback(pend, pend_total);
                if (lane == 0) s_off = o;
            }
            __syncthreads();
            const unsigned long long off = s_off;
            const uint32_t* tp = P.tmp_pos + (size_t)pend * P.tile_rows;
            const uint32_t* ta = P.tmp_aux + (size_t)pend * P.tile_rows;
            for (uint32_t j = threadIdx.x; j < pend_total; j += NT) {
                P.out_pos[off + j] = __ldcs(tp + j);
                P.out_aux[off + j] = __ldcs(ta + j);
            }
        }
    }
    // the refine kernel (a programmatic dependent, if launched as one) may start
    asm volatile("griddepcontrol.launch_dependents;" ::: "memory");
}

// Move the tiles' candidate slices from the workspace to their final offsets.
// One CTA per chunk of kCompactTiles consecutive tiles (a chunk never straddles
// a group of 2^kGroupShift tiles): the chunk's offset is the sum of the group
// totals before its group (accumulated with one atomic per tile by the select
// kernel) plus the counts of the earlier tiles of its group -- one block-wide
// reduction -- and the tiles' offsets inside the chunk a prefix over
// kCompactTiles counts.  Then warp w copies tile w of the chunk on its own:
// a contiguous slice to a contiguous destination, up to kDeep entries per lane
// in flight, and drops the slice's L2 lines once its lanes have loaded them.
constexpr int kCompactTiles = 8;   // = warps per CTA
__global__ void __launch_bounds__(256) compact_kernel(const __grid_constant__ SelParams P) {
    asm volatile("griddepcontrol.wait;" ::: "memory");   // no-op unless launched as a dependent
    __shared__ unsigned long long red[8];
    __shared__ uint32_t tpre[kCompactTiles + 1];
    const unsigned lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const long long nchunks = (P.num_tiles + kCompactTiles - 1) / kCompactTiles;
    for (long long ch = blockIdx.x; ch < nchunks; ch += gridDim.x) {
        const long long t0 = ch * kCompactTiles;
        const long long g = t0 >> kGroupShift, g0 = g << kGroupShift;
        unsigned long long off = 0;
        for (int i = (int)threadIdx.x; i < (int)g; i += 256) off += __ldcg(P.group_sum + i);
        for (int i = (int)threadIdx.x; i < (int)(t0 - g0); i += 256) off += __ldcg(P.tile_count + g0 + i);
#pragma unroll
        for (int o = 16; o > 0; o >>= 1) off += __shfl_xor_sync(0xffffffffu, off, o);
        if (lane == 0) red[warp] = off;
        if (warp == 0) {
            const long long t = t0 + lane;
            uint32_t c = (lane < kCompactTiles && t < P.num_tiles) ? __ldcg(P.tile_count + t) : 0u;
            uint32_t incl = c;
#pragma unroll
            for (int o = 1; o < kCompactTiles; o <<= 1) {
                const uint32_t y = __shfl_up_sync(0xffffffffu, incl, o);
                if (lane >= (unsigned)o) incl += y;
            }
            if (lane < kCompactTiles) tpre[lane + 1] = incl;
            if (lane == 0) tpre[0] = 0;
        }
        __syncthreads();
        unsigned long long base = 0;
#pragma unroll
        for (int w = 0; w < 8; ++w) base += red[w];
        if (t0 + kCompactTiles >= P.num_tiles && threadIdx.x == 0) *P.out_count = (long long)(base + tpre[kCompactTiles]);
        // warp `warp` copies tile t0 + warp
        const uint32_t c = tpre[warp + 1] - tpre[warp];
        const size_t so = (size_t)(t0 + warp) * P.tile_rows;
        const uint32_t* sp = P.tmp_pos + so;
        const uint32_t* sa = P.tmp_aux + so;
        uint32_t* dp = P.out_pos + base + tpre[warp];
        uint32_t* da = P.out_aux + base + tpre[warp];
        constexpr int kDeep = 16;   // a tile at Q6 selectivity (~330 candidates) is one round
        for (uint32_t e0 = 0; e0 < c; e0 += kDeep * 32) {
            uint32_t vp[kDeep], va[kDeep];
#pragma unroll
            for (int k = 0; k < kDeep; ++k) {
                const uint32_t e = e0 + k * 32 + lane;
                if (e < c) {
                    vp[k] = __ldcs(sp + e);   // streaming: each slice is read once
                    va[k] = __ldcs(sa + e);
                }
            }
#pragma unroll
            for (int k = 0; k < kDeep; ++k) {
                const uint32_t e = e0 + k * 32 + lane;
                if (e < c) {
                    dp[e] = vp[k];
                    da[e] = va[k];
                }
            }
        }
        __syncwarp();   // every lane has loaded its entries before the slice's lines are dropped
        // the slice is dead: drop its L2 lines without writing them back (slices are 128-B aligned,
        // 32 entries per line)
        for (uint32_t L = lane; L < (c + 31) / 32; L += 32) {
            asm volatile("discard.global.L2 [%0], 128;" ::"l"(sp + 32 * L) : "memory");
            asm volatile("discard.global.L2 [%0], 128;" ::"l"(sa + 32 * L) : "memory");
        }
        __syncthreads();   // red / tpre are reused by the next chunk
    }
}

// ----------------------------------------------------------------- fused a3+a5+a6

// Each warp owns a 1024 * BPT-row slice of the tile.  Its candidate rows are
// compacted into a per-warp list in shared memory (a 16-bit row offset with
// the definite flag in bit 15 -- the candidate relation of PAPER.md:368-374,
// kept on chip), then the lanes take kLanesPer consecutive-in-round entries
// each and refine / aggregate them in parallel, so the residual and aggregate
// gathers of a whole warp are in flight together (Alg. 2).
constexpr int kPer = 2;               // list entries per lane per pass
constexpr int kGSlot = 32 * kPer;     // async-gather entries per warp per tile (first pass)
constexpr int kGDepth = 4;            // tiles of gathers in flight per warp

__device__ __forceinline__ void cp_async4(uint32_t* dst, const uint32_t* src) {
    asm volatile("cp.async.ca.shared.global" AR_GHINT " [%0], [%1], 4;" ::"r"(smem_u32(dst)), "l"(src) : "memory");
}
__device__ __forceinline__ void cp_async_commit() { asm volatile("cp.async.commit_group;" ::: "memory"); }
template <int N>
__device__ __forceinline__ void cp_async_wait() { asm volatile("cp.async.wait_group %0;" ::"n"(N) : "memory"); }

// Sum this lane's landed entries of one async-gather slot: value of the gathered
// packed column (1-2 words, shift) times the pre-computed other factor.
__device__ __forceinline__ unsigned long long gather_drain(const uint32_t* slot, uint32_t lane, const AggCol& G) {
    unsigned long long acc = 0;
#pragma unroll
    for (int q = 0; q < kPer; ++q) {
        const uint32_t ei = q * 32 + lane;
        const uint32_t info = slot[2 * kGSlot + ei];
        if (!(info >> 31)) continue;
        const uint32_t sh = (info >> 26) & 31u, mult = info & ((1u << 26) - 1u);
        const uint32_t lo = slot[ei];
        uint32_t v = lo >> sh;
        if (sh + G.w > 32u) v = __funnelshift_r(lo, slot[kGSlot + ei], sh);
        if (G.w < 32) v &= (1u << G.w) - 1u;
        acc += (unsigned long long)(v + G.base) * mult;
    }
    return acc;
}
constexpr uint32_t kDefFlag = 0x8000u;

// Major of predicate c at block-local row l of global block `blk` of the tile.
__device__ __forceinline__ uint32_t stage_value(const SelParams& P, const uint32_t* stg, int c, uint32_t blk,
                                                uint32_t l) {
    const uint32_t w = P.p[c].w;
    return plane_value(stg + P.p[c].soff + blk * w, w, l);
}

template <class PS, int NW, int BPT>
__global__ void __launch_bounds__((NW + 1) * 32, 2) fused_kernel(const __grid_constant__ SelParams P) {
    constexpr int kWarpRows = 32 * 32 * BPT;
    extern __shared__ __align__(128) unsigned char smem[];
    const SmemLayout L = carve(smem, P.nstages, false);
    const unsigned warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    init_barriers<NW>(P, L);
    // per-warp candidate lists live after the stage ring, then the async-gather slots
    uint16_t* list = reinterpret_cast<uint16_t*>(L.stages + (size_t)P.nstages * P.stage_words) + warp * kWarpRows;
    uint32_t* gslot = reinterpret_cast<uint32_t*>(reinterpret_cast<uint16_t*>(L.stages +
                                                  (size_t)P.nstages * P.stage_words) + NW * kWarpRows) +
                      warp * (kGDepth * kGSlot * 3);

    if (warp == NW) {
        if (lane == 0) produce(P, L);
        return;
    }

    unsigned long long sum = 0, nres = 0, ncand = 0, ndef = 0;
    uint32_t gseq = 0;   // async-gather tiles issued by this warp
    uint32_t s = 0, ph = 0;
    for (;; s = (s + 1 == P.nstages) ? (ph ^= 1u, 0u) : s + 1) {
        mbar_wait(L.full + s, ph, P.suspend_ns);
        const long long t = L.slot[s];
        if (t < 0) break;
        const uint32_t* stg = L.stages + (size_t)s * P.stage_words;
        const int64_t tile_r0 = t * (int64_t)P.tile_rows;
        const int64_t r0 = tile_r0 + (int64_t)threadIdx.x * (32 * BPT);

        // a3: candidate / definite masks of this thread's blocks
        PS ps;
        ps.load(P, stg);
        uint32_t cm[BPT], dm[BPT];
#pragma unroll
        for (int b = 0; b < BPT; ++b) cm[b] = dm[b] = valid_mask(r0 + 32 * b, P.n);
        ps.eval(P, cm, dm);
        uint32_t cnt = 0;
#pragma unroll
        for (int b = 0; b < BPT; ++b) {
            cnt += __popc(cm[b]);
            ndef += __popc(dm[b]);
        }
        ncand += cnt;
        const bool exact_mode = P.exact_mode != 0;
        if (P.nagg == 0 && !exact_mode) {
            // COUNT: a definite candidate is a result (Alg. 2 never touches it) -- counted here,
            // only the non-definite ones go through the list and the residual gathers
            cnt = 0;
#pragma unroll
            for (int b = 0; b < BPT; ++b) {
                nres += __popc(dm[b]);
                cm[b] &= ~dm[b];
                dm[b] = 0u;
                cnt += __popc(cm[b]);
            }
        }
        if (exact_mode) {
            // a5 in place: exact predicate on major + residual planes of the candidate rows;
            // the list below then holds result rows only (no per-candidate refine pass)
            uint32_t xm[BPT];
#pragma unroll
            for (int b = 0; b < BPT; ++b) xm[b] = cm[b];
            ps.exact(P, stg, xm);
            cnt = 0;
#pragma unroll
            for (int b = 0; b < BPT; ++b) {
                cm[b] = xm[b];
                dm[b] = xm[b];        // every listed row is a result: marked definite, skips the refine pass
                cnt += __popc(xm[b]);
            }
        }

        // compact the warp's candidates into its list (ascending row order)
        uint32_t incl = cnt;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            const uint32_t y = __shfl_up_sync(0xffffffffu, incl, o);
            if (lane >= (unsigned)o) incl += y;
        }
        const uint32_t total = __shfl_sync(0xffffffffu, incl, 31);
        uint32_t e = incl - cnt;   // this thread's first slot in the warp list
#pragma unroll
        for (int b = 0; b < BPT; ++b) {
            uint32_t m = cm[b];
            while (m) {
                const uint32_t l = __ffs(m) - 1;
                m &= m - 1;
                list[e++] = (uint16_t)((((lane * BPT + b) << 5) | l) | (((dm[b] >> l) & 1u) ? kDefFlag : 0u));
            }
        }
        __syncwarp();

        // a5 + a6 over the list: each lane takes kPer entries per pass
        const uint32_t row_in_tile0 = warp * kWarpRows;
        const uint64_t row_base = (uint64_t)tile_r0 + row_in_tile0;
        for (uint32_t base = 0; base < total; base += 32 * kPer) {
            uint32_t off[kPer];
            bool ok[kPer], dfn[kPer];
#pragma unroll
            for (int q = 0; q < kPer; ++q) {
                const uint32_t k = base + q * 32 + lane;
                const uint32_t e = k < total ? list[k] : 0u;
                ok[q] = k < total;
                dfn[q] = (e & kDefFlag) != 0;
                off[q] = e & 0x7fffu;   // row offset inside the warp slice
            }
            // refine non-definite entries (Alg. 2): residual + major -> exact value -> predicate
            PS::for_pred(P, [&](auto cc) {
                const SelPred& p = P.p[int(cc)];
                if (p.k == 0) return;   // exact already at the approximation
                const uint32_t w = PS::pw(P, cc);
                uint32_t r[kPer];
#pragma unroll
                for (int q = 0; q < kPer; ++q) {
                    const bool need = ok[q] && !dfn[q];
                    if (p.res_stream)
                        r[q] = need ? plane_value(stg + p.res_soff + ((row_in_tile0 + off[q]) >> 5) * p.k, p.k,
                                                  off[q] & 31u)
                                    : 0u;
                    else
                        r[q] = need ? residual_get(p.residual, row_base + off[q], p.k, p.rlayout) : 0u;
                }
#pragma unroll
                for (int q = 0; q < kPer; ++q) {
                    if (!ok[q] || dfn[q]) continue;
                    const uint32_t* pl = stg + p.soff + ((row_in_tile0 + off[q]) >> 5) * w;
                    const uint32_t l = off[q] & 31u;
                    uint32_t m = 0;
#pragma unroll
                    for (uint32_t j = 0; j < w; ++j) m |= ((pl[j] >> l) & 1u) << j;
                    const uint32_t v = ((m << p.k) | r[q]) + p.base;
                    ok[q] = (v >= p.lo) && (v <= p.hi);
                }
            });
#pragma unroll
            for (int q = 0; q < kPer; ++q) nres += ok[q];
            if (P.async_agg && base == 0) {
                // a6, asynchronous: the other factor (a predicate column's value) now, the gathered
                // column's 1-2 words by cp.async into this tile's slot; summed kGDepth-1 tiles later
                uint32_t* slot = gslot + (gseq % kGDepth) * (kGSlot * 3);
                const AggCol& G = P.a[P.gidx];
#pragma unroll
                for (int q = 0; q < kPer; ++q) {
                    const uint32_t ei = q * 32 + lane;
                    uint32_t mult = 1u;
                    if (ok[q] && P.nagg > 1) {
                        const AggCol& A = P.a[1 - P.gidx];
                        PS::for_pred(P, [&](auto cc) {
                            if (int(cc) != A.pred) return;
                            const SelPred& p = P.p[int(cc)];
                            const uint32_t w = PS::pw(P, cc);
                            const uint32_t* pl = stg + p.soff + ((row_in_tile0 + off[q]) >> 5) * w;
                            const uint32_t l = off[q] & 31u;
                            uint32_t m = 0;
#pragma unroll
                            for (uint32_t j = 0; j < w; ++j) m |= ((pl[j] >> l) & 1u) << j;
                            uint32_t r = 0u;
                            if (p.k)
                                r = p.res_stream ? plane_value(stg + p.res_soff + ((row_in_tile0 + off[q]) >> 5) * p.k,
                                                               p.k, off[q] & 31u)
                                                 : residual_get(p.residual, row_base + off[q], p.k, p.rlayout);
                            mult = ((m << p.k) | r) + p.base;
                        });
                    }
                    uint32_t info = 0u;
                    if (ok[q]) {
                        const uint64_t bit = (row_base + off[q]) * (uint64_t)G.w;
                        const uint32_t* src = G.major + (bit >> 5);
                        const uint32_t sh = (uint32_t)(bit & 31);
                        cp_async4(slot + ei, src);
                        if (sh + G.w > 32u) cp_async4(slot + kGSlot + ei, src + 1);
                        info = (1u << 31) | (sh << 26) | mult;   // mult < 2^26 (checked on the host)
                    }
                    slot[2 * kGSlot + ei] = info;
                }
                cp_async_commit();
                ++gseq;
                if (gseq >= (uint32_t)kGDepth) {       // consume the tile issued kGDepth-1 tiles ago
                    cp_async_wait<kGDepth - 1>();
                    sum += gather_drain(gslot + (gseq % kGDepth) * (kGSlot * 3), lane, G);
                }
            } else if (P.nagg > 0) {
                unsigned long long prod[kPer];
#pragma unroll
                for (int q = 0; q < kPer; ++q) prod[q] = ok[q] ? 1ull : 0ull;
                for (int a = 0; a < P.nagg; ++a) {
                    const AggCol& A = P.a[a];
                    uint32_t v[kPer];
#pragma unroll
                    for (int q = 0; q < kPer; ++q) v[q] = 0u;
                    if (A.pred >= 0) {
                        // an aggregate that is also a predicate column: its major is in the stage
                        PS::for_pred(P, [&](auto cc) {
                            if (int(cc) != A.pred) return;
                            const SelPred& p = P.p[int(cc)];
                            const uint32_t w = PS::pw(P, cc);
#pragma unroll
                            for (int q = 0; q < kPer; ++q) {
                                if (!ok[q]) continue;
                                const uint32_t* pl = stg + p.soff + ((row_in_tile0 + off[q]) >> 5) * w;
                                const uint32_t l = off[q] & 31u;
                                uint32_t m = 0;
#pragma unroll
                                for (uint32_t j = 0; j < w; ++j) m |= ((pl[j] >> l) & 1u) << j;
                                uint32_t r = 0u;
                                if (p.k)
                                    r = p.res_stream
                                            ? plane_value(stg + p.res_soff + ((row_in_tile0 + off[q]) >> 5) * p.k, p.k,
                                                          off[q] & 31u)
                                            : residual_get(p.residual, row_base + off[q], p.k, p.rlayout);
                                v[q] = ((m << p.k) | r) + p.base;
                            }
                        });
                    } else {
#pragma unroll
                        for (int q = 0; q < kPer; ++q) v[q] = ok[q] ? agg_gather(A, row_base + off[q]) : 0u;
                    }
#pragma unroll
                    for (int q = 0; q < kPer; ++q) prod[q] *= v[q];
                }
#pragma unroll
                for (int q = 0; q < kPer; ++q) sum += prod[q];
            }
        }
        __syncwarp();
        if (lane == 0) mbar_arrive(L.empty + s);
    }
    if (P.async_agg) {   // drain the gathers still in flight
        cp_async_wait<0>();
        const AggCol& G = P.a[P.gidx];
        for (uint32_t k = (gseq >= (uint32_t)kGDepth ? gseq - kGDepth + 1 : 0); k < gseq; ++k)
            sum += gather_drain(gslot + (k % kGDepth) * (kGSlot * 3), lane, G);
    }

    // CTA reduction, then one atomic per counter
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) {
        sum += __shfl_xor_sync(0xffffffffu, sum, o);
        nres += __shfl_xor_sync(0xffffffffu, nres, o);
        ncand += __shfl_xor_sync(0xffffffffu, ncand, o);
        ndef += __shfl_xor_sync(0xffffffffu, ndef, o);
    }
    if (lane == 0) {
        atomicAdd(P.out4 + 0, sum);
        atomicAdd(P.out4 + 1, nres);
        atomicAdd(P.out4 + 2, ncand);
        atomicAdd(P.out4 + 3, ndef);
    }
}

}  // namespace ard

// ------------------------------------------------------------------------ host

namespace ar {

// Kernel configurations: (consumer warps, blocks per thread) of the ordered
// select and of the fused kernel, and the decomposition shapes with
// specialised kernels.  Any other shape takes the DynPlanes path.
constexpr int kSelNW = 4, kSelBPT = 2;
constexpr int kFusNW = 8, kFusBPT = 1;

template <int... Ws>
struct ShapeEntry {
    static bool match(const ard::SelParams& P) {
        constexpr int n = sizeof...(Ws);
        constexpr int w[] = {Ws..., 0};
        if (P.npred != n) return false;
        for (int c = 0; c < n; ++c)
            if ((int)P.p[c].w != w[c]) return false;
        return true;
    }
    template <int BPT>
    static const void* select_fn_b(bool carry) {
        using PS = ard::FixedPlanes<BPT, Ws...>;
        return carry ? (const void*)ard::select_tile_kernel<PS, kSelNW, BPT, true>
                     : (const void*)ard::select_tile_kernel<PS, kSelNW, BPT, false>;
    }
    static const void* select_fn(bool carry, int bpt) {
        return bpt == 4 ? select_fn_b<4>(carry) : select_fn_b<kSelBPT>(carry);
    }
    static const void* select_rr_fn(bool carry) {
        using PS = ard::FixedPlanes<kSelBPT, Ws...>;
        return carry ? (const void*)ard::select_rr_kernel<PS, kSelNW, kSelBPT, true>
                     : (const void*)ard::select_rr_kernel<PS, kSelNW, kSelBPT, false>;
    }
    static const void* fused_fn() {
        using PS = ard::FixedPlanes<kFusBPT, Ws...>;
        return (const void*)ard::fused_kernel<PS, kFusNW, kFusBPT>;
    }
};

// Q6 (l_shipdate 24/8 -> 4 major bits, l_discount 4, l_quantity 6); single
// columns at 8 / 16 / 24 / 32 major bits (configs C1, C3); two 24-bit columns
// (spatial range query).
template <class... Es>
struct ShapeList {
    static bool find(const ard::SelParams& P, bool fused, bool carry, const void** fn) {
        return (try_one<Es>(P, fused, carry, fn) || ...);
    }
    static bool find_rr(const ard::SelParams& P, bool carry, const void** fn) {
        return ((Es::match(P) ? (*fn = Es::select_rr_fn(carry), true) : false) || ...);
    }
    template <class E>
    static bool try_one(const ard::SelParams& P, bool fused, bool carry, const void** fn) {
        if (!E::match(P)) return false;
        *fn = fused ? E::fused_fn() : E::select_fn(carry, (int)P.bpt);
        return true;
    }

};
using Shapes = ShapeList<ShapeEntry<4, 4, 6>, ShapeEntry<8>, ShapeEntry<16>, ShapeEntry<24>, ShapeEntry<32>,
                         ShapeEntry<24, 24>>;

int kernel_warps(bool fused) { return fused ? kFusNW : kSelNW; }               // compute warps
static int kernel_threads(bool fused) { return 32 * (kernel_warps(fused) + (fused ? 1 : 0)); }  // + producer (fused)
// blocks of 32 rows per select thread: AR_SEL_BPT = 4 gives 16384-row tiles (compiled shapes only)
int kernel_bpt(bool fused) {
    static const int sel_bpt = getenv("AR_SEL_BPT") && atoi(getenv("AR_SEL_BPT")) == 4 ? 4 : kSelBPT;
    return fused ? kFusBPT : sel_bpt;
}

const void* select_kernel_fn(const ard::SelParams& P, bool fused) {
    const void* fn = nullptr;
    if (!getenv("AR_FORCE_GENERIC") && Shapes::find(P, fused, P.carry != 0, &fn)) return fn;
    if (fused) return (const void*)ard::fused_kernel<ard::DynPlanes<kFusBPT>, kFusNW, kFusBPT>;
    if (P.bpt != kSelBPT) return nullptr;   // runtime widths: 2 blocks per thread only
    return P.carry ? (const void*)ard::select_tile_kernel<ard::DynPlanes<kSelBPT>, kSelNW, kSelBPT, true>
                   : (const void*)ard::select_tile_kernel<ard::DynPlanes<kSelBPT>, kSelNW, kSelBPT, false>;
}

// The one-kernel ordered select (select_rr_kernel) for this shape: compiled shapes, else runtime widths.
const void* select_rr_kernel_fn(const ard::SelParams& P) {
    const void* fn = nullptr;
    if (P.bpt != kSelBPT) return nullptr;
    if (!getenv("AR_FORCE_GENERIC") && Shapes::find_rr(P, P.carry != 0, &fn)) return fn;
    return P.carry ? (const void*)ard::select_rr_kernel<ard::DynPlanes<kSelBPT>, kSelNW, kSelBPT, true>
                   : (const void*)ard::select_rr_kernel<ard::DynPlanes<kSelBPT>, kSelNW, kSelBPT, false>;
}
size_t select_rr_smem_bytes(uint32_t stage_words, uint32_t nstages) {
    return 2ull * ard::kRrEntries * (4 + 2) + (size_t)nstages * stage_words * 4;
}
// Cooperative launch: the look-back waits on other CTAs' tiles, so every CTA must be
// resident; a grid that cannot be fails with an error instead of hanging.
ar_status launch_select_rr(const void* fn, const ard::SelParams& P, int grid, size_t smem, cudaStream_t s) {
    opt_in_max_smem(fn);
    void* args[] = {const_cast<ard::SelParams*>(&P)};
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = dim3(grid);
    cfg.blockDim = dim3(kernel_threads(false));
    cfg.dynamicSmemBytes = smem;
    cfg.stream = s;
    cudaLaunchAttribute attr[1];
    attr[0].id = cudaLaunchAttributeCooperative;
    attr[0].val.cooperative = 1;
    cfg.attrs = attr;
    cfg.numAttrs = 1;
    AR_TRY_CUDA(cudaLaunchKernelExC(&cfg, fn, args));
    return AR_OK;
}

size_t select_smem_bytes(uint32_t stage_words, uint32_t nstages, bool staging) {
    size_t head = nstages * (8 + 8 + 8) + 32 * 4 + 8 * 8;
    if (staging) return 1ull * ard::kStageEntries * 4 + (size_t)nstages * stage_words * 4;   // select: tile buffers
    head = (head + 127) & ~size_t(127);
    size_t bytes = head + 128 + (size_t)nstages * stage_words * 4;
    if (!staging) bytes += (size_t)kFusNW * 32 * 32 * kFusBPT * 2   // per-warp candidate lists (u16)
                         + (size_t)kFusNW * ard::kGDepth * ard::kGSlot * 3 * 4;   // async-gather slots
    return bytes;
}

static void set_max_smem(const void* fn) { opt_in_max_smem(fn); }

int select_occupancy(const void* fn, size_t smem, bool fused) {
    int blocks = 0;
    set_max_smem(fn);
    cudaOccupancyMaxActiveBlocksPerMultiprocessor(&blocks, fn, kernel_threads(fused), smem);
    return blocks;
}

// Plain launch of a scan kernel (select_tile_kernel: one tile per CTA, no CTA
// waits on another; fused_kernel: persistent, tiles handed out round-robin and
// each CTA's partial SUM / counts added atomically, so neither needs its CTAs
// co-resident).
ar_status launch_scan(const void* fn, const ard::SelParams& P, int grid, size_t smem, bool fused, cudaStream_t s) {
    set_max_smem(fn);
    void* args[] = {const_cast<ard::SelParams*>(&P)};
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = dim3(grid);
    cfg.blockDim = dim3(kernel_threads(fused));
    cfg.dynamicSmemBytes = smem;
    cfg.stream = s;
    AR_TRY_CUDA(cudaLaunchKernelExC(&cfg, fn, args));
    return AR_OK;
}

// compact_kernel; after the persistent select it is a programmatic dependent
// launch (the select's producer triggers it once its last tile is loading).
ar_status launch_select_rest(const ard::SelParams& P, bool pdl, cudaStream_t s) {
    // one CTA per chunk: the block scheduler refills an SM as soon as a chunk is done
    const long long chunks = (P.num_tiles + ard::kCompactTiles - 1) / ard::kCompactTiles;
    const int grid = (int)std::min<long long>(chunks, 1ll << 30);
    ard::SelParams Q = P;
    void* args[] = {&Q};
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = dim3(grid);
    cfg.blockDim = dim3(256);
    cfg.stream = s;
    cudaLaunchAttribute attr[1];
    attr[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
    attr[0].val.programmaticStreamSerializationAllowed = pdl ? 1 : 0;
    cfg.attrs = attr;
    cfg.numAttrs = 1;
    AR_TRY_CUDA(cudaLaunchKernelExC(&cfg, (const void*)ard::compact_kernel, args));
    return AR_OK;
}

}  // namespace ar

// select.cu -- step a3: approximate selection + stable compaction over SLICED
// majors (s IV-B), and the one-pass fused A&R kernel
// (a3 + a5 + a6).
//
// Structure (both kernels): persistent CTAs, one producer warp + kSelWarps
// consumer warps.  The producer streams 4096-row tiles of every predicate's
// bit planes into a ring of shared-memory stages with 1-D TMA bulk copies
// (cp.async.bulk, completion on an mbarrier), so several tiles of HBM traffic
// are always in flight per SM.  Each consumer thread owns one 32-row block of
// the tile and evaluates every range predicate on the bit planes with borrow
// chains: per plane and per bound one 3-input logic op decides 32 rows at once
// (DESIGN "Kernel a3").  The select kernel then compacts candidate rows in
// ascending order: per-thread popc, block scan, decoupled look-back across
// tiles (dynamic tile tickets), shared-memory staging and coalesced stores.
#include "kernels.cuh"

namespace ard {

// Range test lo <= v <= hi of the 32 rows of one block whose W bit planes are
// x[0..W) (x[j] = bit j of the 32 values).  v < lo iff subtracting lo borrows
// out of the top bit; v > hi iff hi - v borrows.  One LOP3 per plane and bound.
template <int W>
__device__ __forceinline__ uint32_t range_mask(const uint32_t* x, uint32_t lo, uint32_t hi) {
    uint32_t bl = 0, bh = 0;
#pragma unroll
    for (int j = 0; j < W; ++j) {
        const uint32_t L = 0u - ((lo >> j) & 1u);
        const uint32_t H = 0u - ((hi >> j) & 1u);
        bl = (~x[j] & (L | bl)) | (x[j] & L & bl);   // borrow of v - lo
        bh = (~H & (x[j] | bh)) | (H & x[j] & bh);   // borrow of hi - v
    }
    return ~(bl | bh);
}

template <int W>
__device__ __forceinline__ void eval_pred_w(const uint32_t* __restrict__ pl, const SelPred& p, uint32_t& cm,
                                            uint32_t& dm) {
    uint32_t x[W > 0 ? W : 1];
#pragma unroll
    for (int j = 0; j < W; ++j) x[j] = pl[j];
    const uint32_t c = range_mask<W>(x, p.clo, p.chi);
    cm &= c;
    if (p.mode == 0) {
        dm &= c;
    } else if (p.mode == 1) {
        dm &= range_mask<W>(x, p.dlo, p.dhi);
    } else {
        dm = 0;
    }
}

__device__ __forceinline__ void eval_pred(const uint32_t* __restrict__ pl, const SelPred& p, uint32_t& cm,
                                          uint32_t& dm) {
    switch (p.w) {
#define AR_W(W) \
    case W: eval_pred_w<W>(pl, p, cm, dm); break;
        AR_W(0) AR_W(1) AR_W(2) AR_W(3) AR_W(4) AR_W(5) AR_W(6) AR_W(7) AR_W(8)
        AR_W(9) AR_W(10) AR_W(11) AR_W(12) AR_W(13) AR_W(14) AR_W(15) AR_W(16)
        AR_W(17) AR_W(18) AR_W(19) AR_W(20) AR_W(21) AR_W(22) AR_W(23) AR_W(24)
        AR_W(25) AR_W(26) AR_W(27) AR_W(28) AR_W(29) AR_W(30) AR_W(31) AR_W(32)
#undef AR_W
        default: break;
    }
}

// Major of row l (0..31) of a block from its bit planes in shared memory.
__device__ __forceinline__ uint32_t plane_value(const uint32_t* pl, uint32_t w, uint32_t l) {
    uint32_t m = 0;
    for (uint32_t j = 0; j < w; ++j) m |= ((pl[j] >> l) & 1u) << j;
    return m;
}

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
        L.st_aux = L.st_pos + kSelTileRows;
        p = reinterpret_cast<unsigned char*>(L.st_aux + kSelTileRows);
    } else {
        L.st_pos = L.st_aux = nullptr;
    }
    uintptr_t a = (reinterpret_cast<uintptr_t>(p) + 127) & ~uintptr_t(127);
    L.stages = reinterpret_cast<uint32_t*>(a);
    return L;
}

// Producer: one elected lane streams tiles into the stage ring.  Tile order
// comes from `next_tile` (a ticket for the ordered select, a static stride for
// the fused kernel); a negative tile index ends the stream.
template <typename NextTile>
__device__ __forceinline__ void produce(const SelParams& P, const SmemLayout& L, NextTile next_tile) {
    const uint64_t pol = policy_evict_first();
    for (uint32_t i = 0;; ++i) {
        const uint32_t s = i % P.nstages;
        if (i >= P.nstages) mbar_wait(L.empty + s, ((i / P.nstages) - 1) & 1);
        const long long t = next_tile(i);
        if (t < 0) {
            L.slot[s] = -1;
            mbar_arrive(L.full + s);
            return;
        }
        L.slot[s] = t;
        const int64_t r0 = t * (int64_t)kSelTileRows;
        const int64_t rows = min((int64_t)kSelTileRows, P.n - r0);
        const uint32_t groups = (uint32_t)((rows + 127) / 128);   // 128-row groups, 16 B per plane
        uint32_t bytes = 0;
        for (int c = 0; c < P.npred; ++c) bytes += groups * 16u * P.p[c].w;
        mbar_arrive_expect_tx(L.full + s, bytes);
        uint32_t* stg = L.stages + (size_t)s * P.stage_words;
        for (int c = 0; c < P.npred; ++c) {
            const uint32_t w = P.p[c].w;
            if (w == 0) continue;
            const uint32_t* src = P.p[c].planes + (size_t)t * (kSelTileRows / 32) * w;
            bulk_g2s(stg + P.p[c].soff, src, groups * 16u * w, L.full + s, pol);
        }
    }
}

template <bool kCarry>
__global__ void __launch_bounds__((kSelWarps + 1) * 32) select_kernel(const __grid_constant__ SelParams P) {
    extern __shared__ __align__(128) unsigned char smem[];
    const SmemLayout L = carve(smem, P.nstages, true);
    const unsigned warp = threadIdx.x >> 5, lane = threadIdx.x & 31;

    if (threadIdx.x == 0) {
        for (uint32_t s = 0; s < P.nstages; ++s) {
            mbar_init(L.full + s, 1);
            mbar_init(L.empty + s, kSelWarps);
        }
        fence_mbar_init();
    }
    __syncthreads();

    if (warp == kSelWarps) {
        if (lane == 0)
            produce(P, L, [&](uint32_t) -> long long {
                const long long t = (long long)atomicAdd(P.ticket, 1u);
                return t < P.num_tiles ? t : -1;
            });
        return;
    }

    for (uint32_t i = 0;; ++i) {
        const uint32_t s = i % P.nstages;
        mbar_wait(L.full + s, (i / P.nstages) & 1);
        const long long t = L.slot[s];
        if (t < 0) break;
        const uint32_t* stg = L.stages + (size_t)s * P.stage_words;
        const int64_t r0 = t * (int64_t)kSelTileRows + (int64_t)threadIdx.x * 32;

        uint32_t cm = valid_mask(r0, P.n), dm = cm;
        for (int c = 0; c < P.npred; ++c) eval_pred(stg + P.p[c].soff + threadIdx.x * P.p[c].w, P.p[c], cm, dm);

        const uint32_t cnt = __popc(cm);
        uint32_t total;
        const uint32_t excl = block_excl_scan<kSelThreads>(cnt, L.warp_tot, total, 1);

        if (warp == 0) {
            unsigned long long prefix = 0;
            if (t == 0) {
                if (lane == 0) st_release(P.status, kFlagPrefix | total);
            } else {
                if (lane == 0) st_release(P.status + t, kFlagAgg | total);
                prefix = lookback(P.status, t, lane);
                if (lane == 0) st_release(P.status + t, kFlagPrefix | (prefix + total));
            }
            if (lane == 0) {
                L.misc[0] = prefix;
                if (t == P.num_tiles - 1) *P.out_count = (long long)(prefix + total);
            }
        }

        // stage this thread's candidates (ascending) at their tile-local offsets
        uint32_t m = cm, o = excl;
        while (m) {
            const uint32_t l = __ffs(m) - 1;
            m &= m - 1;
            uint32_t aux = ((dm >> l) & 1u) << 31;
            if (kCarry) {
                for (int c = 0; c < P.npred; ++c)
                    aux |= plane_value(stg + P.p[c].soff + threadIdx.x * P.p[c].w, P.p[c].w, l) << P.p[c].ashift;
            }
            L.st_pos[o] = (uint32_t)(r0 + l);
            L.st_aux[o] = aux;
            ++o;
        }
        bar_sync(1, kSelThreads);
        if (lane == 0) mbar_arrive(L.empty + s);   // planes of stage s no longer needed

        const unsigned long long off = L.misc[0];
        for (uint32_t j = threadIdx.x; j < total; j += kSelThreads) {
            P.out_pos[off + j] = L.st_pos[j];
            P.out_aux[off + j] = L.st_aux[j];
        }
    }
}

// ----------------------------------------------------------------- fused a3+a5+a6

__device__ __forceinline__ uint32_t agg_value(const AggCol& a, const SelParams& P, const uint32_t* stg,
                                              uint32_t bt, uint32_t l, uint64_t row) {
    if (a.pred >= 0) {
        const SelPred& p = P.p[a.pred];
        const uint32_t m = plane_value(stg + p.soff + bt * p.w, p.w, l);
        const uint32_t r = a.k ? packed_get_any(a.residual, row, a.k) : 0u;
        return ((m << a.k) | r) + a.base;
    }
    return value_get(a.major, a.residual, row, a.w, a.k, a.layout, a.base);
}

__global__ void __launch_bounds__((kSelWarps + 1) * 32) fused_kernel(const __grid_constant__ SelParams P) {
    extern __shared__ __align__(128) unsigned char smem[];
    const SmemLayout L = carve(smem, P.nstages, false);
    const unsigned warp = threadIdx.x >> 5, lane = threadIdx.x & 31;

    if (threadIdx.x == 0) {
        for (uint32_t s = 0; s < P.nstages; ++s) {
            mbar_init(L.full + s, 1);
            mbar_init(L.empty + s, kSelWarps);
        }
        fence_mbar_init();
    }
    __syncthreads();

    if (warp == kSelWarps) {
        if (lane == 0)
            produce(P, L, [&](uint32_t i) -> long long {
                const long long t = (long long)blockIdx.x + (long long)i * gridDim.x;
                return t < P.num_tiles ? t : -1;
            });
        return;
    }

    unsigned long long sum = 0, nres = 0, ncand = 0, ndef = 0;
    for (uint32_t i = 0;; ++i) {
        const uint32_t s = i % P.nstages;
        mbar_wait(L.full + s, (i / P.nstages) & 1);
        const long long t = L.slot[s];
        if (t < 0) break;
        const uint32_t* stg = L.stages + (size_t)s * P.stage_words;
        const int64_t r0 = t * (int64_t)kSelTileRows + (int64_t)threadIdx.x * 32;

        uint32_t cm = valid_mask(r0, P.n), dm = cm;
        for (int c = 0; c < P.npred; ++c) eval_pred(stg + P.p[c].soff + threadIdx.x * P.p[c].w, P.p[c], cm, dm);
        ncand += __popc(cm);
        ndef += __popc(dm);

        // refine the non-definite candidates inline (Alg. 2 on the fly)
        uint32_t res = dm, nd = cm & ~dm;
        while (nd) {
            const uint32_t l = __ffs(nd) - 1;
            nd &= nd - 1;
            bool ok = true;
            for (int c = 0; c < P.npred && ok; ++c) {
                const SelPred& p = P.p[c];
                if (p.k == 0) continue;   // exact already at the approximation
                const uint32_t m = plane_value(stg + p.soff + threadIdx.x * p.w, p.w, l);
                const uint32_t r = packed_get_any(p.residual, (uint64_t)(r0 + l), p.k);
                const uint32_t v = ((m << p.k) | r) + p.base;
                ok = (v >= p.lo) && (v <= p.hi);
            }
            if (ok) res |= 1u << l;
        }
        nres += __popc(res);
        if (P.nagg > 0) {
            uint32_t m = res;
            while (m) {
                const uint32_t l = __ffs(m) - 1;
                m &= m - 1;
                const uint64_t row = (uint64_t)(r0 + l);
                unsigned long long prod = agg_value(P.a[0], P, stg, threadIdx.x, l, row);
                if (P.nagg > 1) prod *= agg_value(P.a[1], P, stg, threadIdx.x, l, row);
                sum += prod;
            }
        }
        __syncwarp();
        if (lane == 0) mbar_arrive(L.empty + s);
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

namespace ar {

size_t select_smem_bytes(uint32_t stage_words, uint32_t nstages, bool staging) {
    size_t head = nstages * (8 + 8 + 8) + 32 * 4 + 8 * 8;
    if (staging) head += 2ull * ard::kSelTileRows * 4;
    head = (head + 127) & ~size_t(127);
    return head + 128 + (size_t)nstages * stage_words * 4;
}

static bool g_attr_done[3] = {false, false, false};

static void set_max_smem(const void* fn, int idx) {
    if (!g_attr_done[idx]) {
        cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, 227 * 1024);
        g_attr_done[idx] = true;
    }
}

int select_occupancy(size_t smem, bool fused) {
    int blocks = 0;
    const void* fn = fused ? (const void*)ard::fused_kernel : (const void*)ard::select_kernel<true>;
    set_max_smem(fn, fused ? 2 : 0);
    if (!fused) set_max_smem((const void*)ard::select_kernel<false>, 1);
    cudaOccupancyMaxActiveBlocksPerMultiprocessor(&blocks, fn, (ard::kSelWarps + 1) * 32, smem);
    return blocks;
}

ar_status launch_select(const ard::SelParams& P, int grid, size_t smem, cudaStream_t s) {
    const dim3 block((ard::kSelWarps + 1) * 32);
    if (P.carry) {
        set_max_smem((const void*)ard::select_kernel<true>, 0);
        ard::select_kernel<true><<<grid, block, smem, s>>>(P);
    } else {
        set_max_smem((const void*)ard::select_kernel<false>, 1);
        ard::select_kernel<false><<<grid, block, smem, s>>>(P);
    }
    AR_CHECK_LAUNCH("select_kernel");
    return AR_OK;
}

ar_status launch_fused(const ard::SelParams& P, int grid, size_t smem, cudaStream_t s) {
    set_max_smem((const void*)ard::fused_kernel, 2);
    ard::fused_kernel<<<grid, (ard::kSelWarps + 1) * 32, smem, s>>>(P);
    AR_CHECK_LAUNCH("fused_kernel");
    return AR_OK;
}

}  // namespace ar

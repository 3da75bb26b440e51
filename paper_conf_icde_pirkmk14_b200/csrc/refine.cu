// refine.cu -- step a5 (selection refinement, Algorithm 2)
// and step a6 (SUM over exact values).
//
// The candidate list is ascending (stable compaction in a3), so the join with
// the residual is a positional ("invisible") lookup: each
// candidate's residual is gathered at its row position, from HBM or, for
// host-resident residuals, straight over the host link through a mapped
// pointer.  Each thread owns 8 consecutive candidates (two 16-B loads of
// positions and of aux words), so its residual gathers are independent loads
// in flight together.  Refine keeps order with the same decoupled look-back
// as a3; refine+SUM needs no order (integer sums are exact in any order).
#include "rl_common.cuh"

namespace ard {

// Exact re-evaluation of a non-definite candidate (Alg. 2: join with the
// residual, "+bw" concatenation, CONDITION).
__device__ __forceinline__ bool refine_keep(const RefParams& P, uint32_t pos, uint32_t aux) {
    if (aux & AR_AUX_DEFINITE) return true;
    bool ok = true;
    for (int c = 0; c < P.npred; ++c) {
        const RefPred& p = P.p[c];
        if (!p.check) continue;
        const uint32_t m = p.carried ? ((aux >> p.ashift) & (p.w == 32 ? 0xffffffffu : ((1u << p.w) - 1u)))
                                     : major_get(p.major, pos, p.w, p.layout);
        const uint32_t r = residual_get(p.residual, pos, p.k, p.rlayout);
        const uint32_t v = ((m << p.k) | r) + p.base;
        ok = ok && (v >= p.lo) && (v <= p.hi);
    }
    return ok;
}

__device__ __forceinline__ uint32_t agg_value_at(const RefParams& P, const AggCol& a, uint32_t pos, uint32_t aux) {
    if (a.pred >= 0 && P.p[a.pred].carried) {
        const RefPred& p = P.p[a.pred];
        const uint32_t m = (aux >> p.ashift) & (p.w == 32 ? 0xffffffffu : ((1u << p.w) - 1u));
        const uint32_t r = a.k ? residual_get(a.residual, pos, a.k, a.rlayout) : 0u;
        return ((m << a.k) | r) + a.base;
    }
    return agg_gather(a, pos);
}

__device__ __forceinline__ void load8(const uint32_t* base, uint64_t j0, long long count, uint32_t (&v)[8]) {
    if (j0 + 8 <= (uint64_t)count) {
        const uint4 a = *reinterpret_cast<const uint4*>(base + j0);
        const uint4 b = *reinterpret_cast<const uint4*>(base + j0 + 4);
        v[0] = a.x; v[1] = a.y; v[2] = a.z; v[3] = a.w;
        v[4] = b.x; v[5] = b.y; v[6] = b.z; v[7] = b.w;
    } else {
#pragma unroll
        for (int i = 0; i < 8; ++i) v[i] = (j0 + i < (uint64_t)count) ? base[j0 + i] : 0u;
    }
}

// Batched gathers of 8 candidates' parts (predicated, non-volatile loads: the
// 8 candidates' loads of one step are in flight together).
// SLICED part of width w at rows pos[i] where (pred >> i) & 1: w/4 vector steps
// (a 32-row block's w planes are contiguous; w % 4 == 0 keeps them 16-B aligned),
// otherwise word by word.
template <bool kWide = false>   // kWide: the w == 8 case with both 16-B halves in flight (128 registers)
__device__ __forceinline__ void sliced_batch8(const uint32_t* s, const uint32_t (&pos)[8], uint32_t pred, int w,
                                              uint32_t (&out)[8]) {
#pragma unroll
    for (int i = 0; i < 8; ++i) out[i] = 0u;
    if (kWide && w == 8) {   // both 16-B halves of every block in flight together (one gather latency, not two)
        uint4 a[8], b[8];
#pragma unroll
        for (int i = 0; i < 8; ++i) {
            a[i] = ld_gather_if4(s + (uint64_t)(pos[i] >> 5) * 8, (pred >> i) & 1u);
            b[i] = ld_gather_if4(s + (uint64_t)(pos[i] >> 5) * 8 + 4, (pred >> i) & 1u);
        }
#pragma unroll
        for (int i = 0; i < 8; ++i) {
            const uint32_t x[8] = {a[i].x, a[i].y, a[i].z, a[i].w, b[i].x, b[i].y, b[i].z, b[i].w};
            out[i] = rl::row_bits<8>(x, pos[i] & 31u);
        }
    } else if ((w & 3) == 0) {
        for (int q = 0; q < w / 4; ++q) {
            uint4 a[8];
#pragma unroll
            for (int i = 0; i < 8; ++i) a[i] = ld_gather_if4(s + (uint64_t)(pos[i] >> 5) * w + 4 * q, (pred >> i) & 1u);
#pragma unroll
            for (int i = 0; i < 8; ++i) {
                const uint32_t l = pos[i] & 31u;
                const uint32_t x[4] = {a[i].x, a[i].y, a[i].z, a[i].w};
                out[i] |= rl::row_bits<4>(x, l) << (4 * q);
            }
        }
    } else {
        for (int j = 0; j < w; ++j) {
            uint32_t a[8];
#pragma unroll
            for (int i = 0; i < 8; ++i) a[i] = ld_gather_if(s + (uint64_t)(pos[i] >> 5) * w + j, (pred >> i) & 1u);
#pragma unroll
            for (int i = 0; i < 8; ++i) out[i] |= ((a[i] >> (pos[i] & 31u)) & 1u) << j;
        }
    }
}
template <bool kWide = false>
__device__ __forceinline__ void part_batch8(const uint32_t* s, const uint32_t (&pos)[8], uint32_t pred, int w,
                                            int layout, uint32_t (&out)[8]) {
    if (w == 0) {
#pragma unroll
        for (int i = 0; i < 8; ++i) out[i] = 0u;
    } else if (layout == AR_LAYOUT_SLICED) {
        sliced_batch8<kWide>(s, pos, pred, w, out);
    } else if ((layout & 0xff) == AR_LAYOUT_SLICED) {   // split residual planes
#pragma unroll
        for (int i = 0; i < 8; ++i) out[i] = residual_get_if(s, pos[i], w, layout, (pred >> i) & 1u);
    } else {
#pragma unroll
        for (int i = 0; i < 8; ++i) out[i] = packed_get_if(s, pos[i], w, (pred >> i) & 1u);
    }
}

// Alg. 2 on 8 candidates: definite ones are kept untouched;
// every non-definite one is joined with its residual (and, when the
// approximation is not carried, its major) and re-evaluated exactly.
template <bool kWide = false>
__device__ __forceinline__ uint32_t refine_batch8(const RefParams& P, const uint32_t (&pos)[8],
                                                  const uint32_t (&aux)[8], uint32_t valid) {
    uint32_t def = 0;
#pragma unroll
    for (int i = 0; i < 8; ++i) def |= (aux[i] >> 31) << i;
    def &= valid;
    uint32_t need = valid & ~def;
    for (int c = 0; c < P.npred && need; ++c) {
        const RefPred& p = P.p[c];
        if (!p.check) continue;
        uint32_t m[8], r[8];
        if (p.carried) {
            const uint32_t mask = p.w == 32 ? 0xffffffffu : ((1u << p.w) - 1u);
#pragma unroll
            for (int i = 0; i < 8; ++i) m[i] = (aux[i] >> p.ashift) & mask;
        } else {
            part_batch8(p.major, pos, need, (int)p.w, (int)p.layout, m);
        }
        part_batch8<kWide>(p.residual, pos, need, (int)p.k, (int)p.rlayout, r);
#pragma unroll
        for (int i = 0; i < 8; ++i) {
            const uint32_t v = (p.k >= 32 ? r[i] : ((m[i] << p.k) | r[i])) + p.base;
            if (!(v >= p.lo && v <= p.hi)) need &= ~(1u << i);
        }
    }
    return def | need;
}

// Ordered refine (positions out).  Persistent CTAs, tile t = blockIdx + i *
// gridDim (2048 candidates), decoupled look-back across tiles (Merrill &
// Garland, lookback_inclusive): each tile publishes its count at once and its
// inclusive prefix when resolved.  Software-pipelined: a tile's kept positions
// wait in shared memory while the CTA refines its next tile (whose candidates
// were loaded one tile ahead), then go out at the resolved offset -- a round
// after the counts around it were published, so the walk is short.  Every CTA
// is resident (cooperative launch), so the counts waited for always come.
// kWide (a checked predicate with an unsplit SLICED 8-plane residual): both 16-B
// halves of every candidate's residual block in flight together -- one gather
// latency per tile instead of two -- at 128 registers (2 CTAs per SM); the
// other shapes keep 4 CTAs per SM.
template <bool kWide>
__global__ void __launch_bounds__(kRefThreads, kWide ? 2 : 4) refine_kernel(const __grid_constant__ RefParams P) {
    __shared__ uint32_t st_pos[2][kRefTile];   // kept positions of the current and the pending tile
    // two sets of warp totals, by tile parity: no barrier follows a tile's block scan, so the next
    // tile's scan must not overwrite totals a slower warp may still be reading
    __shared__ uint32_t warp_tot[2][kRefThreads / 32];
    __shared__ unsigned long long s_off;
    const unsigned warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const long long count = *P.in_count;
    const long long num_tiles = (count + kRefTile - 1) / kRefTile;
    long long pend = -1;                // tile whose positions wait in st_pos[pbuf] for their offset
    uint32_t pend_total = 0, cb = 0, pbuf = 0;
    // Warp 0 writes out the pending tile while the other warps refine the next one (their next
    // block-scan barrier waits for it, which also orders the buffer's reuse): its neighbours'
    // counts were published while this CTA refined, so the look-back is normally short.
    auto resolve_w0 = [&]() {
        const unsigned long long prefix = lookback_inclusive(P.status, pend, pend_total, lane);
        if (lane == 0 && pend == num_tiles - 1) *P.out_count = (long long)(prefix + pend_total);
        const uint32_t* sp = st_pos[pbuf];
        for (uint32_t j = lane; j < pend_total; j += 32) P.out_pos[prefix + j] = sp[j];
    };
    // A pending tile with many kept positions is copied out by the whole CTA (warp 0 alone would
    // hold the CTA up at the next barrier for longer than the barrier here costs).
    auto resolve = [&]() {
        if (pend_total <= (uint32_t)kRefWarpCopy) {
            if (warp == 0) resolve_w0();
            return;
        }
        if (warp == 0) {
            const unsigned long long prefix = lookback_inclusive(P.status, pend, pend_total, lane);
            if (lane == 0) {
                s_off = prefix;
                if (pend == num_tiles - 1) *P.out_count = (long long)(prefix + pend_total);
            }
        }
        __syncthreads();
        const unsigned long long off = s_off;
        const uint32_t* sp = st_pos[pbuf];
        for (uint32_t j = threadIdx.x; j < pend_total; j += kRefThreads) P.out_pos[off + j] = sp[j];
    };
    uint32_t npos[8], naux[8];
    if ((long long)blockIdx.x < num_tiles) {
        const uint64_t j0 = (uint64_t)blockIdx.x * kRefTile + threadIdx.x * kRefPerThread;
        load8(P.in_pos, j0, count, npos);
        load8(P.in_aux, j0, count, naux);
    }
    for (long long t = blockIdx.x; t < num_tiles; t += gridDim.x) {
        const uint64_t j0 = (uint64_t)t * kRefTile + threadIdx.x * kRefPerThread;
        uint32_t pos[8], aux[8];
#pragma unroll
        for (int i = 0; i < 8; ++i) {
            pos[i] = npos[i];
            aux[i] = naux[i];
        }
        if (t + gridDim.x < num_tiles) {
            const uint64_t j1 = j0 + (uint64_t)gridDim.x * kRefTile;
            load8(P.in_pos, j1, count, npos);
            load8(P.in_aux, j1, count, naux);
        }
        uint32_t valid = 0;
#pragma unroll
        for (int i = 0; i < 8; ++i) valid |= (j0 + i < (uint64_t)count ? 1u : 0u) << i;
        const uint32_t keep = refine_batch8<kWide>(P, pos, aux, valid);

        const uint32_t cnt = __popc(keep);
        uint32_t total;
        const uint32_t excl = block_excl_scan<kRefThreads>(cnt, warp_tot[cb], total, 1);
        if (threadIdx.x == 0) st_relaxed(P.status + t, kFlagAgg | total);   // publish the count at once
        uint32_t o = excl;
        uint32_t* sp = st_pos[cb];
#pragma unroll
        for (int i = 0; i < 8; ++i)
            if (keep & (1u << i)) sp[o++] = pos[i];
        if (pend >= 0) resolve();
        pend = t;
        pend_total = total;
        pbuf = cb;
        cb ^= 1u;
    }
    __syncthreads();   // the last tile's positions are staged
    if (pend >= 0) resolve();
}

template <typename T>
__device__ __forceinline__ void block_add(T v, unsigned long long* out) {
    __shared__ unsigned long long red[32];
    unsigned long long x = (unsigned long long)v;
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) x += __shfl_xor_sync(0xffffffffu, x, o);
    const unsigned warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    __syncthreads();
    if (lane == 0) red[warp] = x;
    __syncthreads();
    if (threadIdx.x == 0) {
        unsigned long long s = 0;
        for (unsigned i = 0; i < (blockDim.x + 31) / 32; ++i) s += red[i];
        if (s) atomicAdd(out, s);
    }
}

// Refine + SUM in two batched phases per thread: first every residual the 8
// candidates need (gathers in flight together), then every aggregate value of
// the kept ones -- two dependent round trips per 8 candidates, not 16.  The
// gathers are predicated non-volatile loads (common.cuh: ld_gather_if).
__global__ void __launch_bounds__(kRefThreads, 4) refine_sum_kernel(const __grid_constant__ RefParams P) {
    const long long count = *P.in_count;
    const long long num_tiles = (count + kRefTile - 1) / kRefTile;
    unsigned long long sum = 0, kept = 0;
    for (long long t = blockIdx.x; t < num_tiles; t += gridDim.x) {
        const uint64_t j0 = (uint64_t)t * kRefTile + threadIdx.x * kRefPerThread;
        uint32_t pos[8], aux[8];
        load8(P.in_pos, j0, count, pos);
        load8(P.in_aux, j0, count, aux);
        uint32_t keep = 0, need = 0;
#pragma unroll
        for (int i = 0; i < 8; ++i) {
            if (j0 + i < (uint64_t)count) {
                keep |= 1u << i;
                if (!(aux[i] & AR_AUX_DEFINITE)) need |= 1u << i;
            }
        }
        for (int c = 0; c < P.npred && need; ++c) {   // Alg. 2 on the non-definite candidates
            const RefPred& p = P.p[c];
            if (!p.check) continue;
            uint32_t r[8], m[8];
#pragma unroll
            for (int i = 0; i < 8; ++i) r[i] = residual_get_if(p.residual, pos[i], p.k, p.rlayout, (need >> i) & 1u);
#pragma unroll
            for (int i = 0; i < 8; ++i)
                m[i] = p.carried ? ((aux[i] >> p.ashift) & (p.w == 32 ? 0xffffffffu : ((1u << p.w) - 1u)))
                                 : ((need >> i) & 1u ? major_get(p.major, pos[i], p.w, p.layout) : 0u);
#pragma unroll
            for (int i = 0; i < 8; ++i) {
                const uint32_t v = ((m[i] << p.k) | r[i]) + p.base;
                if (((need >> i) & 1u) && !((v >= p.lo) && (v <= p.hi))) keep &= ~(1u << i);
            }
        }
        kept += __popc(keep);
        if (P.nagg > 0 && keep) {
            unsigned long long prod[8];
#pragma unroll
            for (int i = 0; i < 8; ++i) prod[i] = 1;
            for (int c = 0; c < P.nagg; ++c) {
                const AggCol& a = P.a[c];
                uint32_t v[8];
                if (a.pred >= 0 && P.p[a.pred].carried) {
                    const RefPred& p = P.p[a.pred];
#pragma unroll
                    for (int i = 0; i < 8; ++i) {
                        const uint32_t mm = (aux[i] >> p.ashift) & (p.w == 32 ? 0xffffffffu : ((1u << p.w) - 1u));
                        const uint32_t rr =
                            a.k ? residual_get_if(a.residual, pos[i], a.k, a.rlayout, (keep >> i) & 1u) : 0u;
                        v[i] = ((mm << a.k) | rr) + a.base;
                    }
                } else if (a.k == 0 && a.layout == AR_LAYOUT_PACKED && a.w > 0) {
#pragma unroll
                    for (int i = 0; i < 8; ++i) v[i] = packed_get_if(a.major, pos[i], (int)a.w, (keep >> i) & 1u) + a.base;
                } else {
#pragma unroll
                    for (int i = 0; i < 8; ++i) v[i] = (keep >> i) & 1u ? agg_gather(a, pos[i]) : 0u;
                }
#pragma unroll
                for (int i = 0; i < 8; ++i) prod[i] *= v[i];
            }
#pragma unroll
            for (int i = 0; i < 8; ++i)
                if ((keep >> i) & 1u) sum += prod[i];
        }
    }
    if (P.out_sum) block_add(sum, P.out_sum);
    if (P.out_cnt) block_add(kept, P.out_cnt);
}

// Refine + SUM specialised for one decomposed predicate with a SLICED
// residual of K = 4 / 8 planes (a 32-row block's residual is one 16 / 32-B
// sector) and SUM factors that are k = 0 predicate columns (value in the aux
// word) or at most one bit-packed gathered column (l_extendedprice in Q6).
// Straight-line code (no per-candidate branches), so each thread's gathers are
// in flight together:
//   phase 1: residual sectors of the non-definite candidates AND the gathered
//            factor of the definite ones (kept for sure: Alg. 2 never touches
//            them);
//   phase 2: the gathered factor of the non-definite candidates that survived.
template <int K>
__global__ void __launch_bounds__(kRefThreads, 2) refine_sum_sliced_kernel(const __grid_constant__ RefParams P) {
    const long long count = *P.in_count;
    const long long num_tiles = (count + kRefTile - 1) / kRefTile;
    const RefPred& q = P.p[P.fast_chk];
    const uint32_t qmask = q.w == 32 ? 0xffffffffu : ((1u << q.w) - 1u);
    const int g = P.fast_g;   // gathered factor, or -1
    // two factors, one gathered and one carried predicate column (Q6): its shift / mask / base once
    const int f2 = (P.nagg == 2 && g >= 0) ? 1 - g : -1;
    const uint32_t f2_sh = f2 >= 0 ? P.p[P.a[f2].pred].ashift : 0u;
    const uint32_t f2_w = f2 >= 0 ? P.p[P.a[f2].pred].w : 0u;
    const uint32_t f2_mask = f2_w >= 32 ? 0xffffffffu : ((1u << f2_w) - 1u);
    const uint32_t f2_base = f2 >= 0 ? P.a[f2].base : 0u;
    unsigned long long sum = 0, kept = 0;
    // the next tile's candidates are loaded while this one's gathers are in flight
    uint32_t npos[8], naux[8];
    if (blockIdx.x < num_tiles) {
        const uint64_t j0 = (uint64_t)blockIdx.x * kRefTile + threadIdx.x * kRefPerThread;
        load8(P.in_pos, j0, count, npos);
        load8(P.in_aux, j0, count, naux);
    }
    for (long long t = blockIdx.x; t < num_tiles; t += gridDim.x) {
        const uint64_t j0 = (uint64_t)t * kRefTile + threadIdx.x * kRefPerThread;
        uint32_t pos[8], aux[8];
#pragma unroll
        for (int i = 0; i < 8; ++i) {
            pos[i] = npos[i];
            aux[i] = naux[i];
        }
        if (t + gridDim.x < num_tiles) {
            const uint64_t j1 = (uint64_t)(t + gridDim.x) * kRefTile + threadIdx.x * kRefPerThread;
            load8(P.in_pos, j1, count, npos);
            load8(P.in_aux, j1, count, naux);
        }
        uint32_t valid = 0, def = 0;
#pragma unroll
        for (int i = 0; i < 8; ++i) {
            valid |= (j0 + i < (uint64_t)count ? 1u : 0u) << i;
            def |= (aux[i] >> 31) << i;
        }
        def &= valid;
        const uint32_t need = valid & ~def;
        // phase 1
        uint4 ra[8], rb[8];
#pragma unroll
        for (int i = 0; i < 8; ++i) {
            const uint32_t* blk = q.residual + (uint64_t)(pos[i] >> 5) * K;
            ra[i] = ld_gather_if4(blk, (need >> i) & 1u);
            if constexpr (K == 8) rb[i] = ld_gather_if4(blk + 4, (need >> i) & 1u);
        }
        uint32_t gv[8];
        if (g >= 0) {
            const AggCol& a = P.a[g];
#pragma unroll
            for (int i = 0; i < 8; ++i) gv[i] = packed_get_if(a.major, pos[i], (int)a.w, (def >> i) & 1u);
        }
        uint32_t keep = def;
#pragma unroll
        for (int i = 0; i < 8; ++i) {
            const uint32_t l = pos[i] & 31u;
            uint32_t x[K];
            x[0] = ra[i].x; x[1] = ra[i].y; x[2] = ra[i].z; x[3] = ra[i].w;
            if constexpr (K == 8) {
                x[4] = rb[i].x; x[5] = rb[i].y; x[6] = rb[i].z; x[7] = rb[i].w;
            }
            const uint32_t r = rl::row_bits<K>(x, l);
            const uint32_t v = ((((aux[i] >> q.ashift) & qmask) << K) | r) + q.base;
            keep |= (((need >> i) & 1u) && v >= q.lo && v <= q.hi ? 1u : 0u) << i;
        }
        kept += __popc(keep);
        if (P.nagg == 0 || !keep) continue;
        // phase 2
        if (g >= 0) {
            const AggCol& a = P.a[g];
            const uint32_t late = keep & need;
#pragma unroll
            for (int i = 0; i < 8; ++i) {
                const uint32_t v = packed_get_if(a.major, pos[i], (int)a.w, (late >> i) & 1u);
                gv[i] = ((late >> i) & 1u ? v : gv[i]) + a.base;
            }
        }
        if (f2 >= 0) {   // Q6: the gathered factor times one carried predicate column (shift / mask hoisted)
#pragma unroll
            for (int i = 0; i < 8; ++i)
                if ((keep >> i) & 1u) sum += (unsigned long long)gv[i] * (((aux[i] >> f2_sh) & f2_mask) + f2_base);
            continue;
        }
#pragma unroll
        for (int i = 0; i < 8; ++i) {
            if (!((keep >> i) & 1u)) continue;
            unsigned long long prod = 1;
            for (int c = 0; c < P.nagg; ++c) {
                const AggCol& a = P.a[c];
                if (c == g) {
                    prod *= gv[i];
                } else {
                    const RefPred& p = P.p[a.pred];
                    prod *= ((aux[i] >> p.ashift) & (p.w == 32 ? 0xffffffffu : ((1u << p.w) - 1u))) + a.base;
                }
            }
            sum += prod;
        }
    }
    if (P.out_sum) block_add(sum, P.out_sum);
    if (P.out_cnt) block_add(kept, P.out_cnt);
}

__global__ void __launch_bounds__(kRefThreads) sum_kernel(const __grid_constant__ SumParams P) {
    const long long count = *P.count;
    unsigned long long sum = 0;
    const long long stride = (long long)gridDim.x * kRefThreads;
    for (long long j = (long long)blockIdx.x * kRefThreads + threadIdx.x; j < count; j += stride) {
        const uint32_t pos = P.pos[j];
        unsigned long long prod = 1;
        for (int c = 0; c < P.nagg; ++c) {
            const AggCol& a = P.a[c];
            prod *= agg_gather(a, pos);
        }
        sum += prod;
    }
    block_add(sum, P.out_sum);
}

// MIN / MAX (s IV-F, Fig. 6).  "The result of the
// approximation of a minimum has to assuredly include the tuple ID of the
// actual minimum.  To guarantee this, the error bounds of the applied
// selections are propagated to the aggregation": a definite candidate is
// certainly in R, so (MIN) nothing whose Y major exceeds the smallest definite
// major mD can be the minimum.  Three passes over the candidate relation:
//   minmax_approx_kernel : min / max of Y's major over candidates and over
//                          definite candidates (the approximate answer); each
//                          candidate's Y major is kept in the workspace;
//   minmax_refine_kernel : the candidates with major <= mD (MIN; >= MD for MAX;
//                          every candidate when none is definite) are refined --
//                          Alg. 2 on the predicates, then Y's residual -- and
//                          the exact extreme taken ("a join of the candidate set
//                          with the input residuals and the calculation of the
//                          minimum");
//   minmax_final_kernel  : out7 (values mapped back from the key domain).
__device__ __forceinline__ uint32_t y_major(const MinMaxParams& P, uint32_t pos, uint32_t aux) {
    const AggCol& y = P.y;
    if (y.pred >= 0 && P.r.p[y.pred].carried) {
        const RefPred& p = P.r.p[y.pred];
        return (aux >> p.ashift) & (p.w == 32 ? 0xffffffffu : ((1u << p.w) - 1u));
    }
    return y.w ? major_get(y.major, pos, (int)y.w, (int)y.layout) : 0u;
}

__global__ void minmax_init_kernel(unsigned int* ws, unsigned long long* wc) {
    if (threadIdx.x < 5) ws[threadIdx.x] = (threadIdx.x & 1) && threadIdx.x < 4 ? 0u : 0xffffffffu;
    if (threadIdx.x < 3) wc[threadIdx.x] = 0ull;
}

__global__ void __launch_bounds__(kRefThreads) minmax_approx_kernel(const __grid_constant__ MinMaxParams P) {
    const long long count = *P.r.in_count;
    const long long num_tiles = (count + kRefTile - 1) / kRefTile;
    uint32_t mnC = 0xffffffffu, mxC = 0u, mnD = 0xffffffffu, mxD = 0u;
    unsigned long long nd = 0;
    const AggCol& y = P.y;
    const bool carried = y.pred >= 0 && P.r.p[y.pred].carried;
    for (long long t = blockIdx.x; t < num_tiles; t += gridDim.x) {   // 8 candidates per thread
        const uint64_t j0 = (uint64_t)t * kRefTile + threadIdx.x * kRefPerThread;
        uint32_t pos[8], aux[8], m[8];
        load8(P.r.in_pos, j0, count, pos);
        load8(P.r.in_aux, j0, count, aux);
        uint32_t valid = 0;
#pragma unroll
        for (int i = 0; i < 8; ++i) valid |= (j0 + i < (uint64_t)count ? 1u : 0u) << i;
        if (carried) {
#pragma unroll
            for (int i = 0; i < 8; ++i) m[i] = y_major(P, pos[i], aux[i]);
        } else {
            part_batch8(y.major, pos, valid, (int)y.w, (int)y.layout, m);   // gathers in flight together
        }
#pragma unroll
        for (int i = 0; i < 8; ++i) {
            if (!((valid >> i) & 1u)) continue;
            P.ymaj[j0 + i] = m[i];   // the refine pass reads it back sequentially instead of gathering again
            mnC = min(mnC, m[i]);
            mxC = max(mxC, m[i]);
            if (aux[i] & AR_AUX_DEFINITE) {
                mnD = min(mnD, m[i]);
                mxD = max(mxD, m[i]);
                ++nd;
            }
        }
    }
    mnC = __reduce_min_sync(0xffffffffu, mnC);
    mxC = __reduce_max_sync(0xffffffffu, mxC);
    mnD = __reduce_min_sync(0xffffffffu, mnD);
    mxD = __reduce_max_sync(0xffffffffu, mxD);
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) nd += __shfl_xor_sync(0xffffffffu, nd, o);
    if ((threadIdx.x & 31) == 0) {
        atomicMin(P.ws + 0, mnC);
        atomicMax(P.ws + 1, mxC);
        atomicMin(P.ws + 2, mnD);
        atomicMax(P.ws + 3, mxD);
        if (nd) atomicAdd(P.wc + 0, nd);
    }
}

__global__ void __launch_bounds__(kRefThreads) minmax_refine_kernel(const __grid_constant__ MinMaxParams P) {
    const long long count = *P.r.in_count;
    const bool any_def = __ldcg(P.wc + 0) != 0ull;
    const bool is_min = P.mode == AR_MIN;
    // refine threshold: MIN keeps m <= (D ? min_D : max_C), MAX keeps m >= (D ? max_D : min_C)
    const uint32_t thr = is_min ? (any_def ? __ldcg(P.ws + 2) : __ldcg(P.ws + 1))
                                : (any_def ? __ldcg(P.ws + 3) : __ldcg(P.ws + 0));
    uint32_t best = 0xffffffffu;   // exact key, complemented for MAX
    unsigned long long nref = 0, surv = 0;
    const long long stride = (long long)gridDim.x * kRefThreads;
    for (long long j = (long long)blockIdx.x * kRefThreads + threadIdx.x; j < count; j += stride) {
        const uint32_t m = __ldcs(P.ymaj + j);
        if (is_min ? m > thr : m < thr) continue;
        const uint32_t pos = P.r.in_pos[j], aux = P.r.in_aux[j];
        ++nref;
        if (!refine_keep(P.r, pos, aux)) continue;
        ++surv;
        const uint32_t r = P.y.k ? residual_get(P.y.residual, pos, (int)P.y.k, (int)P.y.rlayout) : 0u;
        const uint32_t key = (P.y.k >= 32 ? r : ((m << P.y.k) | r)) + P.y.base;
        best = min(best, is_min ? key : ~key);
    }
    best = __reduce_min_sync(0xffffffffu, best);
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) {
        nref += __shfl_xor_sync(0xffffffffu, nref, o);
        surv += __shfl_xor_sync(0xffffffffu, surv, o);
    }
    if ((threadIdx.x & 31) == 0) {
        if (surv) {
            atomicMin(P.ws + 4, best);
            atomicAdd(P.wc + 2, surv);
        }
        if (nref) atomicAdd(P.wc + 1, nref);
    }
}

__device__ __forceinline__ long long key_value(uint32_t key, uint32_t flip) {
    const uint32_t v = key ^ flip;
    return flip ? (long long)(int32_t)v : (long long)v;
}

__global__ void minmax_final_kernel(const __grid_constant__ MinMaxParams P) {
    if (threadIdx.x != 0) return;
    const long long nc = *P.r.in_count;
    const unsigned long long nd = P.wc[0];
    const bool is_min = P.mode == AR_MIN;
    const AggCol& y = P.y;
    const uint64_t two_k = 1ull << y.k;
    long long lo = 0, hi = 0;
    if (nc > 0) {
        const uint64_t mlo = is_min ? P.ws[0] : (nd ? P.ws[3] : P.ws[0]);   // bucket whose bottom bounds it
        const uint64_t mhi = is_min ? (nd ? P.ws[2] : P.ws[1]) : P.ws[1];   // bucket whose top bounds it
        const uint64_t klo = (uint64_t)y.base + mlo * two_k;
        uint64_t khi = (uint64_t)y.base + mhi * two_k + two_k - 1;
        if (khi > 0xffffffffull) khi = 0xffffffffull;
        lo = key_value((uint32_t)klo, y.flip);
        hi = key_value((uint32_t)khi, y.flip);
    }
    const unsigned long long surv = P.wc[2];
    const uint32_t best = is_min ? P.ws[4] : ~P.ws[4];
    P.out7[0] = surv ? key_value(best, y.flip) : 0;
    P.out7[1] = (long long)surv;
    P.out7[2] = lo;
    P.out7[3] = hi;
    P.out7[4] = (long long)P.wc[1];
    P.out7[5] = (long long)nd;
    P.out7[6] = nc;
}

// Grouped COUNT / SUM (s IV-E/F; Fig. 4 "select count(*)
// from R where A<5 groupby B" with B GPU-resident).  The paper expects group
// keys to be low-cardinality columns kept whole on the GPU,
// so the approximate pre-grouping is already exact and only the selection's
// false positives must be removed before aggregating: 8 candidates per
// thread are refined (refine_batch8), their keys and factors gathered in one
// batch, and accumulated into per-CTA group tables in shared memory (the
// "grouping table"; group id = key value, so no hash probing), flushed with
// one global atomic per non-empty group and CTA.
__device__ __forceinline__ void factor_batch8(const RefParams& P, const AggCol& a, const uint32_t (&pos)[8],
                                              const uint32_t (&aux)[8], uint32_t pred, uint32_t (&v)[8]) {
    if (a.pred >= 0 && P.p[a.pred].carried && a.k == 0) {
        const RefPred& p = P.p[a.pred];
        const uint32_t mask = p.w == 32 ? 0xffffffffu : ((1u << p.w) - 1u);
#pragma unroll
        for (int i = 0; i < 8; ++i) v[i] = ((aux[i] >> p.ashift) & mask) + a.base;
    } else if (a.k == 0) {
        part_batch8(a.major, pos, pred, (int)a.w, (int)a.layout, v);
#pragma unroll
        for (int i = 0; i < 8; ++i) v[i] += a.base;
    } else {
#pragma unroll
        for (int i = 0; i < 8; ++i) v[i] = (pred >> i) & 1u ? agg_value_at(P, a, pos[i], aux[i]) : 0u;
    }
}

constexpr int kGroupRepMax = 256;   // up to this many groups every warp gets its own table

__global__ void __launch_bounds__(kRefThreads, 2) group_sum_kernel(const __grid_constant__ GroupParams P) {
    extern __shared__ unsigned long long gtab_all[];   // per table: [ngroups] sums, [ngroups] counts
    const int G = P.ngroups;
    // few groups: one table per warp, so the atomics of a hot group contend within a warp only
    const int nrep = G <= kGroupRepMax ? kRefThreads / 32 : 1;
    for (int g = threadIdx.x; g < 2 * G * nrep; g += kRefThreads) gtab_all[g] = 0ull;
    __syncthreads();
    unsigned long long* gtab = gtab_all + (nrep > 1 ? (threadIdx.x >> 5) * 2 * G : 0);
    const long long count = *P.r.in_count;
    const long long num_tiles = (count + kRefTile - 1) / kRefTile;
    for (long long t = blockIdx.x; t < num_tiles; t += gridDim.x) {
        const uint64_t j0 = (uint64_t)t * kRefTile + threadIdx.x * kRefPerThread;
        uint32_t pos[8], aux[8];
        load8(P.r.in_pos, j0, count, pos);
        load8(P.r.in_aux, j0, count, aux);
        uint32_t valid = 0;
#pragma unroll
        for (int i = 0; i < 8; ++i) valid |= (j0 + i < (uint64_t)count ? 1u : 0u) << i;
        const uint32_t keep = refine_batch8<true>(P.r, pos, aux, valid);   // 8-plane residual halves together
        if (!keep) continue;
        uint32_t key[8];
        if (P.gids) {   // ids of the approximation group operator, aligned with the candidates
            uint32_t g8[8];
            load8(P.gids, j0, count, g8);
#pragma unroll
            for (int i = 0; i < 8; ++i) key[i] = g8[i] < (uint32_t)G ? g8[i] : 0u;
        } else {
            factor_batch8(P.r, P.key, pos, aux, keep, key);
        }
        unsigned long long prod[8];
#pragma unroll
        for (int i = 0; i < 8; ++i) prod[i] = 1ull;
        for (int c = 0; c < P.r.nagg; ++c) {
            uint32_t v[8];
            factor_batch8(P.r, P.r.a[c], pos, aux, keep, v);
#pragma unroll
            for (int i = 0; i < 8; ++i) prod[i] *= v[i];
        }
#pragma unroll
        for (int i = 0; i < 8; ++i) {
            if (!((keep >> i) & 1u)) continue;
            if (P.r.nagg > 0) atomicAdd(gtab + key[i], prod[i]);
            atomicAdd(gtab + G + key[i], 1ull);
        }
    }
    __syncthreads();
    for (int g = threadIdx.x; g < G; g += kRefThreads) {
        unsigned long long sm = 0, c = 0;
        for (int r = 0; r < nrep; ++r) {
            sm += gtab_all[r * 2 * G + g];
            c += gtab_all[r * 2 * G + G + g];
        }
        if (c) {
            if (P.r.nagg > 0) atomicAdd(P.out + g, sm);
            atomicAdd(P.out + G + g, c);
        }
    }
}

// sumapproximate (Fig. 7 bwd.sumapproximate): the approximate
// answer from the approximation subplan alone, before any residual is read
// (PAPER.md:360-362, 894-897), as strict error bounds.  With
// definite <= R <= candidates and each value in its bucket
// [b + m 2^k, b + m 2^k + 2^k - 1]:
//   sum_lo = sum_{definite} prod_c bucket_min_c  <=  SUM(R)  <=  sum_hi = sum_{cand} prod_c bucket_max_c
//   count_lo = |definite| <= |R| <= count_hi = |candidates|
__device__ __forceinline__ void bucket_bounds(const AggCol& a, uint32_t p, unsigned long long& lo,
                                              unsigned long long& hi) {
    const uint32_t m = a.w ? major_get(a.major, p, (int)a.w, (int)a.layout) : 0u;
    lo = ((unsigned long long)m << a.k) + a.base;
    hi = lo + ((1ull << a.k) - 1ull);
    if (hi > 0xffffffffull) hi = 0xffffffffull;
}

__global__ void __launch_bounds__(kRefThreads) approx_sum_kernel(const __grid_constant__ ApproxSumParams P) {
    const long long count = *P.count;
    unsigned long long slo = 0, shi = 0, ndef = 0;
    const long long stride = (long long)gridDim.x * kRefThreads;
    for (long long j = (long long)blockIdx.x * kRefThreads + threadIdx.x; j < count; j += stride) {
        const uint32_t pos = P.pos[j];
        const bool def = (P.aux[j] & AR_AUX_DEFINITE) != 0;
        ndef += def;
        if (P.nagg > 0) {
            unsigned long long plo = 1, phi = 1;
            for (int c = 0; c < P.nagg; ++c) {
                unsigned long long lo, hi;
                bucket_bounds(P.a[c], pos, lo, hi);
                plo *= lo;
                phi *= hi;
            }
            shi += phi;
            if (def) slo += plo;
        }
    }
    block_add(slo, &P.out4[0]);
    block_add(shi, &P.out4[1]);
    block_add(ndef, &P.out4[2]);
    if (blockIdx.x == 0 && threadIdx.x == 0) P.out4[3] = (unsigned long long)count;
}

// Positional projection (Fig. 7 bwd.leftjoinapproximate / bwd.leftjoinrefine,
// PAPER.md:884-889; invisible join on positions):
// out[j] = value of column a at row pos[j] -- exact ((major << k) | residual) + b,
// or its approximation b + (major << k) (the bucket minimum; error in [0, 2^k - 1]).
__global__ void __launch_bounds__(kRefThreads) project_kernel(const __grid_constant__ ProjectParams P) {
    const long long count = *P.count;
    const long long stride = (long long)gridDim.x * kRefThreads;
    for (long long j = (long long)blockIdx.x * kRefThreads + threadIdx.x; j < count; j += stride) {
        const uint32_t p = P.pos[j];
        uint32_t v;
        if (P.exact) {
            v = agg_gather(P.a, p);
        } else {
            const uint32_t m = P.a.w ? major_get(P.a.major, p, (int)P.a.w, (int)P.a.layout) : 0u;
            v = (m << P.a.k) + P.a.base;
        }
        P.out[j] = v ^ P.a.flip;   // back from the key domain of a signed column
    }
}

}  // namespace ard

namespace ar {

const void* refine_kernel_fn(bool wide) {
    return wide ? (const void*)ard::refine_kernel<true> : (const void*)ard::refine_kernel<false>;
}
// Cooperative: the look-back (lookback_inclusive) waits on tiles of other
// CTAs, so the whole grid must be co-resident; a cooperative launch guarantees
// that or fails (cudaErrorCooperativeLaunchTooLarge, e.g. under an MPS SM
// limit or beside a persistent kernel) rather than hanging.
ar_status launch_refine(const ard::RefParams& P, int grid, bool wide, cudaStream_t s) {
    void* args[] = {const_cast<ard::RefParams*>(&P)};
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = dim3(grid);
    cfg.blockDim = dim3(ard::kRefThreads);
    cfg.stream = s;
    cudaLaunchAttribute attr[1];
    attr[0].id = cudaLaunchAttributeCooperative;
    attr[0].val.cooperative = 1;
    cfg.attrs = attr;
    cfg.numAttrs = 1;
    AR_TRY_CUDA(cudaLaunchKernelExC(&cfg, refine_kernel_fn(wide), args));
    return AR_OK;
}
ar_status launch_refine_sum(const ard::RefParams& P, int grid, cudaStream_t s) {
    if (P.fast_k == 8 || P.fast_k == 4) {
        const void* fn = P.fast_k == 8 ? (const void*)ard::refine_sum_sliced_kernel<8>
                                       : (const void*)ard::refine_sum_sliced_kernel<4>;
        int occ = 0;
        cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, fn, ard::kRefThreads, 0);
        const int g2 = std::max(1, std::min(grid, num_sms() * std::max(occ, 1)));
        ard::RefParams Q = P;
        void* args[] = {&Q};
        AR_TRY_CUDA(cudaLaunchKernel(fn, dim3(g2), dim3(ard::kRefThreads), args, 0, s));
        return AR_OK;
    }
    ard::refine_sum_kernel<<<grid, ard::kRefThreads, 0, s>>>(P);
    AR_CHECK_LAUNCH("refine_sum_kernel");
    return AR_OK;
}
ar_status launch_sum(const ard::SumParams& P, int grid, cudaStream_t s) {
    ard::sum_kernel<<<grid, ard::kRefThreads, 0, s>>>(P);
    AR_CHECK_LAUNCH("sum_kernel");
    return AR_OK;
}
ar_status launch_approx_sum(const ard::ApproxSumParams& P, int grid, cudaStream_t s) {
    ard::approx_sum_kernel<<<grid, ard::kRefThreads, 0, s>>>(P);
    AR_CHECK_LAUNCH("approx_sum_kernel");
    return AR_OK;
}
ar_status launch_project(const ard::ProjectParams& P, int grid, cudaStream_t s) {
    ard::project_kernel<<<grid, ard::kRefThreads, 0, s>>>(P);
    AR_CHECK_LAUNCH("project_kernel");
    return AR_OK;
}
ar_status launch_minmax(const ard::MinMaxParams& P, int grid, cudaStream_t s) {
    ard::minmax_init_kernel<<<1, 32, 0, s>>>(P.ws, P.wc);
    AR_CHECK_LAUNCH("minmax_init_kernel");
    ard::minmax_approx_kernel<<<grid, ard::kRefThreads, 0, s>>>(P);
    AR_CHECK_LAUNCH("minmax_approx_kernel");
    ard::minmax_refine_kernel<<<grid, ard::kRefThreads, 0, s>>>(P);
    AR_CHECK_LAUNCH("minmax_refine_kernel");
    ard::minmax_final_kernel<<<1, 32, 0, s>>>(P);
    AR_CHECK_LAUNCH("minmax_final_kernel");
    return AR_OK;
}
ar_status launch_group_sum(const ard::GroupParams& P, int grid, cudaStream_t s) {
    const int nrep = P.ngroups <= ard::kGroupRepMax ? ard::kRefThreads / 32 : 1;
    const size_t smem = (size_t)2 * P.ngroups * nrep * sizeof(unsigned long long);
    if (smem > 48 * 1024) {
        AR_TRY_CUDA(cudaFuncSetAttribute((const void*)ard::group_sum_kernel,
                                         cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem));
    }
    ard::group_sum_kernel<<<grid, ard::kRefThreads, smem, s>>>(P);
    AR_CHECK_LAUNCH("group_sum_kernel");
    return AR_OK;
}

}  // namespace ar

// rl_common.cuh -- device helpers of the persistent TMA-pipelined one-pass
// kernel (fused.cu): compile-time decomposition shapes, shared-memory plane
// loads and the bit-plane range tests of step a3.
#pragma once
#include <type_traits>

#include "kernels.cuh"

namespace ard {
namespace rl {

template <int I>
using ic = std::integral_constant<int, I>;
template <int N, int I = 0, class F>
__device__ __forceinline__ void static_for(F&& f) {
    if constexpr (I < N) {
        f(ic<I>{});
        static_for<N, I + 1>(f);
    }
}

// Decomposition shape: per predicate (h << 12) | (w_major << 6) | residual
// width k, h > 0 for a split residual whose h high planes are streamed (the
// k - h low planes are gathered for the rows the high planes leave undecided).
template <int... WK>
struct Shape {
    static constexpr bool kDynamic = false;
    static constexpr int N = sizeof...(WK);
    static constexpr int w(int c) {
        constexpr int a[] = {((WK >> 6) & 63)..., 0};
        return a[c];
    }
    static constexpr int k(int c) {
        constexpr int a[] = {(WK & 63)..., 0};
        return a[c];
    }
    static constexpr int h(int c) {
        constexpr int a[] = {((WK >> 12) & 15)..., 0};
        return a[c];
    }
    static constexpr int split() {   // the one predicate with a split residual, or -1
        for (int i = 0; i < N; ++i)
            if (h(i) > 0) return i;
        return -1;
    }
    static constexpr int kl() { return split() < 0 ? 0 : k(split()) - h(split()); }   // gathered low planes
    static constexpr int pk() {      // the one predicate with a bit-packed residual (k > 8), or -1
        for (int i = 0; i < N; ++i)
            if (k(i) > 8) return i;
        return -1;
    }
    static constexpr int rk(int c) { return k(c) <= 8 ? k(c) : 0; }   // SLICED residual words per block
    static constexpr int off(int c) {   // global plane index of predicate c (its ashift)
        int o = 0;
        for (int i = 0; i < c; ++i) o += w(i);
        return o;
    }
    static constexpr int kofs(int c) {  // first SLICED residual word of predicate c in a block's residual words
        int o = 0;
        for (int i = 0; i < c; ++i) o += rk(i);
        return o;
    }
    static constexpr int ksum() { return kofs(N); }
};

// Runtime shape (any widths, any number of predicates): the one-pass kernel
// reads widths, plane offsets and bounds from the parameters.  Selected with
// the sentinel shape WK = {-1} for decompositions without a compiled shape.
struct DynShape {
    static constexpr bool kDynamic = true;
    static constexpr int N = 0;
    static constexpr int split() { return -1; }   // split / packed residuals need a compiled shape
    static constexpr int kl() { return 0; }
    static constexpr int pk() { return -1; }
};
template <int... WK>
struct ShapeOf {
    using type = Shape<WK...>;
};
template <>
struct ShapeOf<-1> {
    using type = DynShape;
};

// The K residual words of SLICED block `gblk` (K <= 8 planes, K words at
// res + gblk * K), as predicated gathers (.L2::64B): issued for the blocks
// that hold a non-definite candidate, consumed a tile later.
template <int K>
__device__ __forceinline__ void res_issue(uint32_t* r, const uint32_t* res, uint64_t gblk, bool pred, bool hint) {
    const uint32_t* p = res + gblk * K;
    if constexpr (K % 4 == 0) {
#pragma unroll
        for (int q = 0; q < K / 4; ++q) {
            const uint4 v = hint ? ld_gather_if4(p + 4 * q, pred) : ld_gather_if4_nh(p + 4 * q, pred);
            r[4 * q] = v.x; r[4 * q + 1] = v.y; r[4 * q + 2] = v.z; r[4 * q + 3] = v.w;
        }
    } else {
#pragma unroll
        for (int j = 0; j < K; ++j) r[j] = hint ? ld_gather_if(p + j, pred) : ld_gather_if_nh(p + j, pred);
    }
}

// W consecutive 32-bit words from shared memory, vectorised as far as the
// width allows (a block's planes start at a multiple of W words).
template <int W>
__device__ __forceinline__ void lds_words(uint32_t (&x)[W], const uint32_t* p) {
    if constexpr (W % 4 == 0) {
#pragma unroll
        for (int q = 0; q < W / 4; ++q) {
            const uint4 v = reinterpret_cast<const uint4*>(p)[q];
            x[4 * q] = v.x; x[4 * q + 1] = v.y; x[4 * q + 2] = v.z; x[4 * q + 3] = v.w;
        }
    } else if constexpr (W % 2 == 0) {
#pragma unroll
        for (int q = 0; q < W / 2; ++q) {
            const uint2 v = reinterpret_cast<const uint2*>(p)[q];
            x[2 * q] = v.x; x[2 * q + 1] = v.y;
        }
    } else {
#pragma unroll
        for (int j = 0; j < W; ++j) x[j] = p[j];
    }
}

// Borrow steps (see select.cu): v < lo iff v - lo borrows out of the top plane.
__device__ __forceinline__ uint32_t bsub(uint32_t x, uint32_t cbit, uint32_t b) {
    uint32_t d;
    asm("lop3.b32 %0, %1, %2, %3, 0x8E;" : "=r"(d) : "r"(x), "r"(cbit), "r"(b));
    return d;
}
__device__ __forceinline__ uint32_t brsub(uint32_t x, uint32_t cbit, uint32_t b) {
    uint32_t d;
    asm("lop3.b32 %0, %1, %2, %3, 0xB2;" : "=r"(d) : "r"(x), "r"(cbit), "r"(b));
    return d;
}

// Value of row l from W planes held in registers.
template <int W>
__device__ __forceinline__ uint32_t row_of(const uint32_t (&x)[W], uint32_t l) {
    uint32_t v = 0;
#pragma unroll
    for (int j = 0; j < W; ++j) v |= ((x[j] >> l) & 1u) << j;
    return v;
}

// Bits l of planes x[0..W) as a W-bit value (bit j from plane j): two
// instructions per plane -- shift the plane's bit l down to bit 0, then funnel
// it into the top of the accumulator -- and one final shift.
template <int W>
__device__ __forceinline__ uint32_t row_bits(const uint32_t (&x)[W], uint32_t l) {
    uint32_t acc = 0;
#pragma unroll
    for (int j = 0; j < W; ++j) acc = __funnelshift_r(acc, x[j] >> l, 1);
    return W >= 32 ? acc : acc >> (32 - W);
}

// Per-block evaluation of every predicate on the 32 rows of block `blk` of a
// stage (vm = valid rows): candidate mask cm (major in the candidate range of
// every predicate), definite mask dm (major in the definite range of every
// decomposed predicate, candidate range otherwise) and -- with kExact, for
// shapes whose residual planes are streamed (K = residual width) -- the exact
// mask em: one borrow chain over the residual then the major planes (the
// bitwise concatenation "+bw") against the exact bounds.
// Without kExact, K > 0 only marks a decomposed predicate.  A split residual
// (H = S::h(C) > 0, its H high planes streamed): em gets the candidate rows of
// the relaxation at granularity 2^(K-H) over (major << H | high planes), and um
// the ones of them that are not definite there -- the rows whose K - H low
// planes decide (progressive refinement, DESIGN s6.3d), as ul | uh: ul = below
// the fine definite range (fine bucket of the lower bound), uh = above it (that
// of the upper bound) -- setup_scan encodes the ranges so, see api.cu.
template <class S, bool kExact>
__device__ __forceinline__ void eval_block(const SelParams& P, const uint32_t* stg, uint32_t blk, uint32_t vm,
                                           uint32_t& cm, uint32_t& dm, uint32_t& em, uint32_t& ul, uint32_t& uh) {
    cm = dm = em = vm;
    ul = uh = 0u;
    static_for<S::N>([&](auto cc) {
        constexpr int C = decltype(cc)::value;
        constexpr int W = S::w(C), K = S::k(C), O = S::off(C);
        uint32_t x[W];
        lds_words<W>(x, stg + P.p[C].soff + blk * W);
        uint32_t cl = 0, ch = 0;
#pragma unroll
        for (int j = 0; j < W; ++j) {
            cl = bsub(x[j], P.pm[O + j][0], cl);
            ch = brsub(x[j], P.pm[O + j][1], ch);
        }
        const uint32_t c = ~(cl | ch);
        cm &= c;
        if constexpr (K == 0) {   // k = 0: candidate = definite = exact
            dm &= c;
            em &= c;
        } else {
            uint32_t dl = 0, dh = 0;   // mode 2 (no definite bucket) has empty bounds in pm
#pragma unroll
            for (int j = 0; j < W; ++j) {
                dl = bsub(x[j], P.pm[O + j][2], dl);
                dh = brsub(x[j], P.pm[O + j][3], dh);
            }
            dm &= ~(dl | dh);
            if constexpr (K > 8) {   // bit-packed residual (gathered-residual kernel): the check code bits
                ul = dl;
                uh = dh;
            }
            if constexpr (kExact && S::h(C) > 0) {
                constexpr int H = S::h(C);
                uint32_t r[H];
                lds_words<H>(r, stg + P.p[C].res_soff + blk * H);
                uint32_t fl = 0, fh = 0, gl = 0, gh = 0;
#pragma unroll
                for (int j = 0; j < H; ++j) {
                    fl = bsub(r[j], P.pmh[C][j][0], fl);
                    fh = brsub(r[j], P.pmh[C][j][1], fh);
                    gl = bsub(r[j], P.pmh[C][j][2], gl);
                    gh = brsub(r[j], P.pmh[C][j][3], gh);
                }
#pragma unroll
                for (int j = 0; j < W; ++j) {
                    fl = bsub(x[j], P.pmh[C][H + j][0], fl);
                    fh = brsub(x[j], P.pmh[C][H + j][1], fh);
                    gl = bsub(x[j], P.pmh[C][H + j][2], gl);
                    gh = brsub(x[j], P.pmh[C][H + j][3], gh);
                }
                em &= ~(fl | fh);
                ul = gl;
                uh = gh;
            } else if constexpr (kExact) {
                uint32_t r[K];
                lds_words<K>(r, stg + P.p[C].res_soff + blk * K);
                uint32_t el = 0, eh = 0;
#pragma unroll
                for (int j = 0; j < K; ++j) {
                    el = bsub(r[j], P.pmx[C][j][0], el);
                    eh = brsub(r[j], P.pmx[C][j][1], eh);
                }
#pragma unroll
                for (int j = 0; j < W; ++j) {
                    el = bsub(x[j], P.pmx[C][K + j][0], el);
                    eh = brsub(x[j], P.pmx[C][K + j][1], eh);
                }
                em &= ~(el | eh);
            }
        }
    });
}

// eval_block for a runtime shape: the same borrow chains with the widths and
// bound masks of the parameters (residual planes streamed where res_stream).
__device__ __forceinline__ void eval_block_dyn(const SelParams& P, const uint32_t* stg, uint32_t blk, uint32_t vm,
                                               uint32_t& cm, uint32_t& dm, uint32_t& em) {
    cm = dm = em = vm;
    for (int c = 0; c < P.npred; ++c) {
        const SelPred& p = P.p[c];
        const uint32_t W = p.w, O = p.ashift;
        const uint32_t* xp = stg + p.soff + blk * W;
        uint32_t cl = 0, ch = 0, dl = 0, dh = 0;
        for (uint32_t j = 0; j < W; ++j) {
            const uint32_t x = xp[j];
            cl = bsub(x, P.pm[O + j][0], cl);
            ch = brsub(x, P.pm[O + j][1], ch);
            dl = bsub(x, P.pm[O + j][2], dl);
            dh = brsub(x, P.pm[O + j][3], dh);
        }
        const uint32_t cc = ~(cl | ch);
        cm &= cc;
        if (p.k == 0) {
            dm &= cc;
            em &= cc;
            continue;
        }
        dm &= ~(dl | dh);
        if (!p.res_stream) {   // the dynamic kernel runs in exact mode only (every residual streamed)
            em = 0u;
            continue;
        }
        const uint32_t K = p.k;
        const uint32_t* rp = stg + p.res_soff + blk * K;
        uint32_t el = 0, eh = 0;
        for (uint32_t j = 0; j < K; ++j) {
            const uint32_t r = rp[j];
            el = bsub(r, P.pmx[c][j][0], el);
            eh = brsub(r, P.pmx[c][j][1], eh);
        }
        for (uint32_t j = 0; j < W; ++j) {
            const uint32_t x = xp[j];
            el = bsub(x, P.pmx[c][K + j][0], el);
            eh = brsub(x, P.pmx[c][K + j][1], eh);
        }
        em &= ~(el | eh);
    }
}

// Exact value of predicate c's column at row l of block blk from the stage (runtime shape).
__device__ __forceinline__ uint32_t stage_value_dyn(const SelParams& P, const uint32_t* stg, int c, uint32_t blk,
                                                    uint32_t l) {
    const SelPred& p = P.p[c];
    uint32_t m = 0;
    const uint32_t* xp = stg + p.soff + blk * p.w;
    for (uint32_t j = 0; j < p.w; ++j) m |= ((xp[j] >> l) & 1u) << j;
    if (p.k > 0 && p.res_stream) {
        uint32_t r = 0;
        const uint32_t* rp = stg + p.res_soff + blk * p.k;
        for (uint32_t j = 0; j < p.k; ++j) r |= ((rp[j] >> l) & 1u) << j;
        return ((m << p.k) | r) + p.base;
    }
    return m + p.base;
}

}  // namespace rl
}  // namespace ard

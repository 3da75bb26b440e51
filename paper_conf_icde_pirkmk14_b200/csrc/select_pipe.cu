// select_pipe.cu -- step a3, the ordered approximate select (ar_approx_select,
// PAPER.md:606-632, s IV-B), as a persistent TMA-pipelined scan.
//
// Persistent CTAs (one producer warp + NW consumer warps) stream 8192-row
// tiles of every predicate's SLICED majors into a ring of shared-memory stages
// (produce_ring).  Per tile each consumer thread decides one 32-row block
// (eval_block: candidate and definite masks by borrow chains on the bit planes),
// then:
//   1. the warp's candidate rows go to a per-warp list in shared memory
//      (ascending: warp w owns rows [1024 w, 1024 w + 1024) of the tile), a
//      named barrier gives every warp its offset inside the tile;
//   2. the lanes take list entries in parallel -- definite flag and the
//      approximation tuple (the candidate relation's (ID, Approx) pairs of
//      Fig. 4) read from the stage -- and write (pos, aux)
//      with coalesced stores to the tile's slice of the workspace;
//   3. the tile's count goes to tile_count[t] and, with one atomic, to the total
//      of its group of 2^kGroupShift tiles.
// compact_kernel (select.cu) then moves every slice to its final offset, so no
// CTA ever waits for another (DESIGN s6.2).
#include "rl_common.cuh"

namespace ard {
namespace rl {

template <int NW, int... WK>
__global__ void __launch_bounds__((NW + 1) * 32, 2) select_pipe_kernel(const __grid_constant__ SelParams P) {
    using S = Shape<WK...>;
    constexpr int NT = NW * 32;
    constexpr int kWarpRows = 32 * 32;
    extern __shared__ __align__(128) unsigned char smem[];
    __shared__ uint32_t wtot[2][NW];   // per-warp candidate counts, double-buffered by tile parity
    uint64_t* full = reinterpret_cast<uint64_t*>(smem);
    uint64_t* empty = full + P.nstages;
    long long* slot = reinterpret_cast<long long*>(empty + P.nstages);
    const size_t head_bytes = ((size_t)P.nstages * 24 + 127) & ~size_t(127);
    uint32_t* stages = reinterpret_cast<uint32_t*>(smem + head_bytes);
    const unsigned warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    uint16_t* list = reinterpret_cast<uint16_t*>(stages + (size_t)P.nstages * P.stage_words) + warp * kWarpRows;
    if (threadIdx.x == 0) {
        for (uint32_t s = 0; s < P.nstages; ++s) {
            mbar_init(full + s, 1);
            mbar_init(empty + s, NW);
        }
        fence_mbar_init();
    }
    __syncthreads();
    if (warp == NW) {
        if (lane == 0) produce_ring(P, full, empty, slot, stages);
        return;
    }

    uint32_t s = 0, ph = 0, par = 0;
    for (;; s = (s + 1 == P.nstages) ? (ph ^= 1u, 0u) : s + 1, par ^= 1u) {
        mbar_wait(full + s, ph, P.suspend_ns);
        const long long t = slot[s];
        if (t < 0) break;
        const uint32_t* stg = stages + (size_t)s * P.stage_words;
        const int64_t tile_r0 = t * (int64_t)P.tile_rows;
        const uint32_t blk = threadIdx.x;   // rows [32 blk, 32 blk + 32) of the tile
        const uint32_t vm = tile_r0 + (int64_t)P.tile_rows <= P.n ? 0xffffffffu
                                                                   : valid_mask(tile_r0 + 32 * (int64_t)blk, P.n);
        uint32_t cm, dm, em;
        eval_block<S, false>(P, stg, blk, vm, cm, dm, em);
        const uint32_t cnt = __popc(cm);
        uint32_t incl = cnt;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            const uint32_t y = __shfl_up_sync(0xffffffffu, incl, o);
            if (lane >= (unsigned)o) incl += y;
        }
        const uint32_t wtotal = __shfl_sync(0xffffffffu, incl, 31);
        if (lane == 0) wtot[par][warp] = wtotal;
        // this thread's candidates -> the warp list: 10-bit row in the warp slice | definite << 15
        uint32_t e = incl - cnt;
        for (uint32_t m = cm; m; m &= m - 1) {
            const uint32_t l = __ffs(m) - 1;
            list[e++] = (uint16_t)((lane << 5) | l | (((dm >> l) & 1u) << 15));
        }
        bar_sync(1, NT);   // every warp's count is in wtot[par]
        uint32_t before = 0, total = 0;
#pragma unroll
        for (int w = 0; w < NW; ++w) {
            const uint32_t x = wtot[par][w];
            before += (w < (int)warp) ? x : 0u;
            total += x;
        }
        if (threadIdx.x == 0) {
            P.tile_count[t] = total;
            if (total) atomicAdd(P.group_sum + (t >> kGroupShift), (unsigned long long)total);
        }
        // lanes in parallel: (pos, aux) of the warp's candidates, coalesced into the tile's slice
        uint32_t* dpos = P.tmp_pos + (size_t)t * P.tile_rows + before;
        uint32_t* daux = P.tmp_aux + (size_t)t * P.tile_rows + before;
        const uint32_t wrow0 = (uint32_t)tile_r0 + warp * kWarpRows;
        for (uint32_t j = lane; j < wtotal; j += 32) {
            const uint32_t v = list[j];
            const uint32_t r = v & 0x3ffu;
            uint32_t aux = (v & 0x8000u) << 16;   // AR_AUX_DEFINITE
            if (P.carry) {
                const uint32_t b = warp * 32 + (r >> 5), l = r & 31u;
                static_for<S::N>([&](auto cc) {
                    constexpr int C = decltype(cc)::value;
                    constexpr int W = S::w(C), O = S::off(C);
                    uint32_t x[W];
                    lds_words<W>(x, stg + P.p[C].soff + b * W);
                    aux |= row_of<W>(x, l) << O;
                });
            }
            dpos[j] = wrow0 + r;
            daux[j] = aux;
        }
        __syncwarp();
        if (lane == 0) mbar_arrive(empty + s);
    }
}

}  // namespace rl
}  // namespace ard

// ------------------------------------------------------------------------ host

namespace ar {

namespace {

// Shape code per predicate: (w_major << 6) | 1 if decomposed (k > 0: definite
// range differs from the candidate range), else w_major << 6.
constexpr int WD(int w, int d) { return (w << 6) | d; }

template <int... Ws>
bool sp_match(const ard::SelParams& P) {
    constexpr int n = sizeof...(Ws);
    constexpr int wd[] = {Ws..., 0};
    if (P.npred != n) return false;
    for (int c = 0; c < n; ++c)
        if ((int)((P.p[c].w << 6) | (P.p[c].k > 0 ? 1u : 0u)) != wd[c]) return false;
    return true;
}

constexpr int kSpNW = 8;

// Q6; single columns at 8 / 16 / 24 major bits (C1, C3) decomposed or whole; 32-bit
// whole columns; the two-column 24/8 spatial query.
const void* sp_find(const ard::SelParams& P) {
#define AR_SP_TRY(...) \
    if (sp_match<__VA_ARGS__>(P)) return (const void*)ard::rl::select_pipe_kernel<kSpNW, __VA_ARGS__>;
    AR_SP_TRY(WD(4, 1), WD(4, 0), WD(6, 0))
    AR_SP_TRY(WD(8, 1))
    AR_SP_TRY(WD(16, 1))
    AR_SP_TRY(WD(24, 1))
    AR_SP_TRY(WD(8, 0))
    AR_SP_TRY(WD(16, 0))
    AR_SP_TRY(WD(24, 0))
    AR_SP_TRY(WD(32, 0))
    AR_SP_TRY(WD(24, 1), WD(24, 1))
#undef AR_SP_TRY
    return nullptr;
}

}  // namespace

// Launch the pipelined select scan if the shape has a kernel (8192-row tiles,
// like select_tile_kernel, so the workspace layout is shared); *launched = false
// otherwise.
ar_status launch_select_pipe(const ard::SelParams& P0, bool* launched, cudaStream_t s) {
    *launched = false;
    static const bool off = getenv("AR_SELECT_LEGACY") && atoi(getenv("AR_SELECT_LEGACY"));
    if (off || P0.tile_rows != (uint32_t)kSpNW * 1024u) return AR_OK;
    const void* fn = sp_find(P0);
    if (!fn) return AR_OK;
    ard::SelParams P = P0;
    static thread_local const void* opted[32];
    static thread_local int nopted = 0;
    bool seen = false;
    for (int i = 0; i < nopted; ++i) seen |= opted[i] == fn;
    if (!seen) {
        int dev = 0, max_optin = 227 * 1024;
        if (cudaGetDevice(&dev) == cudaSuccess)
            cudaDeviceGetAttribute(&max_optin, cudaDevAttrMaxSharedMemoryPerBlockOptin, dev);
        cudaFuncAttributes fa{};
        if (cudaFuncGetAttributes(&fa, fn) == cudaSuccess) max_optin -= (int)fa.sharedSizeBytes;
        cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, max_optin);
        cudaGetLastError();
        if (nopted < 32) opted[nopted++] = fn;
    }
    const int threads = (kSpNW + 1) * 32;
    auto smem_of = [&](uint32_t st) {
        return (((size_t)st * 24 + 127) & ~size_t(127)) + (size_t)st * P.stage_words * 4 + (size_t)kSpNW * 1024 * 2;
    };
    // deepest ring (<= 8, >= 3 stages) with 2 CTAs per SM, else 1 CTA with >= 2 stages
    uint32_t stages = 0;
    int occ = 0;
    for (int target = 2; target >= 1 && !stages; --target)
        for (uint32_t st = 8; st >= 2; --st) {
            if (target == 2 && st < 3) break;
            int o = 0;
            cudaOccupancyMaxActiveBlocksPerMultiprocessor(&o, fn, threads, smem_of(st));
            if (o >= target) {
                stages = st;
                occ = target;
                break;
            }
        }
    cudaGetLastError();
    if (!stages) return AR_OK;
    P.nstages = stages;
    const int grid = (int)std::min<int64_t>(P.num_tiles, (int64_t)num_sms() * occ);
    void* args[] = {&P};
    AR_TRY_CUDA(cudaLaunchKernel(fn, dim3(grid), dim3(threads), args, smem_of(stages), s));
    *launched = true;
    return AR_OK;
}

}  // namespace ar

// decompose.cu -- step a1: BWD decomposition + bit packing (PAPER.md:143-160
// s II-A, Fig. 2; bwdecompose(A, bits) PAPER.md:854-861 s V-A).  One-time,
// outside the timed region.
//   u = v - base, major = u >> k, residual = u & (2^k - 1)
// SLICED majors are built with one warp per 32-row block: W warp ballots give
// the W bit planes.  PACKED streams are built one output word per thread.
#include "kernels.cuh"

namespace ard {

// out[0] = max(d), out[1] = min(d) over the keys d = v ^ flip
__global__ void minmax_kernel(const uint32_t* __restrict__ col, int64_t n, uint32_t flip, uint32_t* out) {
    uint32_t hi = 0, lo = 0xffffffffu;
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += (int64_t)gridDim.x * blockDim.x) {
        const uint32_t d = col[i] ^ flip;
        hi = max(hi, d);
        lo = min(lo, d);
    }
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) {
        hi = max(hi, __shfl_xor_sync(0xffffffffu, hi, o));
        lo = min(lo, __shfl_xor_sync(0xffffffffu, lo, o));
    }
    if ((threadIdx.x & 31) == 0) {
        atomicMax(out, hi);
        atomicMin(out + 1, lo);
    }
}

// One warp per 32-row block; blocks beyond n (up to the 128-row padding) are zero.
// Field of row i: (((col[i] ^ flip) - base) >> shift) & mask (major: shift k; residual: mask 2^k - 1).
__global__ void pack_sliced_kernel(const uint32_t* __restrict__ col, int64_t n, int shift, uint32_t mask,
                                   uint32_t flip, uint32_t base, int w, int64_t nblocks, uint32_t* __restrict__ out) {
    const unsigned lane = threadIdx.x & 31;
    const int64_t warps = (int64_t)gridDim.x * (blockDim.x / 32);
    for (int64_t b = (int64_t)blockIdx.x * (blockDim.x / 32) + (threadIdx.x >> 5); b < nblocks; b += warps) {
        const int64_t row = b * 32 + lane;
        const uint32_t m = row < n ? ((((col[row] ^ flip) - base) >> shift) & mask) : 0u;
        uint32_t mine = 0;
        for (int j = 0; j < w; ++j) {
            const uint32_t plane = __ballot_sync(0xffffffffu, (m >> j) & 1u);
            if ((int)lane == j) mine = plane;
        }
        if ((int)lane < w) out[b * w + lane] = mine;
    }
}

// Output word i holds bits [32 i, 32 i + 32) of the LSB-first stream of the
// w-bit fields x_j = (((col[j] ^ flip) - base) >> shift) & mask.
__global__ void pack_packed_kernel(const uint32_t* __restrict__ col, int64_t n, int shift, uint32_t mask,
                                   uint32_t flip, uint32_t base, int w, uint64_t out_words,
                                   uint32_t* __restrict__ out) {
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < out_words;
         i += (uint64_t)gridDim.x * blockDim.x) {
        const uint64_t b0 = i * 32, b1 = b0 + 32;
        uint64_t j = b0 / (uint64_t)w;
        const uint64_t jend = (b1 + w - 1) / (uint64_t)w;
        uint32_t word = 0;
        for (; j < jend && j < (uint64_t)n; ++j) {
            const uint64_t x = (uint64_t)((((col[j] ^ flip) - base) >> shift) & mask);
            const int64_t off = (int64_t)(j * (uint64_t)w) - (int64_t)b0;   // bit offset of field j in word i
            if (off >= 0)
                word |= (uint32_t)(x << off);
            else
                word |= (uint32_t)(x >> (-off));
        }
        out[i] = word;
    }
}

// Split SLICED residual (k <= 8 planes, h high planes apart): one warp per
// 32-row block b; plane j (bit j of the residual) goes to its super-group's
// high-plane area (j >= k - h) or low-plane area.
__global__ void pack_split_kernel(const uint32_t* __restrict__ col, int64_t n, int k, int h, uint32_t flip,
                                  uint32_t base, int64_t nblocks, uint32_t* __restrict__ out) {
    const unsigned lane = threadIdx.x & 31;
    const int64_t warps = (int64_t)gridDim.x * (blockDim.x / 32);
    for (int64_t b = (int64_t)blockIdx.x * (blockDim.x / 32) + (threadIdx.x >> 5); b < nblocks; b += warps) {
        const int64_t row = b * 32 + lane;
        const uint32_t r = row < n ? (((col[row] ^ flip) - base) & ((1u << k) - 1u)) : 0u;
        uint32_t mine = 0;
        for (int j = 0; j < k; ++j) {
            const uint32_t plane = __ballot_sync(0xffffffffu, (r >> j) & 1u);
            if ((int)lane == j) mine = plane;
        }
        if ((int)lane < k) out[split_word((uint64_t)b, k, h, (int)lane)] = mine;
    }
}

}  // namespace ard

namespace ar {

ar_status launch_pack_split(const uint32_t* col, int64_t n, int k, int h, uint32_t flip, uint32_t base, uint32_t* out,
                            cudaStream_t s) {
    const int64_t nblocks = (int64_t)ceil_div_u64((uint64_t)n, 32ull * kSplitBlocks) * kSplitBlocks;   // whole super-groups (padding zeroed)
    if (nblocks == 0) return AR_OK;
    int grid = (int)std::min<int64_t>((nblocks + 7) / 8, (int64_t)num_sms() * 16);
    ard::pack_split_kernel<<<grid, 256, 0, s>>>(col, n, k, h, flip, base, nblocks, out);
    AR_CHECK_LAUNCH("pack_split_kernel");
    return AR_OK;
}

ar_status launch_decompose_minmax(const uint32_t* col, int64_t n, uint32_t flip, uint32_t* out2, cudaStream_t s) {
    int grid = (int)std::min<int64_t>((n + 255) / 256, (int64_t)num_sms() * 8);
    if (grid < 1) grid = 1;
    ard::minmax_kernel<<<grid, 256, 0, s>>>(col, n, flip, out2);
    AR_CHECK_LAUNCH("minmax_kernel");
    return AR_OK;
}

ar_status launch_pack_sliced(const uint32_t* col, int64_t n, int shift, uint32_t mask, uint32_t flip, uint32_t base,
                             int w, uint32_t* out, cudaStream_t s) {
    const int64_t nblocks = (int64_t)ceil_div_u64((uint64_t)n, 128) * 4;
    if (w == 0 || nblocks == 0) return AR_OK;
    int grid = (int)std::min<int64_t>((nblocks + 7) / 8, (int64_t)num_sms() * 16);
    ard::pack_sliced_kernel<<<grid, 256, 0, s>>>(col, n, shift, mask, flip, base, w, nblocks, out);
    AR_CHECK_LAUNCH("pack_sliced_kernel");
    return AR_OK;
}

ar_status launch_pack_packed(const uint32_t* col, int64_t n, int shift, uint32_t mask, uint32_t flip, uint32_t base,
                             int w, uint64_t out_words, uint32_t* out, cudaStream_t s) {
    if (w == 0 || out_words == 0) return AR_OK;
    int grid = (int)std::min<uint64_t>((out_words + 255) / 256, (uint64_t)num_sms() * 16);
    ard::pack_packed_kernel<<<grid, 256, 0, s>>>(col, n, shift, mask, flip, base, w, out_words, out);
    AR_CHECK_LAUNCH("pack_packed_kernel");
    return AR_OK;
}

}  // namespace ar

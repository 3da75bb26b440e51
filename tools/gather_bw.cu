// gather_bw.cu -- micro-benchmark (tools only): throughput of sparse 4-byte
// gathers with the .L2::64B prefetch hint on B200, the access pattern of the
// refine / SUM steps (ld_gather_if in common.cuh).  Positions are either
// uniformly random over the buffer or ascending at a given density (the
// candidate relation is sorted, and each thread takes 8 consecutive entries).
// Reports gathers/s and the 64-B granule bandwidth (gathers x 64 B / time) --
// the ceiling a gather-bound kernel can reach, next to the streaming peak.
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o /tmp/gbw tools/gather_bw.cu && /tmp/gbw
#include <cstdint>
#include <cstdio>
#include <cuda_runtime.h>

__device__ __forceinline__ uint32_t ld64(const uint32_t* p) {
    uint32_t v;
    asm volatile("ld.global.nc.L2::64B.u32 %0, [%1];" : "=r"(v) : "l"(p));
    return v;
}

// 8 gathers per thread, all issued before any is used
__global__ void gather8(const uint32_t* __restrict__ buf, const uint32_t* __restrict__ idx, uint64_t m,
                        unsigned long long* out) {
    const uint64_t t = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    uint32_t acc = 0;
    for (uint64_t j0 = t * 8; j0 < m; j0 += stride * 8) {
        uint32_t p[8], v[8];
#pragma unroll
        for (int i = 0; i < 8; ++i) p[i] = idx[j0 + i];
#pragma unroll
        for (int i = 0; i < 8; ++i) v[i] = ld64(buf + p[i]);
#pragma unroll
        for (int i = 0; i < 8; ++i) acc += v[i];
    }
    if (acc == 0x12345678u) atomicAdd(out, 1ull);
}

// splitmix-style hash for reproducible positions
__host__ __device__ inline uint64_t mix(uint64_t x) {
    x += 0x9e3779b97f4a7c15ull;
    x = (x ^ (x >> 30)) * 0xbf58476d1ce4e5b9ull;
    x = (x ^ (x >> 27)) * 0x94d049bb133111ebull;
    return x ^ (x >> 31);
}

__global__ void make_random(uint32_t* idx, uint64_t m, uint64_t words) {
    const uint64_t t = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x;
    for (uint64_t j = t; j < m; j += (uint64_t)gridDim.x * blockDim.x) idx[j] = (uint32_t)(mix(j) % words);
}
// ascending positions at density ~1/gap words: word j * gap + jitter
__global__ void make_sorted(uint32_t* idx, uint64_t m, uint32_t gap) {
    const uint64_t t = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x;
    for (uint64_t j = t; j < m; j += (uint64_t)gridDim.x * blockDim.x)
        idx[j] = (uint32_t)(j * gap + mix(j) % gap);
}

int main() {
    const uint64_t words = 1ull << 30;   // 4 GB gather target
    const uint64_t m = 32ull << 20;      // 32 M gathers
    uint32_t *buf, *idx;
    unsigned long long* out;
    cudaMalloc(&buf, words * 4);
    cudaMalloc(&idx, m * 4);
    cudaMalloc(&out, 8);
    cudaMemset(buf, 1, words * 4);
    int sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
    cudaEvent_t a, b;
    cudaEventCreate(&a);
    cudaEventCreate(&b);
    // gap in words between consecutive positions: 1 / density of 4-B rows; 24-bit rows (l_extendedprice,
    // 3 B) at 1.9 % are one every ~52 rows = ~39 words; random = uniform over the buffer
    const int gaps[] = {0, 4, 16, 39, 128};
    for (int gi = 0; gi < 5; ++gi) {
        const int gap = gaps[gi];
        // sorted positions must stay inside the buffer: at most words / gap of them
        const uint64_t m_g = gap ? ((words / gap) & ~uint64_t(7)) < m ? ((words / gap) & ~uint64_t(7)) : m : m;
        if (gap == 0)
            make_random<<<sms * 8, 256>>>(idx, m_g, words);
        else
            make_sorted<<<sms * 8, 256>>>(idx, m_g, (uint32_t)gap);
        for (int ctas = 2; ctas <= 16; ctas *= 2) {
            const int grid = sms * ctas;
            gather8<<<grid, 256>>>(buf, idx, m_g, out);
            cudaEventRecord(a);
            for (int r = 0; r < 5; ++r) gather8<<<grid, 256>>>(buf, idx, m_g, out);
            cudaEventRecord(b);
            cudaEventSynchronize(b);
            float ms = 0;
            cudaEventElapsedTime(&ms, a, b);
            ms /= 5;
            const double gps = m_g / (ms * 1e-3);
            printf("{\"pattern\": \"%s\", \"gap_words\": %d, \"ctas_per_sm\": %d, \"ms\": %.4f, \"gathers_per_s\": %.4g, "
                   "\"granule64_gbs\": %.1f, \"index_gbs\": %.1f}\n",
                   gap ? "sorted" : "random", gap, ctas, ms, gps, gps * 64 / 1e9, gps * 4 / 1e9);
        }
    }
    printf("{\"done\": \"%s\"}\n", cudaGetErrorString(cudaGetLastError()));
    return 0;
}

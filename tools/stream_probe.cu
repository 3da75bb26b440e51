// stream_probe.cu -- read-bandwidth ceilings on this GPU for the access patterns
// of the scan kernels (tools only; not part of the library).
//
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o tools/stream_probe tools/stream_probe.cu
//   tools/stream_probe [MB]
//
// 1. ldg:  grid-stride 16-B loads (ld.global.nc.v4), XOR-reduced, CTAs = k * SMs.
// 2. tma:  persistent CTAs, one producer lane streaming CHUNK-byte 1-D bulk
//          copies (cp.async.bulk) into a ring of NST stages, consumers release
//          each stage at once (the scan kernels' pipeline without compute).
// Buffers rotate over 3 copies (> L2); each point is the best of 3 batches of
// 20 back-to-back launches, timed with CUDA events.
#include <cstdio>
#include <cstdlib>
#include <cstdint>
#include <cuda_runtime.h>

#define CK(x) do { cudaError_t e = (x); if (e != cudaSuccess) { printf("%s: %s\n", #x, cudaGetErrorString(e)); exit(1); } } while (0)

__global__ void ldg_kernel(const uint4* __restrict__ p, size_t n16, unsigned* out) {
    uint32_t acc = 0;
    for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < n16; i += (size_t)gridDim.x * blockDim.x) {
        uint4 v;
        asm volatile("ld.global.nc.v4.u32 {%0,%1,%2,%3}, [%4];" : "=r"(v.x), "=r"(v.y), "=r"(v.z), "=r"(v.w) : "l"(p + i));
        acc ^= v.x ^ v.y ^ v.z ^ v.w;
    }
    if (acc == 0x12345678u) *out = acc;
}

__device__ __forceinline__ uint32_t smem_u32(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }

__global__ void tma_kernel(const char* __restrict__ src, size_t bytes, uint32_t chunk, uint32_t nst, unsigned* out) {
    extern __shared__ __align__(128) unsigned char smem[];
    uint64_t* full = (uint64_t*)smem;
    uint64_t* empty = full + nst;
    unsigned char* stages = smem + 1024;
    const unsigned warp = threadIdx.x >> 5, lane = threadIdx.x & 31, nw = blockDim.x / 32 - 1;
    if (threadIdx.x == 0) {
        for (uint32_t s = 0; s < nst; ++s) {
            asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(full + s)), "r"(1));
            asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(empty + s)), "r"(nw));
        }
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    __syncthreads();
    const size_t nchunks = (bytes + chunk - 1) / chunk;
    if (warp == nw) {
        if (lane) return;
        uint32_t s = 0, ph = 0;
        for (size_t c = blockIdx.x, i = 0; c < nchunks; c += gridDim.x, ++i) {
            if (i >= nst)
                asm volatile("{\n.reg .pred p;\nW%=:\nmbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n@!p bra W%=;\n}" ::"r"(smem_u32(empty + s)), "r"(ph ^ 1u) : "memory");
            const uint32_t b = (uint32_t)min((size_t)chunk, bytes - c * chunk);
            asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(full + s)), "r"(b) : "memory");
            asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(smem_u32(stages + (size_t)s * chunk)), "l"(src + c * chunk), "r"(b), "r"(smem_u32(full + s)) : "memory");
            if (++s == nst) { s = 0; ph ^= 1u; }
        }
        return;
    }
    uint32_t s = 0, ph = 0, acc = 0;
    for (size_t c = blockIdx.x; c < nchunks; c += gridDim.x) {
        asm volatile("{\n.reg .pred p;\nW%=:\nmbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n@!p bra W%=;\n}" ::"r"(smem_u32(full + s)), "r"(ph) : "memory");
        acc ^= ((const uint32_t*)(stages + (size_t)s * chunk))[threadIdx.x];
        __syncwarp();
        if (lane == 0) asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(smem_u32(empty + s)) : "memory");
        if (++s == nst) { s = 0; ph ^= 1u; }
    }
    if (acc == 0x12345678u) *out = acc;
}

// 3. gather: `per` independent 4-B loads per thread (ld.global.nc.L2::64B) at
//    random 64-B-aligned offsets of the buffer -- the one-pass kernel's
//    l_extendedprice gathers; reported as 64-B granules per second.
__global__ void gather_kernel(const uint32_t* __restrict__ p, size_t words, uint32_t n, uint32_t seed, unsigned* out) {
    uint32_t acc = 0;
    const size_t granules = words / 16;
    for (uint32_t i = blockIdx.x * blockDim.x + threadIdx.x; i < n; i += gridDim.x * blockDim.x) {
        uint32_t v[8];
#pragma unroll
        for (int j = 0; j < 8; ++j) {
            uint64_t h = (uint64_t)(i * 8 + j) * 0x9E3779B97F4A7C15ull + seed;
            h ^= h >> 29;
            const size_t g = (size_t)(h % granules);
            asm volatile("ld.global.nc.L2::64B.u32 %0, [%1];" : "=r"(v[j]) : "l"(p + g * 16));
        }
#pragma unroll
        for (int j = 0; j < 8; ++j) acc ^= v[j];
    }
    if (acc == 0x12345678u) *out = acc;
}

int main(int argc, char** argv) {
    const size_t mb = argc > 1 ? atoi(argv[1]) : 165;
    const size_t bytes = mb << 20;
    int sms = 0;
    CK(cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0));
    char* buf[3];
    for (auto& b : buf) { CK(cudaMalloc(&b, bytes)); CK(cudaMemset(b, 1, bytes)); }
    unsigned* out;
    CK(cudaMalloc(&out, 4));
    cudaEvent_t a, z;
    CK(cudaEventCreate(&a)); CK(cudaEventCreate(&z));
    auto timeit = [&](auto launch) {
        float best = 1e30f;
        for (int it = 0; it < 4; ++it) {
            CK(cudaEventRecord(a));
            for (int r = 0; r < 20; ++r) launch(buf[r % 3]);
            CK(cudaEventRecord(z));
            CK(cudaEventSynchronize(z));
            float ms;
            CK(cudaEventElapsedTime(&ms, a, z));
            if (it) best = std::min(best, ms / 20);
        }
        CK(cudaGetLastError());
        return best;
    };
    for (int k : {2, 4, 8, 16}) {
        float ms = timeit([&](char* b) { ldg_kernel<<<sms * k, 256>>>((const uint4*)b, bytes / 16, out); });
        printf("{\"probe\": \"ldg\", \"MB\": %zu, \"ctas_per_sm\": %d, \"us\": %.2f, \"gbs\": %.0f}\n", mb, k, ms * 1e3, bytes / ms / 1e6);
    }
    for (uint32_t chunk : {4096u, 8192u, 16384u, 32768u})
        for (uint32_t nst : {2u, 4u, 6u})
            for (int ctas : {1, 2}) {
                const size_t smem = 1024 + (size_t)nst * chunk;
                if (smem * ctas > 220 * 1024) continue;
                CK(cudaFuncSetAttribute(tma_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem));
                float ms = timeit([&](char* b) { tma_kernel<<<sms * ctas, 9 * 32, smem>>>(b, bytes, chunk, nst, out); });
                printf("{\"probe\": \"tma\", \"MB\": %zu, \"chunk\": %u, \"stages\": %u, \"ctas_per_sm\": %d, \"us\": %.2f, \"gbs\": %.0f}\n",
                       mb, chunk, nst, ctas, ms * 1e3, bytes / ms / 1e6);
            }
    for (uint32_t ng : {1u << 20, 1u << 22}) {   // x 8 loads per index
        for (int k : {4, 8, 16}) {
            int it = 0;
            float ms = timeit([&](char* b) { gather_kernel<<<sms * k, 256>>>((const uint32_t*)b, bytes / 4, ng, ++it, out); });
            const double g = 8.0 * ng;
            printf("{\"probe\": \"gather64\", \"MB\": %zu, \"gathers\": %.0f, \"ctas_per_sm\": %d, \"us\": %.2f, "
                   "\"granules_per_s\": %.3e, \"gbs_64B\": %.0f}\n", mb, g, k, ms * 1e3, g / ms * 1e3, g * 64 / ms / 1e6);
        }
    }
    return 0;
}

// gather_probe.cu -- micro-benchmark (tools only): DRAM bytes moved per random
// 4-byte gather on B200 for several load flavours, to size the sector-granular
// gather roofline of the refine step.  Build + run under ncu:
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o /tmp/gp tools/gather_probe.cu
//   ncu --metrics dram__bytes_read.sum,gpu__time_duration.sum /tmp/gp
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

__device__ __forceinline__ uint32_t ld_default(const uint32_t* p) { return *p; }
__device__ __forceinline__ uint32_t ld_nc(const uint32_t* p) { return __ldg(p); }
__device__ __forceinline__ uint32_t ld_cs(const uint32_t* p) { return __ldcs(p); }
__device__ __forceinline__ uint32_t ld_na(const uint32_t* p) {
    uint32_t v;
    asm volatile("ld.global.L1::no_allocate.u32 %0, [%1];" : "=r"(v) : "l"(p));
    return v;
}
__device__ __forceinline__ uint32_t ld_64b(const uint32_t* p) {
    uint32_t v;
    asm volatile("ld.global.L2::64B.u32 %0, [%1];" : "=r"(v) : "l"(p));
    return v;
}

__device__ __forceinline__ uint32_t ld_cv(const uint32_t* p) {
    uint32_t v;
    asm volatile("ld.global.cv.u32 %0, [%1];" : "=r"(v) : "l"(p));
    return v;
}
__device__ __forceinline__ uint32_t ld_relaxed(const uint32_t* p) {
    uint32_t v;
    asm volatile("ld.relaxed.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p));
    return v;
}
__device__ __forceinline__ uint32_t ld_lu(const uint32_t* p) {
    uint32_t v;
    asm volatile("ld.global.lu.u32 %0, [%1];" : "=r"(v) : "l"(p));
    return v;
}
__device__ __forceinline__ uint32_t ld_cg(const uint32_t* p) {
    uint32_t v;
    asm volatile("ld.global.cg.u32 %0, [%1];" : "=r"(v) : "l"(p));
    return v;
}
__device__ __forceinline__ uint32_t ld_mmio(const uint32_t* p) {
    uint32_t v;
    asm volatile("ld.volatile.global.u32 %0, [%1];" : "=r"(v) : "l"(p));
    return v;
}

template <int MODE>
__global__ void gather(const uint32_t* __restrict__ buf, uint64_t nwords, uint64_t n, uint64_t seed,
                       unsigned long long* out) {
    uint64_t acc = 0;
    for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n; i += (uint64_t)gridDim.x * blockDim.x) {
        uint64_t z = (i + seed) * 0x9E3779B97F4A7C15ull;
        z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
        z ^= z >> 31;
        const uint32_t* p = buf + (z % nwords);
        uint32_t v;
        if (MODE == 0) v = ld_default(p);
        else if (MODE == 1) v = ld_nc(p);
        else if (MODE == 2) v = ld_cs(p);
        else if (MODE == 3) v = ld_na(p);
        else if (MODE == 4) v = ld_64b(p);
        else if (MODE == 5) v = ld_cv(p);
        else if (MODE == 6) v = ld_relaxed(p);
        else if (MODE == 7) v = ld_lu(p);
        else if (MODE == 8) v = ld_cg(p);
        else v = ld_mmio(p);
        acc += v;
    }
    if (acc == 0x123456789ull) atomicAdd(out, acc);
}

// cp.async (LDGSTS) 16-B gathers into shared memory
__global__ void gather_ldgsts(const uint32_t* __restrict__ buf, uint64_t nwords, uint64_t n, uint64_t seed,
                              unsigned long long* out) {
    __shared__ __align__(16) uint32_t sm[256 * 4];
    uint64_t acc = 0;
    for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n; i += (uint64_t)gridDim.x * blockDim.x) {
        uint64_t z = (i + seed) * 0x9E3779B97F4A7C15ull;
        z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
        z ^= z >> 31;
        const uint32_t* p = buf + ((z % nwords) & ~3ull);
        uint32_t dst = (uint32_t)__cvta_generic_to_shared(sm + threadIdx.x * 4);
        asm volatile("cp.async.cg.shared.global [%0], [%1], 16;" ::"r"(dst), "l"(p) : "memory");
        asm volatile("cp.async.wait_all;" ::: "memory");
        acc += sm[threadIdx.x * 4];
    }
    if (acc == 0x123456789ull) atomicAdd(out, acc);
}

// TMA bulk 16-B gathers into shared memory (one mbarrier per thread)
__global__ void gather_bulk(const uint32_t* __restrict__ buf, uint64_t nwords, uint64_t n, uint64_t seed,
                            unsigned long long* out) {
    __shared__ __align__(16) uint32_t sm[256 * 4];
    __shared__ __align__(8) uint64_t bar[256];
    uint32_t b = (uint32_t)__cvta_generic_to_shared(bar + threadIdx.x);
    asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(b));
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    uint64_t acc = 0;
    uint32_t phase = 0;
    for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n; i += (uint64_t)gridDim.x * blockDim.x) {
        uint64_t z = (i + seed) * 0x9E3779B97F4A7C15ull;
        z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
        z ^= z >> 31;
        const uint32_t* p = buf + ((z % nwords) & ~3ull);
        uint32_t dst = (uint32_t)__cvta_generic_to_shared(sm + threadIdx.x * 4);
        asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], 16;" ::"r"(b) : "memory");
        asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], 16, [%2];" ::"r"(dst),
                     "l"(p), "r"(b)
                     : "memory");
        asm volatile(
            "{\n\t.reg .pred q;\nW_%=:\n\tmbarrier.try_wait.parity.shared::cta.b64 q, [%0], %1;\n\t@!q bra W_%=;\n}" ::"r"(b),
            "r"(phase)
            : "memory");
        phase ^= 1;
        acc += sm[threadIdx.x * 4];
    }
    if (acc == 0x123456789ull) atomicAdd(out, acc);
}

int main() {
    const uint64_t nwords = (1ull << 30) / 4 * 2;   // 2 GB
    const uint64_t n = 1 << 22;                      // 4 M gathers (~0.2 % of the 32-B sectors)
    uint32_t* buf;
    unsigned long long* out;
    cudaMalloc(&buf, nwords * 4);
    cudaMalloc(&out, 8);
    cudaMemset(buf, 1, nwords * 4);
    void* flush;
    cudaMalloc(&flush, 512ull << 20);
    for (int limit : {0}) {
        if (limit) {
            cudaError_t e = cudaDeviceSetLimit(cudaLimitMaxL2FetchGranularity, limit);
            size_t got = 0;
            cudaDeviceGetLimit(&got, cudaLimitMaxL2FetchGranularity);
            printf("set L2 fetch granularity %d -> %s, now %zu\n", limit, cudaGetErrorString(e), got);
        }
        for (int mode = 0; mode < 10; ++mode) {
            cudaMemset(flush, mode, 512ull << 20);
            switch (mode) {
                case 0: gather<0><<<1184, 256>>>(buf, nwords, n, 1, out); break;
                case 1: gather<1><<<1184, 256>>>(buf, nwords, n, 2, out); break;
                case 2: gather<2><<<1184, 256>>>(buf, nwords, n, 3, out); break;
                case 3: gather<3><<<1184, 256>>>(buf, nwords, n, 4, out); break;
                case 4: gather<4><<<1184, 256>>>(buf, nwords, n, 5, out); break;
                case 5: gather<5><<<1184, 256>>>(buf, nwords, n, 6, out); break;
                case 6: gather<6><<<1184, 256>>>(buf, nwords, n, 7, out); break;
                case 7: gather<7><<<1184, 256>>>(buf, nwords, n, 8, out); break;
                case 8: gather<8><<<1184, 256>>>(buf, nwords, n, 9, out); break;
                case 9: gather<9><<<1184, 256>>>(buf, nwords, n, 10, out); break;
            }
        }
        for (int mode = 0; mode < 2; ++mode) {
            cudaMemset(flush, mode, 512ull << 20);
            if (mode == 0) gather_ldgsts<<<1184, 256>>>(buf, nwords, n, 11, out);
            else gather_bulk<<<1184, 256>>>(buf, nwords, n, 12, out);
        }
    }
    cudaDeviceSynchronize();
    printf("done %s\n", cudaGetErrorString(cudaGetLastError()));
    return 0;
}

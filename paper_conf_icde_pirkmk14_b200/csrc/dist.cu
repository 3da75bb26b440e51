// dist.cu -- step a4: row-sharded multi-GPU exchange over NCCL (NVLink 5 /
// NVSwitch).  The paper never splits one query across GPUs;
// the build shards rows (BASELINE north_star): each rank scans its own row
// range, then exchanges 8-byte counts (ncclAllGather -> global offsets) and
// reduces the int64 SUM (ncclAllReduce).  Messages are tiny: latency-bound.
// The shard geometry, the exclusive prefix and the placement of a rank's
// slice in the concatenated result are separate calls, so the exchange can be
// checked for every rank of any world size on one GPU (tests/test_gpu_dist.py).
#include <nccl.h>

#include "kernels.cuh"

namespace ard {

// Exclusive prefix of the gathered per-rank counts: the rank's offset in the
// concatenated, globally ordered result, and the total.  world <= a few
// hundred: one warp, each lane sums a strided subset.
__global__ void exclusive_offset_kernel(const long long* all, int world, int rank, long long* off,
                                        long long* total) {
    const unsigned lane = threadIdx.x;
    long long before = 0, all_sum = 0;
    for (int r = (int)lane; r < world; r += 32) {
        const long long c = all[r];
        all_sum += c;
        if (r < rank) before += c;
    }
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) {
        before += __shfl_xor_sync(0xffffffffu, before, o);
        all_sum += __shfl_xor_sync(0xffffffffu, all_sum, o);
    }
    if (lane == 0) {
        *off = before;
        if (total) *total = all_sum;
    }
}

// out[*goff + j] = row0 + pos[j] for j < *count (the rank's slice of the
// concatenated result as int64 global row positions).
__global__ void concat_positions_kernel(const uint32_t* __restrict__ pos, const long long* count, long long row0,
                                        const long long* goff, long long* out, long long capacity,
                                        unsigned int* overflow) {
    const long long c = *count, o = *goff;
    if (o < 0 || o + c > capacity) {
        if (blockIdx.x == 0 && threadIdx.x == 0) atomicOr(overflow, 1u);
        return;
    }
    for (long long j = blockIdx.x * (long long)blockDim.x + threadIdx.x; j < c; j += (long long)gridDim.x * blockDim.x)
        out[o + j] = row0 + (long long)pos[j];
}

}  // namespace ard

namespace ar {
ar_status launch_exclusive_offset(const long long* all_counts, int world, int rank, long long* out, long long* total,
                                  cudaStream_t s) {
    ard::exclusive_offset_kernel<<<1, 32, 0, s>>>(all_counts, world, rank, out, total);
    AR_CHECK_LAUNCH("exclusive_offset_kernel");
    return AR_OK;
}
}  // namespace ar

struct ar_dist {
    ncclComm_t comm;
    int rank;
    int world;
};

static ar_status nccl_fail(ncclResult_t r, const char* where) {
    ar::set_error("%s: %s", where, ncclGetErrorString(r));
    return AR_ERR_NCCL;
}

#define AR_TRY_NCCL(expr)                                 \
    do {                                                  \
        ncclResult_t _r = (expr);                         \
        if (_r != ncclSuccess) return nccl_fail(_r, #expr); \
    } while (0)

extern "C" {

size_t ar_dist_unique_id_bytes(void) { return sizeof(ncclUniqueId); }

ar_status ar_dist_get_unique_id(void* id_out) {
    if (!id_out) {
        ar::set_error("ar_dist_get_unique_id: null output");
        return AR_ERR_INVALID;
    }
    ncclUniqueId id;
    AR_TRY_NCCL(ncclGetUniqueId(&id));
    memcpy(id_out, &id, sizeof(id));
    return AR_OK;
}

ar_status ar_dist_init(ar_dist** d, const void* unique_id, int32_t rank, int32_t world) {
    if (!d || !unique_id || world < 1 || rank < 0 || rank >= world) {
        ar::set_error("ar_dist_init: bad arguments (rank=%d world=%d)", rank, world);
        return AR_ERR_INVALID;
    }
    ncclUniqueId id;
    memcpy(&id, unique_id, sizeof(id));
    ncclComm_t comm;
    AR_TRY_NCCL(ncclCommInitRank(&comm, world, id, rank));
    ar_dist* h = new ar_dist{comm, rank, world};
    *d = h;
    return AR_OK;
}

ar_status ar_dist_offsets(ar_dist* d, const int64_t* local_count_dev, int64_t* all_counts_dev,
                          int64_t* global_offset_dev, void* stream) {
    if (!d || !local_count_dev || !all_counts_dev || !global_offset_dev) {
        ar::set_error("ar_dist_offsets: null argument");
        return AR_ERR_INVALID;
    }
    cudaStream_t s = (cudaStream_t)stream;
    AR_TRY_NCCL(ncclAllGather(local_count_dev, all_counts_dev, 1, ncclInt64, d->comm, s));
    return ar::launch_exclusive_offset((const long long*)all_counts_dev, d->world, d->rank,
                                       (long long*)global_offset_dev, nullptr, s);
}

ar_status ar_dist_shard_range(int64_t n, int32_t world, int32_t rank, int64_t* row0, int64_t* rows) {
    if (n < 0 || world < 1 || rank < 0 || rank >= world || !row0 || !rows) {
        ar::set_error("ar_dist_shard_range: bad arguments (n=%lld rank=%d world=%d)", (long long)n, rank, world);
        return AR_ERR_INVALID;
    }
    const int64_t per_raw = (n + world - 1) / world;
    const int64_t per = (per_raw + AR_SHARD_ALIGN_ROWS - 1) / AR_SHARD_ALIGN_ROWS * AR_SHARD_ALIGN_ROWS;
    const int64_t start = std::min<int64_t>(n, (int64_t)rank * per);
    const int64_t end = std::min<int64_t>(n, start + per);
    *row0 = start;
    *rows = end - start;
    return AR_OK;
}

ar_status ar_dist_exclusive_offsets(const int64_t* all_counts_dev, int32_t world, int32_t rank,
                                    int64_t* global_offset_dev, int64_t* total_dev, void* stream) {
    if (!all_counts_dev || !global_offset_dev || world < 1 || rank < 0 || rank >= world) {
        ar::set_error("ar_dist_exclusive_offsets: bad arguments (rank=%d world=%d)", rank, world);
        return AR_ERR_INVALID;
    }
    return ar::launch_exclusive_offset((const long long*)all_counts_dev, world, rank, (long long*)global_offset_dev,
                                       (long long*)total_dev, (cudaStream_t)stream);
}

ar_status ar_dist_concat_positions(const ar_positions* local, int64_t row0, const int64_t* global_offset_dev,
                                   int64_t* out_global, int64_t out_capacity, uint32_t* overflow_dev, void* stream) {
    if (!local || !local->pos || !local->count || !global_offset_dev || !out_global || !overflow_dev ||
        row0 < 0 || out_capacity < 0) {
        ar::set_error("ar_dist_concat_positions: null argument or negative row0 / capacity");
        return AR_ERR_INVALID;
    }
    if (local->capacity <= 0) return AR_OK;
    const int grid = (int)std::min<int64_t>((local->capacity + 255) / 256, (int64_t)ar::num_sms() * 4);
    ard::concat_positions_kernel<<<grid, 256, 0, (cudaStream_t)stream>>>(
        local->pos, (const long long*)local->count, (long long)row0, (const long long*)global_offset_dev,
        (long long*)out_global, (long long)out_capacity, overflow_dev);
    AR_CHECK_LAUNCH("concat_positions_kernel");
    return AR_OK;
}

ar_status ar_dist_sum(ar_dist* d, int64_t* values_dev, int32_t n, void* stream) {
    if (!d || !values_dev || n < 1) {
        ar::set_error("ar_dist_sum: bad argument");
        return AR_ERR_INVALID;
    }
    AR_TRY_NCCL(ncclAllReduce(values_dev, values_dev, (size_t)n, ncclInt64, ncclSum, d->comm, (cudaStream_t)stream));
    return AR_OK;
}

void ar_dist_free(ar_dist* d) {
    if (!d) return;
    ncclCommDestroy(d->comm);
    delete d;
}

}  // extern "C"

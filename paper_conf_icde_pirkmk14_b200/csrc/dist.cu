// dist.cu -- step a4: row-sharded multi-GPU exchange over NCCL (NVLink 5 /
// NVSwitch).  The paper never splits one query across GPUs;
// the build shards rows (BASELINE north_star): each rank scans its own row
// range, then exchanges 8-byte counts (ncclAllGather -> global offsets) and
// reduces the int64 SUM (ncclAllReduce).  Messages are tiny: latency-bound.
#include <nccl.h>

#include "kernels.cuh"

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
                                       (long long*)global_offset_dev, s);
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

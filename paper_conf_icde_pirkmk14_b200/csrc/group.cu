// group.cu -- the approximation group operator (s IV-E):
// "hash-based grouping to assign group IDs to unique values", the output
// positionally aligned with the input.  Rows are those of a position list
// (the candidate relation, or refined positions); the grouping value of a row
// is its approximate value (the bucket minimum base + (major << k), i.e. the
// pre-grouping on approximate values) or, in exact mode, the exact value
// ((major << k) | residual) + base.  Group ids are dense, 0 .. #groups - 1, in
// order of first insertion (so they depend on scheduling; the key of every id
// is written out).  ar_refine_group_sum_ids (refine.cu) then eliminates the
// selection's false positives and aggregates per id.
#include "kernels.cuh"

namespace ard {

struct GroupIdParams {
    const uint32_t* pos;
    const long long* count;
    AggCol key;                       // the grouping column (any layout, k, base, sign)
    int32_t exact;                    // 1: exact value (reads the residual), 0: approximate value
    unsigned long long* table;        // open addressing, linear probing; slot = (value << 32) | (id + 1), 0 = empty
    unsigned long long mask;          // slots - 1
    uint32_t max_groups;
    uint32_t* gids;                   // [count] group id per row (aligned with pos)
    uint32_t* group_keys;             // [max_groups] grouping value (a signed column's int32 bits) per id
    unsigned long long* ngroups;      // distinct values inserted (may exceed max_groups: then overflow)
    uint32_t* overflow;               // bit 0: more than max_groups values, bit 1: table full
};

constexpr unsigned long long kPending = 0xffffffffull;

__device__ __forceinline__ uint32_t mix32(uint32_t x) {   // murmur3 finaliser
    x ^= x >> 16;
    x *= 0x85ebca6bu;
    x ^= x >> 13;
    x *= 0xc2b2ae35u;
    x ^= x >> 16;
    return x;
}

// Id of grouping value v (key domain): find its slot, or claim an empty one, take the next id and
// publish it.  A thread that meets a claimed slot of the same value waits for the id.
__device__ uint32_t group_insert(const GroupIdParams& P, uint32_t v, uint32_t value_bits) {
    unsigned long long h = mix32(v) & P.mask;
    const unsigned long long tag = (unsigned long long)v << 32;
    for (unsigned long long probe = 0; probe <= P.mask; ++probe, h = (h + 1) & P.mask) {
        unsigned long long cur = ld_relaxed(P.table + h);
        if (cur == 0ull) {
            const unsigned long long prev = atomicCAS(P.table + h, 0ull, tag | kPending);
            if (prev == 0ull) {
                unsigned long long g = atomicAdd(P.ngroups, 1ull);
                if (g >= P.max_groups) {
                    atomicOr(P.overflow, 1u);
                    g = P.max_groups - 1;
                }
                P.group_keys[g] = value_bits;
                __threadfence();
                atomicExch(P.table + h, tag | (g + 1));
                return (uint32_t)g;
            }
            cur = prev;
        }
        if ((cur & ~0xffffffffull) == tag) {
            while ((cur & 0xffffffffull) == kPending) {
                __nanosleep(20);
                cur = ld_relaxed(P.table + h);
            }
            return (uint32_t)(cur & 0xffffffffull) - 1u;
        }
    }
    atomicOr(P.overflow, 2u);
    return 0u;
}

__global__ void __launch_bounds__(256) group_ids_kernel(const __grid_constant__ GroupIdParams P) {
    const long long count = *P.count;
    const AggCol& K = P.key;
    const long long stride = (long long)gridDim.x * blockDim.x;
    // whole warps walk the rows so that equal values of a warp are inserted once (__match_any_sync)
    const long long rounded = (count + 31) & ~31ll;
    for (long long j = blockIdx.x * (long long)blockDim.x + threadIdx.x; j < rounded; j += stride) {
        const bool active = j < count;
        uint32_t v = 0;
        if (active) {
            const uint64_t p = P.pos[j];
            if (P.exact) {
                v = value_get(K.major, K.residual, p, (int)K.w, (int)K.k, (int)K.layout, K.base, (int)K.rlayout);
            } else {
                const uint32_t m = major_get(K.major, p, (int)K.w, (int)K.layout);
                v = (K.k >= 32 ? 0u : (m << K.k)) + K.base;   // the bucket minimum: the approximate value
            }
        }
        const unsigned act = __ballot_sync(0xffffffffu, active);
        if (!active) continue;
        const unsigned same = __match_any_sync(act, v);
        const int leader = __ffs(same) - 1;
        uint32_t g = 0;
        if ((int)(threadIdx.x & 31) == leader) g = group_insert(P, v, v ^ K.flip);
        g = __shfl_sync(same, g, leader);
        P.gids[j] = g;
    }
}

}  // namespace ard

using namespace ar;

extern "C" {

size_t ar_group_table_bytes(int64_t slots) { return slots > 0 ? 8 * (size_t)slots : 0; }

ar_status ar_group_ids(const ar_positions* rows, const ar_column* key, int32_t mode, void* table, int64_t table_slots,
                       int32_t max_groups, uint32_t* gids_out, uint32_t* group_keys_out, int64_t* ngroups_dev,
                       uint32_t* overflow_dev, void* stream) {
    if (!rows || !rows->pos || !rows->count || !key || !table || !gids_out || !group_keys_out || !ngroups_dev ||
        !overflow_dev || (mode != AR_GROUP_APPROX && mode != AR_GROUP_EXACT)) {
        set_error("ar_group_ids: null argument or mode %d not AR_GROUP_APPROX / AR_GROUP_EXACT", mode);
        return AR_ERR_INVALID;
    }
    if (max_groups < 1 || table_slots < 2 * (int64_t)max_groups || (table_slots & (table_slots - 1)) != 0) {
        set_error("ar_group_ids: table_slots %lld must be a power of two >= 2 * max_groups (%d >= 1)",
                  (long long)table_slots, max_groups);
        return AR_ERR_RANGE;
    }
    if (key->d.w_major > 0 && !key->major) {
        set_error("ar_group_ids: key column without a major part");
        return AR_ERR_INVALID;
    }
    ard::GroupIdParams P;
    memset(&P, 0, sizeof(P));
    P.pos = rows->pos;
    P.count = (const long long*)rows->count;
    P.key.major = key->major;
    P.key.residual = key->residual;
    P.key.w = (uint32_t)key->d.w_major;
    P.key.k = (uint32_t)key->d.k;
    P.key.layout = (uint32_t)key->d.major_layout;
    P.key.base = key->d.base;
    P.key.rlayout = rlayout_code(key->d);
    P.key.flip = key->d.value_signed ? 0x80000000u : 0u;
    P.key.pred = -1;
    P.exact = (mode == AR_GROUP_EXACT && key->d.k > 0) ? 1 : 0;
    P.table = (unsigned long long*)table;
    P.mask = (unsigned long long)table_slots - 1;
    P.max_groups = (uint32_t)max_groups;
    P.gids = gids_out;
    P.group_keys = group_keys_out;
    P.ngroups = (unsigned long long*)ngroups_dev;
    P.overflow = overflow_dev;
    cudaStream_t s = (cudaStream_t)stream;
    AR_TRY_CUDA(cudaMemsetAsync(table, 0, 8 * (size_t)table_slots, s));
    AR_TRY_CUDA(cudaMemsetAsync(ngroups_dev, 0, sizeof(int64_t), s));
    AR_TRY_CUDA(cudaMemsetAsync(overflow_dev, 0, sizeof(uint32_t), s));
    if (rows->capacity <= 0) return AR_OK;
    const int grid = (int)std::min<int64_t>((rows->capacity + 255) / 256, (int64_t)num_sms() * 8);
    ard::group_ids_kernel<<<grid, 256, 0, s>>>(P);
    AR_CHECK_LAUNCH("group_ids_kernel");
    return AR_OK;
}

}  // extern "C"

// api.cu -- the C ABI (include/ar.h): argument validation, relaxation of the
// predicates (step a2, host scalars), workspace sizing and kernel launches.
#include <algorithm>
#include <cmath>
#include <cstring>
#include <new>

#include "kernels.cuh"

namespace ar {

static thread_local std::string g_err;

void set_error(const char* fmt, ...) {
    char buf[512];
    va_list ap;
    va_start(ap, fmt);
    vsnprintf(buf, sizeof(buf), fmt, ap);
    va_end(ap);
    g_err = buf;
}

ar_status cuda_fail(cudaError_t e, const char* where) {
    set_error("%s: %s (%s)", where, cudaGetErrorString(e), cudaGetErrorName(e));
    return AR_ERR_CUDA;
}

int num_sms() {
    static thread_local int cached_dev = -1, cached_sms = 0;
    int dev = 0, sms = 0;
    if (cudaGetDevice(&dev) != cudaSuccess) return 148;
    if (dev == cached_dev) return cached_sms;
    if (cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev) != cudaSuccess || sms <= 0) return 148;
    cached_dev = dev;
    cached_sms = sms;
    return sms;
}

int current_device() {
    int dev = 0;
    if (cudaGetDevice(&dev) != cudaSuccess) {
        cudaGetLastError();
        return 0;
    }
    return dev;
}

void opt_in_max_smem(const void* fn) {
    struct Done { int dev; const void* fn; };
    static thread_local Done done[128];
    static thread_local int used = 0;
    const int dev = current_device();
    for (int i = 0; i < used; ++i)
        if (done[i].fn == fn && done[i].dev == dev) return;
    int max_optin = 227 * 1024;
    cudaDeviceGetAttribute(&max_optin, cudaDevAttrMaxSharedMemoryPerBlockOptin, dev);
    cudaFuncAttributes a{};
    if (cudaFuncGetAttributes(&a, fn) == cudaSuccess)
        cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, max_optin - (int)a.sharedSizeBytes);
    cudaGetLastError();   // never leave a sticky error behind for a later launch check
    if (used < 128) done[used++] = Done{dev, fn};
}

// Step a2: exact [lo, hi] -> candidate / definite major ranges.
// In u = v - base units, bucket(m) = [m 2^k, m 2^k + 2^k - 1]:
//   cand(m) <=> m 2^k <= uhi && m 2^k + 2^k - 1 >= ulo  <=>  ulo >> k <= m <= uhi >> k
//   def(m)  <=> m 2^k >= ulo && m 2^k + 2^k - 1 <= uhi  <=>  ceil(ulo/2^k) <= m <= floor((uhi+1)/2^k) - 1
// Both ranges are clamped to the stored width (m <= 2^w - 1).
Relaxed relax(uint32_t lo, uint32_t hi, uint32_t base, int k, int w) {
    Relaxed R{};
    R.empty = true;
    if (lo > hi || hi < base) return R;
    const uint64_t ulo = lo < base ? 0 : (uint64_t)(lo - base);
    const uint64_t uhi = (uint64_t)(hi - base);
    const uint64_t maxm = w >= 32 ? 0xffffffffull : ((1ull << w) - 1);
    const uint64_t clo = ulo >> k, chi = std::min<uint64_t>(uhi >> k, maxm);
    if (clo > chi) return R;
    R.empty = false;
    R.clo = (uint32_t)clo;
    R.chi = (uint32_t)chi;
    const uint64_t two_k = 1ull << k;
    const uint64_t dlo = (ulo + two_k - 1) >> k;
    const uint64_t dtop = (uhi + 1) >> k;      // floor((uhi + 1) / 2^k)
    R.def_any = false;
    if (dtop >= 1) {
        const uint64_t dhi = std::min<uint64_t>(dtop - 1, maxm);
        if (dlo <= dhi) {
            R.def_any = true;
            R.dlo = (uint32_t)dlo;
            R.dhi = (uint32_t)dhi;
        }
    }
    return R;
}

static bool valid_col(const ar_column* c) { return c && (c->d.w_major == 0 || c->major); }

// Tuning knobs (read once): AR_STAGES (pipeline stages), AR_CTAS (CTAs per SM).
static int env_int(const char* name, int dflt) {
    const char* v = getenv(name);
    return (v && *v) ? atoi(v) : dflt;
}
static int knob(int which) {
    static int vals[2] = {-2, -2};
    static const char* names[2] = {"AR_STAGES", "AR_CTAS"};
    if (vals[which] == -2) vals[which] = env_int(names[which], 0);
    return vals[which];
}

// Pipeline sizing: the most CTAs per SM (up to 4) that still allow >= 3 stages
// (>= 2 at one CTA per SM), and for that occupancy the deepest ring (<= 8 stages).
static uint32_t pick_stages_uncached(const void* fn, uint32_t stage_words, bool fused, int* ctas_per_sm) {
    const int force_st = knob(0), force_occ = knob(1);
    for (int occ_target = force_occ > 0 ? force_occ : 4; occ_target >= 1; --occ_target) {
        for (int st = 8; st >= 2; --st) {
            if (force_st > 0 && st != force_st) continue;
            const size_t smem = select_smem_bytes(stage_words, (uint32_t)st, !fused);
            if (smem > 227 * 1024) continue;
            const int occ = select_occupancy(fn, smem, fused);
            if (occ >= occ_target && (st >= 3 || occ_target == 1 || force_st > 0)) {
                *ctas_per_sm = occ_target;
                return (uint32_t)st;
            }
        }
        if (force_occ > 0) break;
    }
    *ctas_per_sm = 1;
    return 2;
}

// Memoised per (device, kernel, stage_words): the occupancy queries stay out of the launch path.
static uint32_t pick_stages(const void* fn, uint32_t stage_words, bool fused, int* ctas_per_sm) {
    struct Entry { int dev; const void* fn; uint32_t words; uint32_t stages; int occ; };
    static thread_local Entry cache[32];
    static thread_local int used = 0;
    const int dev = current_device();
    for (int i = 0; i < used; ++i)
        if (cache[i].fn == fn && cache[i].words == stage_words && cache[i].dev == dev) {
            *ctas_per_sm = cache[i].occ;
            return cache[i].stages;
        }
    const uint32_t st = pick_stages_uncached(fn, stage_words, fused, ctas_per_sm);
    if (used < 32) cache[used++] = Entry{dev, fn, stage_words, st, *ctas_per_sm};
    return st;
}

}  // namespace ar

using namespace ar;

extern "C" {

const char* ar_status_str(ar_status s) {
    switch (s) {
        case AR_OK: return "AR_OK";
        case AR_ERR_INVALID: return "AR_ERR_INVALID";
        case AR_ERR_RANGE: return "AR_ERR_RANGE";
        case AR_ERR_CUDA: return "AR_ERR_CUDA";
        case AR_ERR_NCCL: return "AR_ERR_NCCL";
        case AR_ERR_UNSUPPORTED: return "AR_ERR_UNSUPPORTED";
    }
    return "AR_ERR_?";
}

const char* ar_last_error(void) { return g_err.c_str(); }
const char* ar_version(void) { return "ar-b200 0.1 (sm_100a)"; }
static thread_local const char* g_last_scan = "";
const char* ar_last_scan_kernel(void) { return g_last_scan; }

// ------------------------------------------------------------------ a1

size_t ar_decompose_ws_bytes(void) { return 256; }

ar_status ar_decompose_plan(const uint32_t* col, int64_t n, int32_t major_bits, int32_t major_layout,
                            int32_t residual_loc, uint32_t base, int32_t flags, void* ws, size_t ws_bytes,
                            ar_column_desc* desc, void* stream) {
    if (!desc || n < 0 || n >= (int64_t)1 << 32 || (n > 0 && !col)) {
        set_error("ar_decompose_plan: bad column pointer / size (n=%lld)", (long long)n);
        return AR_ERR_INVALID;
    }
    if (major_bits < 1 || major_bits > 32) {
        set_error("ar_decompose_plan: major_bits=%d outside [1,32]", major_bits);
        return AR_ERR_INVALID;
    }
    if ((major_layout != AR_LAYOUT_SLICED && major_layout != AR_LAYOUT_PACKED) ||
        (residual_loc != AR_LOC_DEVICE && residual_loc != AR_LOC_HOST_PINNED) ||
        (flags & ~(AR_DECOMPOSE_SIGNED | AR_DECOMPOSE_BASE_MIN | AR_DECOMPOSE_SPLIT(31))) != 0) {
        set_error("ar_decompose_plan: bad layout (%d), residual location (%d) or flags (%d)", major_layout,
                  residual_loc, flags);
        return AR_ERR_INVALID;
    }
    if (!ws || ws_bytes < ar_decompose_ws_bytes()) {
        set_error("ar_decompose_plan: workspace of %zu bytes < %zu", ws_bytes, ar_decompose_ws_bytes());
        return AR_ERR_INVALID;
    }
    cudaStream_t s = (cudaStream_t)stream;
    const int k = 32 - major_bits;
    const int split = (flags >> 8) & 31;
    if (split && !(k <= 8 && split < k)) {
        set_error("ar_decompose_plan: AR_DECOMPOSE_SPLIT(%d) needs 1 <= h < k <= 8 (k = %d)", split, k);
        return AR_ERR_INVALID;
    }
    const uint32_t flip = (flags & AR_DECOMPOSE_SIGNED) ? 0x80000000u : 0u;
    uint32_t mm[2] = {0u, 0xffffffffu};   // max(d), min(d)
    if (n > 0) {
        AR_TRY_CUDA(cudaMemcpyAsync(ws, mm, 8, cudaMemcpyHostToDevice, s));
        ar_status st = launch_decompose_minmax(col, n, flip, (uint32_t*)ws, s);
        if (st != AR_OK) return st;
        AR_TRY_CUDA(cudaMemcpyAsync(mm, ws, 8, cudaMemcpyDeviceToHost, s));
        AR_TRY_CUDA(cudaStreamSynchronize(s));
    }
    if (flags & AR_DECOMPOSE_BASE_MIN) base = n > 0 ? mm[1] : 0u;
    if (n > 0 && mm[1] < base) {
        set_error("ar_decompose_plan: base %u exceeds the column minimum %u (key domain)", base, mm[1]);
        return AR_ERR_RANGE;
    }
    const uint32_t maxu = n > 0 ? mm[0] - base : 0u;
    const uint32_t maxm = k >= 32 ? 0 : (maxu >> k);
    int w = 0;
    while (w < 32 && (maxm >> w) != 0) ++w;
    memset(desc, 0, sizeof(*desc));
    desc->n = n;
    desc->major_bits = major_bits;
    desc->k = k;
    desc->w_major = w;
    desc->major_layout = major_layout;
    desc->residual_loc = residual_loc;
    desc->base = base;
    desc->major_bytes = major_layout == AR_LAYOUT_SLICED ? sliced_bytes(n, w) : packed_bytes(n, w);
    desc->residual_layout = (k >= 1 && k <= 8) ? AR_LAYOUT_SLICED : AR_LAYOUT_PACKED;
    desc->residual_split = split;
    desc->residual_bytes = split ? split_bytes(n, k)
                                 : (desc->residual_layout == AR_LAYOUT_SLICED ? sliced_bytes(n, k) : packed_bytes(n, k));
    desc->value_signed = flip ? 1 : 0;
    return AR_OK;
}

static ar_status check_desc(const ar_column_desc* d);

ar_status ar_decompose_set_width(ar_column_desc* desc, int32_t w_major) {
    ar_status st = check_desc(desc);
    if (st != AR_OK) return st;
    if (w_major < desc->w_major || w_major > desc->major_bits) {
        set_error("ar_decompose_set_width: w_major %d outside [%d (planned), %d (major_bits)]", w_major, desc->w_major,
                  desc->major_bits);
        return AR_ERR_RANGE;
    }
    desc->w_major = w_major;
    desc->major_bytes = desc->major_layout == AR_LAYOUT_SLICED ? sliced_bytes(desc->n, w_major)
                                                                : packed_bytes(desc->n, w_major);
    return AR_OK;
}

static ar_status check_desc(const ar_column_desc* d) {
    if (!d || d->n < 0 || d->n >= (int64_t)1 << 32 || d->major_bits < 1 || d->major_bits > 32 ||
        d->k != 32 - d->major_bits || d->w_major < 0 || d->w_major > d->major_bits ||
        (d->major_layout != AR_LAYOUT_SLICED && d->major_layout != AR_LAYOUT_PACKED) ||
        (d->residual_loc != AR_LOC_DEVICE && d->residual_loc != AR_LOC_HOST_PINNED) ||
        (d->major_loc != AR_LOC_DEVICE && d->major_loc != AR_LOC_HOST_PINNED) ||
        (d->residual_layout != AR_LAYOUT_SLICED && d->residual_layout != AR_LAYOUT_PACKED) ||
        (d->residual_layout == AR_LAYOUT_SLICED && d->k > 8) ||
        (d->value_signed != 0 && d->value_signed != 1) || d->residual_split < 0 ||
        (d->residual_split > 0 && (d->residual_layout != AR_LAYOUT_SLICED || d->residual_split >= d->k))) {
        set_error("invalid ar_column_desc");
        return AR_ERR_INVALID;
    }
    // the kernels read whole 16-B groups of every part (TMA bulk copies, vector gathers): the
    // descriptor must promise at least the bytes its geometry implies
    const uint64_t need_major = d->major_layout == AR_LAYOUT_SLICED ? sliced_bytes(d->n, d->w_major)
                                                                     : packed_bytes(d->n, d->w_major);
    const uint64_t need_res = d->k == 0 ? 0
                              : d->residual_split ? split_bytes(d->n, d->k)
                              : (d->residual_layout == AR_LAYOUT_SLICED ? sliced_bytes(d->n, d->k)
                                                                        : packed_bytes(d->n, d->k));
    if (d->major_bytes < need_major || d->residual_bytes < need_res) {
        set_error("ar_column_desc: major_bytes %llu / residual_bytes %llu below the %llu / %llu its geometry needs",
                  (unsigned long long)d->major_bytes, (unsigned long long)d->residual_bytes,
                  (unsigned long long)need_major, (unsigned long long)need_res);
        return AR_ERR_RANGE;
    }
    return AR_OK;
}

static ar_status device_alias(const void* p, int loc, const uint32_t** out) {
    if (!p || loc == AR_LOC_DEVICE) {
        *out = (const uint32_t*)p;
        return AR_OK;
    }
    void* dp = nullptr;
    cudaError_t e = cudaHostGetDevicePointer(&dp, const_cast<void*>(p), 0);
    if (e != cudaSuccess) {
        cudaGetLastError();
        set_error("residual buffer is not mapped pinned host memory (%s)", cudaGetErrorString(e));
        return AR_ERR_CUDA;
    }
    *out = (const uint32_t*)dp;
    return AR_OK;
}

ar_status ar_column_wrap(const ar_column_desc* desc, const void* major_buf, const void* residual_buf,
                         ar_column** out) {
    ar_status st = check_desc(desc);
    if (st != AR_OK) return st;
    if (!out || (desc->major_bytes > 0 && !major_buf) || (desc->residual_bytes > 0 && !residual_buf)) {
        set_error("ar_column_wrap: null buffer or output");
        return AR_ERR_INVALID;
    }
    if (((uintptr_t)major_buf & 15u) || ((uintptr_t)residual_buf & 15u)) {
        set_error("ar_column_wrap: part buffers must be 16-B aligned (TMA bulk copies / vector loads)");
        return AR_ERR_INVALID;
    }
    const uint32_t* res = nullptr;
    st = device_alias(residual_buf, desc->residual_loc, &res);
    if (st != AR_OK) return st;
    const uint32_t* maj = nullptr;
    st = device_alias(major_buf, desc->major_loc, &maj);
    if (st != AR_OK) return st;
    ar_column* c = new (std::nothrow) ar_column;
    if (!c) {
        set_error("out of host memory");
        return AR_ERR_RANGE;
    }
    c->d = *desc;
    c->major = maj;
    c->residual = desc->k > 0 ? res : nullptr;
    *out = c;
    return AR_OK;
}

ar_status ar_decompose(const uint32_t* col, const ar_column_desc* desc, void* major_buf, uint64_t major_buf_bytes,
                       void* residual_buf, uint64_t residual_buf_bytes, void* stream, ar_column** out) {
    ar_status st = check_desc(desc);
    if (st != AR_OK) return st;
    if (!out || (desc->n > 0 && !col)) {
        set_error("ar_decompose: null column or output handle");
        return AR_ERR_INVALID;
    }
    if (major_buf_bytes < desc->major_bytes || residual_buf_bytes < desc->residual_bytes) {
        set_error("ar_decompose: buffers (%llu, %llu bytes) smaller than planned (%llu, %llu)",
                  (unsigned long long)major_buf_bytes, (unsigned long long)residual_buf_bytes,
                  (unsigned long long)desc->major_bytes, (unsigned long long)desc->residual_bytes);
        return AR_ERR_RANGE;
    }
    ar_column* c = nullptr;
    st = ar_column_wrap(desc, major_buf, residual_buf, &c);
    if (st != AR_OK) return st;
    cudaStream_t s = (cudaStream_t)stream;
    const int64_t n = desc->n;
    const int w = desc->w_major, k = desc->k;
    const uint32_t flip = desc->value_signed ? 0x80000000u : 0u;
    if (w > 0) {
        uint32_t* mdst = const_cast<uint32_t*>(c->major);   // device alias (mapped when host-resident)
        if (desc->major_layout == AR_LAYOUT_SLICED)
            st = launch_pack_sliced(col, n, k, 0xffffffffu, flip, desc->base, w, mdst, s);
        else
            st = launch_pack_packed(col, n, k, 0xffffffffu, flip, desc->base, w, desc->major_bytes / 4, mdst, s);
    }
    if (st == AR_OK && k > 0) {
        uint32_t* rdst = const_cast<uint32_t*>(c->residual);
        if (desc->residual_split)
            st = launch_pack_split(col, n, k, desc->residual_split, flip, desc->base, rdst, s);
        else if (desc->residual_layout == AR_LAYOUT_SLICED)
            st = launch_pack_sliced(col, n, 0, (1u << k) - 1u, flip, desc->base, k, rdst, s);
        else
            st = launch_pack_packed(col, n, 0, (1u << k) - 1u, flip, desc->base, k, desc->residual_bytes / 4, rdst,
                                    s);
    }
    if (st != AR_OK) {
        delete c;
        return st;
    }
    *out = c;
    return AR_OK;
}

ar_status ar_column_get_desc(const ar_column* col, ar_column_desc* desc) {
    if (!col || !desc) {
        set_error("ar_column_get_desc: null argument");
        return AR_ERR_INVALID;
    }
    *desc = col->d;
    return AR_OK;
}

void ar_column_free(ar_column* col) { delete col; }

// ------------------------------------------------------------- a2 + a3

// Select workspace: per-tile counts (u32) + offsets (u64) + tile-local candidate slices (pos, aux).
// Select workspace, for tiles of >= kSelMinTileRows rows (T_max of them):
//   [group sums u64 x G][tile counts u32 x T_max][pad to 128 B]
//   [tmp_pos u32 x S][tmp_aux u32 x S]
// S = n rounded up to kSelMinTileRows (>= the end of the last tile's slice).
namespace {
struct SelWs {
    uint64_t groups, tiles, slice_rows, counts_bytes, tmp_off, bytes;
};
SelWs sel_ws(int64_t n) {
    SelWs w;
    const uint64_t rows = (uint64_t)std::max<int64_t>(n, 0);
    w.tiles = ceil_div_u64(rows, ard::kSelMinTileRows);
    w.groups = (w.tiles >> ard::kGroupShift) + 1;
    w.slice_rows = w.tiles * ard::kSelMinTileRows;
    w.counts_bytes = 8 * w.groups + 4 * w.tiles;                  // zeroed per call
    w.tmp_off = (w.counts_bytes + 127) & ~uint64_t(127);
    w.bytes = 128 + w.tmp_off + 8 * w.slice_rows;                 // + 128: base alignment
    return w;
}
}  // namespace

size_t ar_select_ws_bytes(int64_t n) { return (size_t)sel_ws(n).bytes; }

// Shared predicate setup of ar_approx_select / ar_select_refine_sum.
static ar_status setup_scan(const ar_pred* preds, int32_t npred, ard::SelParams& P, bool& empty, int64_t& n,
                            bool fused) {
    if (npred < 0 || npred > AR_MAX_PRED || (npred > 0 && !preds)) {
        set_error("npred=%d outside [0,%d] or preds == NULL", npred, AR_MAX_PRED);
        return AR_ERR_INVALID;
    }
    if (npred == 0) {
        set_error("npred == 0: a scan needs at least one predicate column (use [0, 2^32-1] to keep all rows)");
        return AR_ERR_INVALID;
    }
    memset(&P, 0, sizeof(P));
    empty = false;
    n = preds[0].col ? preds[0].col->d.n : -1;
    P.bpt = (uint32_t)kernel_bpt(fused);
    static const int suspend_ns = env_int("AR_SUSPEND_NS", 0);
    P.suspend_ns = (uint32_t)suspend_ns;
    static const int prod_wait = env_int("AR_PROD_WAIT", 0);
    P.prod_wait = (uint32_t)prod_wait;
    static const int debug = env_int("AR_DEBUG", 0);
    P.debug = (uint32_t)debug;
    P.tile_rows = (uint32_t)kernel_warps(fused) * 32u * 32u * P.bpt;
    uint32_t words = 0, ashift = 0;
    for (int c = 0; c < npred; ++c) {
        const ar_column* col = preds[c].col;
        if (!valid_col(col) || col->d.n != n) {
            set_error("predicate %d: null column or n differs from predicate 0", c);
            return AR_ERR_INVALID;
        }
        if (col->d.major_layout != AR_LAYOUT_SLICED || col->d.major_loc != AR_LOC_DEVICE) {
            set_error("predicate %d: the approximate scan needs AR_LAYOUT_SLICED majors in device memory", c);
            return AR_ERR_INVALID;
        }
        const int w = col->d.w_major, k = col->d.k;
        const uint32_t flip = col->d.value_signed ? 0x80000000u : 0u;
        const uint32_t plo = preds[c].lo ^ flip, phi = preds[c].hi ^ flip;   // key domain
        const Relaxed R = relax(plo, phi, col->d.base, k, w);
        if (R.empty) empty = true;
        ard::SelPred& p = P.p[c];
        p.planes = col->major;
        p.w = (uint32_t)w;
        p.mode = k == 0 ? 0u : (R.def_any ? 1u : 2u);
        p.clo = R.clo;
        p.chi = R.chi;
        p.dlo = R.dlo;
        p.dhi = R.dhi;
        p.soff = words;
        p.ashift = ashift;
        p.residual = col->residual;
        p.k = (uint32_t)k;
        p.base = col->d.base;
        p.lo = plo;
        p.hi = phi;
        p.rlayout = rlayout_code(col->d);
        p.res_host = col->d.residual_loc == AR_LOC_HOST_PINNED ? 1u : 0u;
        p.res_hint = 1u;
        p.rsplit = (uint32_t)col->d.residual_split;
        if (p.rsplit && !R.empty) {   // progressive refinement: the high residual planes refine the buckets to 2^(k-h)
            const int kk = k - (int)p.rsplit, ww = w + (int)p.rsplit;
            const Relaxed Rh = relax(plo, phi, col->d.base, kk, ww);
            // Fine bucket U of a candidate that is not definite is clo or chi.  The definite bounds are
            // chosen so that U < dlo <=> U == clo and U > dhi <=> U == chi on those rows (the check code of
            // the result-ring kernel): the relaxation's when it has a definite bucket, else the empty
            // [clo + 1, clo] (chi == clo + 1) or [clo + 1, clo - 1] (chi == clo); where clo + 1 or clo - 1
            // leaves the w + h bits, that code bit is forced through scor.
            const uint64_t maxf = ww >= 32 ? 0xffffffffull : ((1ull << ww) - 1);
            uint64_t dlo = Rh.dlo, dhi = Rh.dhi;
            p.scor = 0;
            if (!Rh.def_any) {
                dlo = (uint64_t)Rh.clo + 1;
                if (dlo > maxf) {
                    dlo = maxf;
                    p.scor |= 1u;
                }
                if (Rh.chi == Rh.clo) {
                    if (Rh.clo == 0) {
                        dhi = 0;
                        p.scor |= 2u;
                    } else {
                        dhi = (uint64_t)Rh.clo - 1;
                    }
                } else {
                    dhi = Rh.clo;
                }
            }
            for (int i = 0; i < ww && i < 32; ++i) {
                P.pmh[c][i][0] = 0u - ((Rh.clo >> i) & 1u);
                P.pmh[c][i][1] = 0u - ((Rh.chi >> i) & 1u);
                P.pmh[c][i][2] = 0u - (uint32_t)((dlo >> i) & 1u);
                P.pmh[c][i][3] = 0u - (uint32_t)((dhi >> i) & 1u);
            }
        }
        words += (P.tile_rows / 32) * (uint32_t)w;
        ashift += (uint32_t)w;
        // the one-pass kernel streams device-resident SLICED residual tiles (k <= 8) with the
        // majors and evaluates the exact predicate on major + residual planes in place -- when
        // most 32-row blocks would need a residual gather anyway (a block's k planes are one
        // sector).  Estimate with majors uniform over [0, 2^w): the non-definite candidate
        // buckets (at most the two boundary ones) hold f of the rows and a block is touched with
        // probability 1 - (1 - f)^32; stream iff that is >= 1/2 (f >= 2.14 %).
        // AR_RES_STREAM=0/1 forces the choice.
        bool stream_res = false;
        if (fused && k > 0 && col->d.residual_loc == AR_LOC_DEVICE && col->residual &&
            col->d.residual_layout == AR_LAYOUT_SLICED && col->d.residual_split == 0 && !R.empty) {
            static const int force = env_int("AR_RES_STREAM", -1);
            const double buckets = std::ldexp(1.0, w);
            const double nondef = (double)(R.chi - R.clo + 1) - (R.def_any ? (double)(R.dhi - R.dlo + 1) : 0.0);
            const double f = std::min(1.0, nondef / buckets);
            stream_res = force >= 0 ? force != 0 : (1.0 - std::pow(1.0 - f, 32.0)) >= 0.5;
        }
        if (stream_res) {
            p.res_stream = 1;
            p.res_soff = words;
            words += (P.tile_rows / 32) * (uint32_t)k;
        }
        // a split residual in HBM: the one-pass kernel streams its h high planes (the fine
        // buckets decide most rows) and gathers the low planes of the rows they leave undecided
        if (p.rsplit && !R.empty) {   // the low bits of the exact bounds (check entries of the one-pass kernels)
            const uint32_t kl = (uint32_t)k - p.rsplit;
            const uint64_t maxu = (uint64_t)k + w >= 32 ? 0xffffffffull : ((1ull << (k + w)) - 1);
            const uint64_t ulo = plo < col->d.base ? 0 : (uint64_t)(plo - col->d.base);
            const uint64_t uhi = std::min<uint64_t>((uint64_t)(phi - col->d.base), maxu);
            p.sflo = (uint32_t)(ulo >> kl);
            p.sfhi = (uint32_t)(uhi >> kl);
            p.sllo = (uint32_t)(ulo & ((1u << kl) - 1u));
            p.slhi = (uint32_t)(uhi & ((1u << kl) - 1u));
        }
        if (fused && p.rsplit && col->d.residual_loc == AR_LOC_DEVICE && col->residual && !R.empty &&
            env_int("AR_SPLIT_STREAM", 1) != 0) {
            p.res_stream = 1;
            p.res_soff = words;
            words += (P.tile_rows / 32) * p.rsplit;
        }
    }
    uint32_t planes = 0;
    for (int c = 0; c < npred; ++c) planes += P.p[c].w;
    if (planes > AR_MAX_PLANES) {
        set_error("sum of w_major over predicates = %u > AR_MAX_PLANES (%d)", planes, AR_MAX_PLANES);
        return AR_ERR_UNSUPPORTED;
    }
    // exact-bound masks for the one-pass kernel: bit i of u = v - base over the
    // concatenated residual (i < k) and major (k <= i < k + w) planes
    P.exact_mode = fused ? 1 : 0;
    for (int c = 0; c < npred; ++c) {
        const ard::SelPred& p = P.p[c];
        if (p.k > 0 && !p.res_stream) P.exact_mode = 0;
        if (p.k == 0) continue;   // (also used by the gathered-residual kernel, fused.cu)
        const uint64_t maxu = p.k + p.w >= 32 ? 0xffffffffull : ((1ull << (p.k + p.w)) - 1);
        const uint64_t ulo = p.lo < p.base ? 0 : (uint64_t)(p.lo - p.base);
        const uint64_t uhi = std::min<uint64_t>((uint64_t)(p.hi - p.base), maxu);
        for (uint32_t i = 0; i < p.k + p.w && i < 32; ++i) {
            P.pmx[c][i][0] = 0u - (uint32_t)((ulo >> i) & 1u);
            P.pmx[c][i][1] = 0u - (uint32_t)((uhi >> i) & 1u);
        }
    }
    for (int c = 0; c < npred; ++c) {
        ard::SelPred& p = P.p[c];
        // Mode 2 (no definite bucket): an empty definite range chosen so that, on a non-definite
        // candidate, "below it" <=> major == clo and "above it" <=> major == chi -- [clo + 1, clo]
        // (chi == clo + 1) or [clo + 1, clo - 1] (chi == clo) -- the check code of the
        // gathered-residual kernel's bit-packed residuals (as for split residuals, setup_scan above);
        // where clo + 1 / clo - 1 leaves the w bits, that code bit is forced through scor.  Mode 1:
        // the relaxation's own definite range has the property.
        uint64_t dlo = p.dlo, dhi = p.dhi;
        if (p.mode == 2) {
            const uint64_t maxm = p.w >= 32 ? 0xffffffffull : ((1ull << p.w) - 1);
            const uint32_t scor0 = p.k > 8 ? 0u : p.scor;
            uint32_t scor = 0;
            dlo = (uint64_t)p.clo + 1;
            if (dlo > maxm) {
                dlo = maxm;
                scor |= 1u;
            }
            if (p.chi == p.clo) {
                if (p.clo == 0) {
                    dhi = 0;
                    scor |= 2u;
                } else {
                    dhi = (uint64_t)p.clo - 1;
                }
            } else {
                dhi = p.clo;
            }
            if (p.k > 8) p.scor = scor; else p.scor = scor0;
        }
        for (uint32_t j = 0; j < p.w; ++j) {
            uint32_t* m = P.pm[p.ashift + j];
            m[0] = 0u - ((p.clo >> j) & 1u);
            m[1] = 0u - ((p.chi >> j) & 1u);
            m[2] = 0u - (uint32_t)((dlo >> j) & 1u);
            m[3] = 0u - (uint32_t)((dhi >> j) & 1u);
        }
        if (p.k > 8 && p.mode != 0) {   // bit-packed residual: the low k bits of the exact bounds (check entries)
            const uint64_t maxu = (uint64_t)p.k + p.w >= 32 ? 0xffffffffull : ((1ull << (p.k + p.w)) - 1);
            const uint64_t ulo = p.lo < p.base ? 0 : (uint64_t)(p.lo - p.base);
            const uint64_t uhi = std::min<uint64_t>((uint64_t)(p.hi - p.base), maxu);
            const uint64_t km = p.k >= 32 ? 0xffffffffull : ((1ull << p.k) - 1);
            p.sllo = (uint32_t)(ulo & km);
            p.slhi = (uint32_t)(uhi & km);
        }
    }
    P.npred = npred;
    P.n = n;
    P.num_tiles = (int64_t)ceil_div_u64((uint64_t)n, P.tile_rows);
    P.stage_words = std::max<uint32_t>(words, 4);
    return AR_OK;
}

ar_status ar_approx_select(const ar_pred* preds, int32_t npred, int32_t flags, ar_cands* out, void* ws,
                           size_t ws_bytes, void* stream) {
    ard::SelParams P;
    bool empty = false;
    int64_t n = 0;
    ar_status st = setup_scan(preds, npred, P, empty, n, false);
    if (st != AR_OK) return st;
    if (!out || !out->pos || !out->aux || !out->count) {
        set_error("ar_approx_select: null output buffer");
        return AR_ERR_INVALID;
    }
    if (out->capacity < n) {
        set_error("ar_approx_select: capacity %lld < n %lld", (long long)out->capacity, (long long)n);
        return AR_ERR_RANGE;
    }
    if (!ws || ws_bytes < ar_select_ws_bytes(n)) {
        set_error("ar_approx_select: workspace %zu < %zu bytes", ws_bytes, ar_select_ws_bytes(n));
        return AR_ERR_RANGE;
    }
    const bool carry = (flags & AR_SELECT_CARRY_APPR) != 0;
    uint32_t abits = 0;
    for (int c = 0; c < npred; ++c) abits += P.p[c].w;
    if (carry && abits > 31) {
        set_error("AR_SELECT_CARRY_APPR: approximation tuple of %u bits does not fit aux bits 0..30", abits);
        return AR_ERR_RANGE;
    }
    out->appr_bits = carry ? (int32_t)std::max<uint32_t>(abits, 1) : 0;
    cudaStream_t s = (cudaStream_t)stream;
    g_last_scan = "";
    if (empty || n == 0) {   // no kernel runs: the count is set here (otherwise the kernels write it)
        AR_TRY_CUDA(cudaMemsetAsync(out->count, 0, sizeof(int64_t), s));
        return AR_OK;
    }
    P.carry = carry ? 1 : 0;
    P.out_pos = out->pos;
    P.out_aux = out->aux;
    P.out_count = (long long*)out->count;
    // workspace (sel_ws): group sums and tile counts (zeroed), tile slices
    const SelWs L = sel_ws(n);
    char* base = (char*)(((uintptr_t)ws + 127) & ~uintptr_t(127));
    // one-kernel ordered select (default): round-robin look-back over per-tile counts (status words,
    // zeroed), entries written once at their final offsets -- no tile slices, no compaction
    // AR_SEL_RR: 0 = never, 2 = always, 1 (default) = when a tile's major planes total >= kRrMinPlanes
    // words per block and the candidate major ranges cover at most kRrEntries / tile_rows of the major
    // domains (product over predicates): with narrower planes the per-tile look-back does not
    // amortise, and tiles past the staging buffer take the slower dense paths (C3 at 8 planes 0.385
    // vs 0.352 ms, at 10 % selectivity 1.39 vs 1.10 ms; Q6: 0.329 vs 0.346 ms; DESIGN s6.2).  Both
    // kernels give the same result; this only picks the faster one.
    static const int rr = env_int("AR_SEL_RR", 1);
    uint32_t planes = 0;
    double frac = 1.0;
    for (int c = 0; c < npred; ++c) {
        const ard::SelPred& p = P.p[c];
        planes += p.w;
        frac *= p.w >= 32 ? ((double)p.chi - p.clo + 1.0) / 4294967296.0
                          : ((double)p.chi - p.clo + 1.0) / (double)(1ull << p.w);
    }
    const bool use_rr = rr == 2 || (rr == 1 && planes >= (uint32_t)ard::kRrMinPlanes &&
                                     frac * P.tile_rows <= (double)ard::kRrEntries);
    const void* rr_fn = use_rr ? select_rr_kernel_fn(P) : nullptr;
    if (rr_fn) {
        static const int rr_bufs = std::min(4, std::max(1, env_int("AR_SEL_RR_BUFS", 1)));
        P.nstages = (uint32_t)rr_bufs;
        P.status = (unsigned long long*)base;   // 8 * num_tiles <= L.counts_bytes
        AR_TRY_CUDA(cudaMemsetAsync(base, 0, 8 * (size_t)P.num_tiles, s));
        P.tmp_pos = (uint32_t*)(base + L.tmp_off);   // slices of dense tiles (> kRrEntries candidates)
        P.tmp_aux = P.tmp_pos + L.slice_rows;
        const size_t smem = select_rr_smem_bytes(P.stage_words, P.nstages);
        const int occ = select_occupancy(rr_fn, smem, false);
        if (occ > 0) {
            static const int rr_ctas = env_int("AR_SEL_RR_CTAS", 0);   // CTAs per SM (0: as many as fit)
            const int per_sm = rr_ctas > 0 ? std::min(rr_ctas, occ) : occ;
            static const int max_grid = env_int("AR_SEL_RR_GRID", 0);   // tests: force several rounds
            int grid = (int)std::min<int64_t>(P.num_tiles, (int64_t)num_sms() * per_sm);
            if (max_grid > 0) grid = std::min(grid, max_grid);
            g_last_scan = "select_rr_kernel";
            return launch_select_rr(rr_fn, P, grid, smem, s);
        }
    }
    P.group_sum = (unsigned long long*)base;
    P.tile_count = (uint32_t*)(base + 8 * L.groups);
    AR_TRY_CUDA(cudaMemsetAsync(base, 0, L.counts_bytes, s));
    P.tmp_pos = (uint32_t*)(base + L.tmp_off);
    P.tmp_aux = P.tmp_pos + L.slice_rows;
    g_last_scan = "select_tile_kernel";
    const void* fn = select_kernel_fn(P, false);
    // one tile per CTA (default): measured fastest -- the kernel is issue-bound, and persistent CTAs
    // with AR_SEL_BUFS = 2 / 3 tile buffers each (the next tiles' loads in flight while one is decided)
    // ran 2 % / 12 % slower on C4 (DESIGN s6.2)
    static const int bufs = std::min(4, std::max(1, env_int("AR_SEL_BUFS", 1)));
    P.nstages = (uint32_t)bufs;
    const size_t smem = select_smem_bytes(P.stage_words, P.nstages, true);
    int grid = (int)P.num_tiles;
    if (bufs > 1) {
        const int occ = std::max(1, select_occupancy(fn, smem, false));
        grid = (int)std::min<int64_t>(P.num_tiles, (int64_t)num_sms() * occ);
    }
    ar_status st2 = launch_scan(fn, P, grid, smem, false, s);
    if (st2 != AR_OK) return st2;
    return launch_select_rest(P, env_int("AR_SEL_PDL", 1) != 0, s);
}

// ------------------------------------------------------------------ a5

size_t ar_refine_ws_bytes(int64_t capacity) {
    return 16 + 8 * ceil_div_u64((uint64_t)std::max<int64_t>(capacity, 0), ard::kRefTile);
}

static ar_status setup_refine(const ar_cands* in, const ar_pred* preds, int32_t npred, ard::RefParams& P) {
    if (!in || !in->pos || !in->aux || !in->count || npred < 1 || npred > AR_MAX_PRED || !preds) {
        set_error("refine: null candidates or bad predicate list (npred=%d)", npred);
        return AR_ERR_INVALID;
    }
    memset(&P, 0, sizeof(P));
    uint32_t ashift = 0, abits = 0;
    for (int c = 0; c < npred; ++c) {
        const ar_column* col = preds[c].col;
        if (!valid_col(col)) {
            set_error("refine: predicate %d has a null column", c);
            return AR_ERR_INVALID;
        }
        ard::RefPred& p = P.p[c];
        p.major = col->major;
        p.residual = col->residual;
        p.w = (uint32_t)col->d.w_major;
        p.k = (uint32_t)col->d.k;
        p.layout = (uint32_t)col->d.major_layout;
        p.base = col->d.base;
        const uint32_t flip = col->d.value_signed ? 0x80000000u : 0u;
        p.lo = preds[c].lo ^ flip;   // key domain
        p.hi = preds[c].hi ^ flip;
        p.rlayout = rlayout_code(col->d);
        p.ashift = ashift;
        p.carried = in->appr_bits > 0 ? 1u : 0u;
        p.check = col->d.k > 0 ? 1u : 0u;
        ashift += p.w;
        abits += p.w;
    }
    if (in->appr_bits > 0 && (uint32_t)std::max<uint32_t>(abits, 1) != (uint32_t)in->appr_bits) {
        set_error("refine: predicates do not match the select that produced the candidates (%u vs %d bits)", abits,
                  in->appr_bits);
        return AR_ERR_INVALID;
    }
    P.npred = npred;
    P.in_pos = in->pos;
    P.in_aux = in->aux;
    P.in_count = (const long long*)in->count;
    return AR_OK;
}

ar_status ar_refine(const ar_cands* in, const ar_pred* preds, int32_t npred, ar_positions* out, void* ws,
                    size_t ws_bytes, void* stream) {
    ard::RefParams P;
    ar_status st = setup_refine(in, preds, npred, P);
    if (st != AR_OK) return st;
    if (!out || !out->pos || !out->count) {
        set_error("ar_refine: null output buffer");
        return AR_ERR_INVALID;
    }
    if (out->capacity < in->capacity) {
        set_error("ar_refine: output capacity %lld < candidate capacity %lld", (long long)out->capacity,
                  (long long)in->capacity);
        return AR_ERR_RANGE;
    }
    if (!ws || ws_bytes < ar_refine_ws_bytes(in->capacity)) {
        set_error("ar_refine: workspace %zu < %zu bytes", ws_bytes, ar_refine_ws_bytes(in->capacity));
        return AR_ERR_RANGE;
    }
    cudaStream_t s = (cudaStream_t)stream;
    AR_TRY_CUDA(cudaMemsetAsync(out->count, 0, sizeof(int64_t), s));
    const uint64_t max_tiles = ceil_div_u64((uint64_t)std::max<int64_t>(in->capacity, 0), ard::kRefTile);
    if (max_tiles == 0) return AR_OK;
    AR_TRY_CUDA(cudaMemsetAsync(ws, 0, 16 + 8 * max_tiles, s));
    P.out_pos = out->pos;
    P.out_count = (long long*)out->count;
    P.status = (unsigned long long*)((char*)ws + 16);   // [0, 16): reserved
    // persistent, round-robin tiles whose look-back waits on the tiles of other CTAs: every CTA must be
    // resident, so the grid is sized from the occupancy on this device and launch_refine launches it
    // cooperatively (a grid that cannot be co-resident fails with an error instead of hanging)
    // the wide instance when a checked predicate has an unsplit SLICED 8-plane residual (its two 16-B
    // halves gathered together, 2 CTAs per SM); the 4-CTA instance otherwise
    // and at most 8 candidate buckets (so a good share of the candidates is in the two boundary
    // buckets and needs its residual: Q6's l_shipdate has 3; C3 at 24 major bits has thousands, nearly
    // all definite, and runs faster with 4 CTAs per SM -- DESIGN s6.4)
    bool wide = false;
    for (int c = 0; c < P.npred; ++c) {
        const ard::RefPred& p = P.p[c];
        if (!p.check || p.rlayout != AR_LAYOUT_SLICED || p.k != 8) continue;
        const uint32_t blo = (p.lo - p.base) >> 8, bhi = (p.hi - p.base) >> 8;
        if (bhi >= blo && bhi - blo < 8) wide = true;
    }
    static const int wide_env = env_int("AR_REFINE_WIDE", 1);
    wide = wide && wide_env != 0;
    struct Occ { int dev; int occ[2]; };
    static thread_local Occ occ_cache[16];
    static thread_local int occ_used = 0;
    const int dev = current_device();
    int* occp = nullptr;
    for (int i = 0; i < occ_used; ++i)
        if (occ_cache[i].dev == dev) occp = occ_cache[i].occ;
    if (!occp && occ_used < 16) {
        occ_cache[occ_used] = Occ{dev, {0, 0}};
        occp = occ_cache[occ_used++].occ;
    }
    int occ = occp ? occp[wide] : 0;
    if (!occ) {
        cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, refine_kernel_fn(wide), ard::kRefThreads, 0);
        cudaGetLastError();
        occ = std::max(occ, 1);
        if (occp) occp[wide] = occ;
    }
    const int grid = (int)std::min<uint64_t>(max_tiles, (uint64_t)num_sms() * occ);
    g_last_scan = "refine_kernel";
    return launch_refine(P, grid, wide, s);
}

// ------------------------------------------------------------------ a6

static ar_status setup_aggs(const ar_column* const* cols, int32_t ncols, const ar_pred* preds, int32_t npred,
                            int64_t n, ard::AggCol* a, int32_t min_cols, bool allow_signed = false) {
    if (ncols < min_cols || ncols > AR_MAX_AGG || (ncols > 0 && !cols)) {
        set_error("sum: ncols=%d outside [%d,%d]", ncols, min_cols, AR_MAX_AGG);
        return AR_ERR_INVALID;
    }
    uint32_t bits = 0;
    for (int i = 0; i < ncols; ++i) {
        const ar_column* c = cols[i];
        if (!valid_col(c) || (n >= 0 && c->d.n != n)) {
            set_error("sum: aggregate column %d is null or has n != %lld", i, (long long)n);
            return AR_ERR_INVALID;
        }
        a[i].major = c->major;
        a[i].residual = c->residual;
        a[i].w = (uint32_t)c->d.w_major;
        a[i].k = (uint32_t)c->d.k;
        a[i].layout = (uint32_t)c->d.major_layout;
        a[i].base = c->d.base;
        a[i].rlayout = rlayout_code(c->d);
        a[i].flip = c->d.value_signed ? 0x80000000u : 0u;
        if (c->d.value_signed && !allow_signed) {
            set_error("sum: aggregate column %d is signed; the unsigned product SUM does not apply", i);
            return AR_ERR_UNSUPPORTED;
        }
        a[i].pred = -1;
        for (int p = 0; p < npred; ++p)
            if (preds[p].col == c) { a[i].pred = p; break; }
        uint32_t vb = (uint32_t)(c->d.w_major + c->d.k);
        if (c->d.base) vb = 32;   // value may use every bit
        bits += vb;
    }
    const int64_t rows = n >= 0 ? n : 1;
    uint32_t lg = 0;
    while (lg < 63 && ((int64_t)1 << lg) < rows) ++lg;
    if (ncols > 0 && bits + lg > 63) {
        set_error("sum: %u value bits + %u count bits > 63: the exact int64 sum could overflow", bits, lg);
        return AR_ERR_RANGE;
    }
    return AR_OK;
}

ar_status ar_sum(const ar_positions* pos, const ar_column* const* cols, int32_t ncols, int64_t* out_sum_dev,
                 void* stream) {
    if (!pos || !pos->pos || !pos->count || !out_sum_dev) {
        set_error("ar_sum: null argument");
        return AR_ERR_INVALID;
    }
    ard::SumParams P;
    memset(&P, 0, sizeof(P));
    const int64_t n = (cols && ncols > 0 && cols[0]) ? cols[0]->d.n : -1;
    ar_status st = setup_aggs(cols, ncols, nullptr, 0, n, P.a, 1);
    if (st != AR_OK) return st;
    P.pos = pos->pos;
    P.count = (const long long*)pos->count;
    P.nagg = ncols;
    P.out_sum = (unsigned long long*)out_sum_dev;
    cudaStream_t s = (cudaStream_t)stream;
    AR_TRY_CUDA(cudaMemsetAsync(out_sum_dev, 0, sizeof(int64_t), s));
    if (pos->capacity <= 0) return AR_OK;
    const int grid = (int)std::min<int64_t>((pos->capacity + 255) / 256, (int64_t)num_sms() * 8);
    return launch_sum(P, grid, s);
}

ar_status ar_sum_approximate(const ar_cands* in, const ar_column* const* cols, int32_t ncols, int64_t* out4_dev,
                             void* stream) {
    if (!in || !in->pos || !in->aux || !in->count || !out4_dev) {
        set_error("ar_sum_approximate: null argument");
        return AR_ERR_INVALID;
    }
    ard::ApproxSumParams P;
    memset(&P, 0, sizeof(P));
    const int64_t n = (cols && ncols > 0 && cols[0]) ? cols[0]->d.n : -1;
    ar_status st = setup_aggs(cols, ncols, nullptr, 0, n, P.a, 0);
    if (st != AR_OK) return st;
    P.pos = in->pos;
    P.aux = in->aux;
    P.count = (const long long*)in->count;
    P.nagg = ncols;
    P.out4 = (unsigned long long*)out4_dev;
    cudaStream_t s = (cudaStream_t)stream;
    AR_TRY_CUDA(cudaMemsetAsync(out4_dev, 0, 4 * sizeof(int64_t), s));
    const int grid = (int)std::max<int64_t>(1, std::min<int64_t>((std::max<int64_t>(in->capacity, 0) + 255) / 256,
                                                                 (int64_t)num_sms() * 8));
    return launch_approx_sum(P, grid, s);
}

ar_status ar_project(const ar_positions* pos, const ar_column* col, int32_t mode, uint32_t* out_values,
                     void* stream) {
    if (!pos || !pos->pos || !pos->count || !out_values || !valid_col(col) ||
        (mode != AR_PROJECT_APPROX && mode != AR_PROJECT_EXACT)) {
        set_error("ar_project: null argument or mode %d not AR_PROJECT_APPROX/EXACT", mode);
        return AR_ERR_INVALID;
    }
    ard::ProjectParams P;
    memset(&P, 0, sizeof(P));
    ar_status st = setup_aggs(&col, 1, nullptr, 0, -1, &P.a, 1, true);
    if (st != AR_OK) return st;
    P.pos = pos->pos;
    P.count = (const long long*)pos->count;
    P.exact = mode == AR_PROJECT_EXACT ? 1 : 0;
    P.out = out_values;
    if (pos->capacity <= 0) return AR_OK;
    const int grid = (int)std::min<int64_t>((pos->capacity + 255) / 256, (int64_t)num_sms() * 8);
    return launch_project(P, grid, (cudaStream_t)stream);
}

ar_status ar_refine_sum(const ar_cands* in, const ar_pred* preds, int32_t npred, const ar_column* const* cols,
                        int32_t ncols, int64_t* out_sum_dev, int64_t* out_count_dev, void* stream) {
    ard::RefParams P;
    ar_status st = setup_refine(in, preds, npred, P);
    if (st != AR_OK) return st;
    st = setup_aggs(cols, ncols, preds, npred, preds[0].col->d.n, P.a, 0);
    if (st != AR_OK) return st;
    P.nagg = ncols;
    P.out_sum = (unsigned long long*)out_sum_dev;
    P.out_cnt = (unsigned long long*)out_count_dev;
    // specialised kernel: exactly one checked predicate, SLICED residual of 4 / 8 planes, carried
    // major; factors = k = 0 carried predicate columns and at most one bit-packed gathered column
    P.fast_k = 0;
    P.fast_chk = -1;
    P.fast_g = -1;
    {
        static const int off = env_int("AR_REFINE_GENERIC", 0);
        bool ok = !off;
        int nchk = 0;
        for (int c = 0; c < P.npred; ++c) {
            const ard::RefPred& p = P.p[c];
            if (!p.check) continue;
            ++nchk;
            P.fast_chk = c;
            ok = ok && p.carried && p.rlayout == AR_LAYOUT_SLICED && (p.k == 4 || p.k == 8);
        }
        ok = ok && nchk == 1;
        for (int i = 0; i < ncols && ok; ++i) {
            const ard::AggCol& a = P.a[i];
            if (a.pred >= 0 && a.k == 0 && P.p[a.pred].carried && a.flip == 0) continue;
            if (a.pred < 0 && a.k == 0 && a.layout == AR_LAYOUT_PACKED && a.w > 0 && a.flip == 0 && P.fast_g < 0) {
                P.fast_g = i;
                continue;
            }
            ok = false;
        }
        if (ok) P.fast_k = (int32_t)P.p[P.fast_chk].k;
    }
    cudaStream_t s = (cudaStream_t)stream;
    if (out_sum_dev && out_count_dev == out_sum_dev + 1) {   // adjacent outputs: one memset node
        AR_TRY_CUDA(cudaMemsetAsync(out_sum_dev, 0, 2 * sizeof(int64_t), s));
    } else {
        if (out_sum_dev) AR_TRY_CUDA(cudaMemsetAsync(out_sum_dev, 0, sizeof(int64_t), s));
        if (out_count_dev) AR_TRY_CUDA(cudaMemsetAsync(out_count_dev, 0, sizeof(int64_t), s));
    }
    const uint64_t max_tiles = ceil_div_u64((uint64_t)std::max<int64_t>(in->capacity, 0), ard::kRefTile);
    if (max_tiles == 0) return AR_OK;
    const int grid = (int)std::min<uint64_t>(max_tiles, (uint64_t)num_sms() * 8);
    g_last_scan = P.fast_k ? "refine_sum_sliced_kernel" : "refine_sum_kernel";
    return launch_refine_sum(P, grid, s);
}

// ----------------------------------------------------------- MIN / MAX (s IV-F)

size_t ar_minmax_ws_bytes(int64_t capacity) { return 64 + 4 * (size_t)std::max<int64_t>(capacity, 0); }

ar_status ar_minmax(const ar_cands* in, const ar_pred* preds, int32_t npred, const ar_column* col, int32_t mode,
                    int64_t* out7_dev, void* ws, size_t ws_bytes, void* stream) {
    ard::MinMaxParams P;
    memset(&P, 0, sizeof(P));
    ar_status st = setup_refine(in, preds, npred, P.r);
    if (st != AR_OK) return st;
    if (!out7_dev || !ws || (mode != AR_MIN && mode != AR_MAX)) {
        set_error("ar_minmax: null output / workspace or mode %d not AR_MIN / AR_MAX", mode);
        return AR_ERR_INVALID;
    }
    if (ws_bytes < ar_minmax_ws_bytes(in->capacity)) {
        set_error("ar_minmax: workspace %zu < %zu bytes", ws_bytes, ar_minmax_ws_bytes(in->capacity));
        return AR_ERR_RANGE;
    }
    const ar_column* const cols[1] = {col};
    st = setup_aggs(cols, 1, preds, npred, preds[0].col->d.n, &P.y, 1, true);
    if (st != AR_OK) return st;
    P.mode = mode;
    P.ws = (unsigned int*)ws;
    P.wc = (unsigned long long*)((char*)ws + 32);
    P.ymaj = (uint32_t*)((char*)ws + 64);
    P.out7 = (long long*)out7_dev;
    cudaStream_t s = (cudaStream_t)stream;
    const int64_t cap = std::max<int64_t>(in->capacity, 1);
    const int grid = (int)std::min<int64_t>((cap + ard::kRefTile - 1) / ard::kRefTile, (int64_t)num_sms() * 8);
    g_last_scan = "minmax_refine_kernel";
    return launch_minmax(P, grid, s);
}

// ----------------------------------------------------------- grouped COUNT / SUM (s IV-E/F)

ar_status ar_refine_group_sum(const ar_cands* in, const ar_pred* preds, int32_t npred, const ar_column* key,
                              const ar_column* const* cols, int32_t ncols, int32_t ngroups, int64_t* out_dev,
                              void* stream) {
    ard::GroupParams P;
    memset(&P, 0, sizeof(P));
    ar_status st = setup_refine(in, preds, npred, P.r);
    if (st != AR_OK) return st;
    if (!out_dev || !valid_col(key) || ngroups < 1 || ngroups > AR_MAX_GROUPS) {
        set_error("ar_refine_group_sum: null output / key, or ngroups %d outside [1, %d]", ngroups, AR_MAX_GROUPS);
        return AR_ERR_INVALID;
    }
    const int64_t n = preds[0].col->d.n;
    if (key->d.n != n) {
        set_error("ar_refine_group_sum: key column has n != %lld", (long long)n);
        return AR_ERR_INVALID;
    }
    if (key->d.k != 0 || key->d.value_signed) {
        set_error("ar_refine_group_sum: the group key must be a GPU-resident (k = 0) unsigned column");
        return AR_ERR_UNSUPPORTED;
    }
    // every key value must be a group id: base + 2^w_major - 1 < ngroups (from the descriptor)
    const uint64_t max_key = (uint64_t)key->d.base + ((1ull << key->d.w_major) - 1ull);
    if (max_key >= (uint64_t)ngroups) {
        set_error("ar_refine_group_sum: key values up to %llu need ngroups > %llu", (unsigned long long)max_key,
                  (unsigned long long)max_key);
        return AR_ERR_RANGE;
    }
    const ar_column* const kc[1] = {key};
    st = setup_aggs(kc, 1, preds, npred, n, &P.key, 1);
    if (st != AR_OK) return st;
    st = setup_aggs(cols, ncols, preds, npred, n, P.r.a, 0);
    if (st != AR_OK) return st;
    P.r.nagg = ncols;
    P.ngroups = ngroups;
    P.out = (unsigned long long*)out_dev;
    cudaStream_t s = (cudaStream_t)stream;
    AR_TRY_CUDA(cudaMemsetAsync(out_dev, 0, 2 * sizeof(int64_t) * (size_t)ngroups, s));
    const int64_t cap = std::max<int64_t>(in->capacity, 1);
    const int grid = (int)std::min<int64_t>((cap + ard::kRefTile - 1) / ard::kRefTile, (int64_t)num_sms() * 4);
    g_last_scan = "group_sum_kernel";
    return launch_group_sum(P, grid, s);
}

ar_status ar_refine_group_sum_ids(const ar_cands* in, const ar_pred* preds, int32_t npred, const uint32_t* gids,
                                  int32_t ngroups, const ar_column* const* cols, int32_t ncols, int64_t* out_dev,
                                  void* stream) {
    ard::GroupParams P;
    memset(&P, 0, sizeof(P));
    ar_status st = setup_refine(in, preds, npred, P.r);
    if (st != AR_OK) return st;
    if (!out_dev || !gids || ngroups < 1 || ngroups > AR_MAX_GROUPS) {
        set_error("ar_refine_group_sum_ids: null output / ids, or ngroups %d outside [1, %d]", ngroups, AR_MAX_GROUPS);
        return AR_ERR_INVALID;
    }
    st = setup_aggs(cols, ncols, preds, npred, preds[0].col->d.n, P.r.a, 0);
    if (st != AR_OK) return st;
    P.r.nagg = ncols;
    P.gids = gids;
    P.ngroups = ngroups;
    P.out = (unsigned long long*)out_dev;
    cudaStream_t s = (cudaStream_t)stream;
    AR_TRY_CUDA(cudaMemsetAsync(out_dev, 0, 2 * sizeof(int64_t) * (size_t)ngroups, s));
    const int64_t cap = std::max<int64_t>(in->capacity, 1);
    const int grid = (int)std::min<int64_t>((cap + ard::kRefTile - 1) / ard::kRefTile, (int64_t)num_sms() * 4);
    g_last_scan = "group_sum_kernel";
    return launch_group_sum(P, grid, s);
}

// ----------------------------------------------------------- fused a3+a5+a6

size_t ar_select_refine_sum_ws_bytes(void) { return kSrsTicketBytes + (size_t)kSrsMaxGrid * 32; }

ar_status ar_select_refine_sum(const ar_pred* preds, int32_t npred, const ar_column* const* cols, int32_t ncols,
                               int64_t* out_dev, void* stream) {
    return ar_select_refine_sum_ws(preds, npred, cols, ncols, 0, out_dev, nullptr, 0, stream);
}

ar_status ar_select_refine_sum_ws(const ar_pred* preds, int32_t npred, const ar_column* const* cols, int32_t ncols,
                                  int32_t flags, int64_t* out_dev, void* ws, size_t ws_bytes, void* stream) {
    if (ws && ws_bytes < ar_select_refine_sum_ws_bytes()) {
        set_error("ar_select_refine_sum_ws: ws_bytes %zu < %zu", ws_bytes, ar_select_refine_sum_ws_bytes());
        return AR_ERR_RANGE;
    }
    if ((flags & ~(AR_SRS_PDL | AR_SRS_PDL_EARLY_READ)) || (flags && !ws)) {
        set_error("ar_select_refine_sum_ws: flags 0x%x invalid (the PDL flags need a workspace)", flags);
        return AR_ERR_INVALID;
    }
    ard::SelParams P;
    bool empty = false;
    int64_t n = 0;
    ar_status st = setup_scan(preds, npred, P, empty, n, true);
    if (st != AR_OK) return st;
    if (!out_dev) {
        set_error("ar_select_refine_sum: null output");
        return AR_ERR_INVALID;
    }
    st = setup_aggs(cols, ncols, preds, npred, n, P.a, 0);
    if (st != AR_OK) return st;
    P.nagg = ncols;
    P.out4 = (unsigned long long*)out_dev;
    // asynchronous gathers when exactly one aggregate column must be gathered (bit-packed, no
    // residual) and the other factor, if any, is a predicate column whose value fits 26 bits
    {
        int g = -1, ng = 0;
        bool ok = ncols >= 1;
        for (int i = 0; i < ncols; ++i) {
            const ard::AggCol& a = P.a[i];
            if (a.pred < 0) {
                ++ng;
                g = i;
                ok = ok && a.k == 0 && a.layout == AR_LAYOUT_PACKED && a.w > 0 && cols[i]->d.major_loc == AR_LOC_DEVICE;
            } else {
                ok = ok && (a.w + a.k) <= 26 && a.base == 0;
            }
        }
        static const int no_async = env_int("AR_NO_ASYNC_GATHER", 0);
        P.async_agg = (ok && ng == 1 && !no_async) ? 1 : 0;
        P.gidx = g < 0 ? 0 : g;
    }
    cudaStream_t s = (cudaStream_t)stream;
    g_last_scan = "";
    if (!ws || empty || n == 0) AR_TRY_CUDA(cudaMemsetAsync(out_dev, 0, 4 * sizeof(int64_t), s));
    if (empty || n == 0) return AR_OK;
    bool launched = false, rg = false;   // the result-ring kernels (fused.cu) where they apply
    const int pdl = (flags & AR_SRS_PDL_EARLY_READ) ? 2 : ((flags & AR_SRS_PDL) ? 1 : 0);
    st = launch_fused_rl(P, cols, ws, pdl, &launched, &rg, s);
    if (st != AR_OK) return st;
    if (launched) {
        g_last_scan = rg ? "fused_rg_kernel" : "fused_rl_kernel";
        return AR_OK;
    }
    g_last_scan = "fused_kernel";
    if (ws) AR_TRY_CUDA(cudaMemsetAsync(out_dev, 0, 4 * sizeof(int64_t), s));   // fused_kernel accumulates
    bool relay = false;   // fused_kernel gathers split residuals (it streams whole residual planes only)
    for (int c = 0; c < P.npred; ++c)
        if (P.p[c].rsplit && P.p[c].res_stream) {
            P.p[c].res_stream = 0;
            P.exact_mode = 0;
            relay = true;
        }
    if (relay) {
        const uint32_t tr = P.tile_rows;
        P.tile_rows = 0;
        retile(P, tr);
    }
    int occ = 1;
    const void* fn = select_kernel_fn(P, true);
    P.nstages = pick_stages(fn, P.stage_words, true, &occ);
    const size_t smem = select_smem_bytes(P.stage_words, P.nstages, false);
    const int grid = (int)std::min<int64_t>(P.num_tiles, (int64_t)num_sms() * occ);
    return launch_scan(fn, P, grid, smem, true, s);
}

}  // extern "C"

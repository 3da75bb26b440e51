/*
 * oracle.c -- TEST INFRASTRUCTURE ONLY.
 *
 * A plain, slow, obviously correct CPU statement of what Approximate & Refine
 * (A&R) over bitwise-distributed (BWD) columns computes, written from
 * H. Pirk, S. Manegold, M. Kersten, "Waste Not... Efficient Co-Processing of
 * Relational Data", ICDE 2014 (cited as PAPER.md:<line>, s<section>).
 *
 * Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline /
 * `--impl reference` legs may load this library.  The product path
 * (paper_conf_icde_pirkmk14_b200/) never imports, links or calls it, and this
 * file shares no code, header, table or constant with the CUDA path.
 *
 * Because A&R is exact (the approximation is a superset; the
 * refined result is correct), the oracle for the final
 * result is the plain definition over the undecomposed columns:
 *   R = [ i ascending : for all predicates c, lo_c <= v_c[i] <= hi_c ]
 *   S = sum_{i in R} prod_{c in agg} v_c[i]              (exact, int64)
 * The intermediates (decomposition, candidate / definite flags) are written
 * out from their definitions too.
 *
 * Every function is pinned by tests/test_oracle_*.py against the paper's
 * worked examples (Fig. 2, 4, 6), closed forms, and brute force.
 */
#include <stdint.h>
#include <stdlib.h>
#include <string.h>
#include <pthread.h>
#include <unistd.h>

/* ----------------------------------------------------------------- threads */

typedef void (*or_chunk_fn)(void* ctx, int t, int64_t begin, int64_t end);
typedef struct { or_chunk_fn fn; void* ctx; int t; int64_t b, e; } or_job;

static void* or_run(void* p) { or_job* j = (or_job*)p; j->fn(j->ctx, j->t, j->b, j->e); return NULL; }

int or_threads_default(void) {
    long c = sysconf(_SC_NPROCESSORS_ONLN);
    return c > 0 ? (int)c : 1;
}

#define OR_MAX_THREADS 256

/* T threads over contiguous row chunks; chunk t is [t*chunk, (t+1)*chunk). */
static int or_parallel(int64_t n, int threads, or_chunk_fn fn, void* ctx, int64_t* bounds) {
    if (threads <= 0) threads = or_threads_default();
    if (threads > OR_MAX_THREADS) threads = OR_MAX_THREADS;
    int64_t chunk = threads > 0 ? (n + threads - 1) / threads : n;
    if (chunk == 0) chunk = 1;
    pthread_t tid[OR_MAX_THREADS];
    or_job jobs[OR_MAX_THREADS];
    int started[OR_MAX_THREADS];
    for (int t = 0; t < threads; ++t) {
        int64_t b = (int64_t)t * chunk, e = b + chunk;
        if (b > n) b = n;
        if (e > n) e = n;
        bounds[2 * t] = b; bounds[2 * t + 1] = e;
        jobs[t] = (or_job){fn, ctx, t, b, e};
        started[t] = (threads > 1) && pthread_create(&tid[t], NULL, or_run, &jobs[t]) == 0;
        if (!started[t]) fn(ctx, t, b, e);
    }
    for (int t = 0; t < threads; ++t) if (started[t]) pthread_join(tid[t], NULL);
    return threads;
}

/* --------------------------------------------------------- decomposition */

/*
 * BWD decomposition, PAPER.md:143-160 (s II-A) and Fig. 2:
 * the value is split at bit granularity into major bits (the approximation)
 * and minor bits (the residual), non-redundantly; leading zeros are removed.
 * With k residual bits (k = 32 - major_bits) and prefix base b
 * (b = 0 in v1):
 *     u = v - b,   major = u >> k,   residual = u mod 2^k.
 * Returns the stored major width w_M = bit length of max(major) (the leading
 * zeros the paper removes).  Either output pointer may be NULL.
 */
int or_decompose(const uint32_t* v, int64_t n, int k, uint32_t base,
                 uint32_t* major, uint32_t* residual) {
    uint64_t two_k = (uint64_t)1 << k;               /* k in [0, 32] */
    uint64_t maxmajor = 0;
    for (int64_t i = 0; i < n; ++i) {
        uint64_t u = (uint64_t)(uint32_t)(v[i] - base);
        uint64_t m = u / two_k;
        uint64_t r = u % two_k;
        if (major) major[i] = (uint32_t)m;
        if (residual) residual[i] = (uint32_t)r;
        if (m > maxmajor) maxmajor = m;
    }
    int w = 0;
    while (w < 64 && (maxmajor >> w) != 0) ++w;
    return w;
}

/* ---------------------------------------------- approximate select flags */

/*
 * Candidate / definite flags of one predicate lo <= v <= hi evaluated on the
 * approximation alone (s IV-B; tight reading SURVEY A2/A6).
 * A major value m stands for its bucket, the 2^k exact values it can hold:
 *     bucket(m) = [ b + m*2^k , b + m*2^k + 2^k - 1 ]
 *   cand(m) <=> bucket(m) intersects [lo, hi]   (superset of the hits)
 *   def(m)  <=> bucket(m) is contained in [lo, hi]  (certain hits)
 * cand / def are byte flags (0/1), either may be NULL.
 */
void or_bucket_flags(const uint32_t* major, int64_t n, int k, uint32_t base,
                     uint32_t lo, uint32_t hi, uint8_t* cand, uint8_t* def) {
    uint64_t two_k = (uint64_t)1 << k;
    for (int64_t i = 0; i < n; ++i) {
        uint64_t first = (uint64_t)base + (uint64_t)major[i] * two_k;
        uint64_t last = first + two_k - 1;
        int c = (first <= (uint64_t)hi) && (last >= (uint64_t)lo) && (lo <= hi);
        int d = (first >= (uint64_t)lo) && (last <= (uint64_t)hi);
        if (cand) cand[i] = (uint8_t)c;
        if (def) def[i] = (uint8_t)d;
    }
}

/*
 * The relaxation function f(x) exactly as printed, with the
 * lost shift operator restored as "<<":
 *     appr(x) = x & ~((1 << resbits) - 1)
 *     '==' : appr(x)               '>=' : appr(x)
 *     '>'  : appr(x) - 1           '<=' : appr(x) + (1 << resbits)
 *     '<'  : appr(x) + (1 << resbits) + 1
 * and the scan keeps the operator: flag = appr(v) op f(x).  Used by tests only,
 * to check printed-f candidates contain the tight candidates.
 * op: 0 '==', 1 '>', 2 '>=', 3 '<', 4 '<='.
 */
void or_paper_f_flags(const uint32_t* v, int64_t n, int k, int op, uint32_t x, uint8_t* flag) {
    int64_t two_k = (int64_t)1 << k;
    int64_t ax = (int64_t)((uint64_t)x & ~(uint64_t)(two_k - 1));
    int64_t fx;
    switch (op) {
        case 0: fx = ax; break;
        case 1: fx = ax - 1; break;
        case 2: fx = ax; break;
        case 3: fx = ax + two_k + 1; break;
        default: fx = ax + two_k; break;
    }
    for (int64_t i = 0; i < n; ++i) {
        int64_t av = (int64_t)((uint64_t)v[i] & ~(uint64_t)(two_k - 1));
        int f;
        switch (op) {
            case 0: f = av == fx; break;
            case 1: f = av > fx; break;
            case 2: f = av >= fx; break;
            case 3: f = av < fx; break;
            default: f = av <= fx; break;
        }
        flag[i] = (uint8_t)f;
    }
}

/* ------------------------------------------------ exact select and SUM */

typedef struct {
    int npred;
    const uint32_t* const* pcols;
    const uint32_t* lo;
    const uint32_t* hi;
    const int* sgn;              /* per predicate: 1 = int32 column (NULL: all uint32) */
    int nagg;
    const uint32_t* const* acols;
    int64_t* out_pos;            /* may be NULL                      */
    int64_t count[OR_MAX_THREADS];
    __int128 sum[OR_MAX_THREADS];
    int64_t* bounds;
    int pass;                    /* 0: count+sum, 1: write positions */
    int64_t offset[OR_MAX_THREADS];
} sel_ctx;

static int row_qualifies(const sel_ctx* c, int64_t i) {
    for (int p = 0; p < c->npred; ++p) {
        if (c->sgn && c->sgn[p]) {          /* signed column: compare as int32 */
            int32_t v = (int32_t)c->pcols[p][i], lo = (int32_t)c->lo[p], hi = (int32_t)c->hi[p];
            if (!(lo <= v && v <= hi)) return 0;
        } else {
            uint32_t v = c->pcols[p][i];
            if (!(c->lo[p] <= v && v <= c->hi[p])) return 0;
        }
    }
    return 1;
}

static void sel_chunk(void* p, int t, int64_t b, int64_t e) {
    sel_ctx* c = (sel_ctx*)p;
    if (c->pass == 0) {
        int64_t cnt = 0;
        __int128 s = 0;
        for (int64_t i = b; i < e; ++i) {
            if (!row_qualifies(c, i)) continue;
            ++cnt;
            if (c->nagg > 0) {
                __int128 prod = 1;
                for (int a = 0; a < c->nagg; ++a) prod *= (__int128)c->acols[a][i];
                s += prod;
            }
        }
        c->count[t] = cnt;
        c->sum[t] = s;
    } else {
        int64_t o = c->offset[t];
        for (int64_t i = b; i < e; ++i)
            if (row_qualifies(c, i)) c->out_pos[o++] = i;
    }
}

/*
 * Exact conjunctive range select + product SUM over the full-precision
 * columns: the plain definition the A&R plan must reproduce (Fig. 3 / Fig. 7,
 * PAPER.md:333-359, 879-893; Q6 shape PAPER.md:1291-1309).
 *   out_pos (optional): ascending positions of qualifying rows
 *   *out_count       : |R|
 *   *out_sum         : sum over R of prod_a acols[a][i]  (0 if nagg == 0)
 * sgn (optional): sgn[p] = 1 compares predicate p's column and bounds as int32
 * (the spatial query of Table I has signed longitudes).
 * Rows are split over `threads` contiguous chunks and chunk results are
 * concatenated / added in chunk order, so the result does not depend on T.
 * Returns 0, or 1 if the exact sum does not fit in int64.
 */
int or_select_sum(int64_t n, int npred, const uint32_t* const* pcols,
                  const uint32_t* lo, const uint32_t* hi, const int* sgn,
                  int nagg, const uint32_t* const* acols,
                  int64_t* out_pos, int64_t* out_count, int64_t* out_sum, int threads) {
    sel_ctx* c = (sel_ctx*)calloc(1, sizeof(sel_ctx));
    int64_t bounds[2 * OR_MAX_THREADS];
    c->npred = npred; c->pcols = pcols; c->lo = lo; c->hi = hi; c->sgn = sgn;
    c->nagg = nagg; c->acols = acols; c->out_pos = out_pos; c->bounds = bounds;
    c->pass = 0;
    int T = or_parallel(n, threads, sel_chunk, c, bounds);
    int64_t total = 0;
    __int128 s = 0;
    for (int t = 0; t < T; ++t) { c->offset[t] = total; total += c->count[t]; s += c->sum[t]; }
    if (out_pos) { c->pass = 1; or_parallel(n, T, sel_chunk, c, bounds); }
    if (out_count) *out_count = total;
    int overflow = (s > (__int128)INT64_MAX) || (s < (__int128)INT64_MIN);
    if (out_sum) *out_sum = (int64_t)s;
    free(c);
    return overflow;
}

/* Product SUM over given positions (SUM(refine) of Fig. 3/7), exact; returns 1 on int64 overflow. */
int or_sum_at(const int64_t* pos, int64_t npos, int nagg, const uint32_t* const* acols, int64_t* out_sum) {
    __int128 s = 0;
    for (int64_t j = 0; j < npos; ++j) {
        __int128 prod = 1;
        for (int a = 0; a < nagg; ++a) prod *= (__int128)acols[a][pos[j]];
        s += prod;
    }
    *out_sum = (int64_t)s;
    return (s > (__int128)INT64_MAX) || (s < (__int128)INT64_MIN);
}

/* ------------------------------------------- approximate answer (bounds) */

/*
 * bwd.sumapproximate (Fig. 7): the answer of the
 * approximation subplan alone, available before any residual is read
 * (PAPER.md:360-362, 894-897), given as strict error bounds.
 * Each value v of a column decomposed with k residual bits and base b is only
 * known to lie in its bucket  [b + m 2^k, b + m 2^k + 2^k - 1],  m = (v - b) >> k
 * (the upper end clamped to 2^32 - 1).  From the candidate / definite rows of
 * the conjunction (or_bucket_flags), since definite <= R <= cand:
 *   out[0] = sum over definite rows of prod_a min(bucket_a)     (<= SUM over R)
 *   out[1] = sum over candidate rows of prod_a max(bucket_a)    (>= SUM over R)
 *   out[2] = |definite|,  out[3] = |candidates|
 * pks/pbase: k and base of each predicate column; aks/abase: of each aggregate.
 * psgn (optional, NULL = all unsigned): psgn[p] = 1 marks an int32 predicate
 * column; its values and bounds are compared in the order-preserving key
 * domain d = v ^ 2^31 (DESIGN R8), in which its base and buckets
 * are defined.  Aggregate factors are unsigned (the ABI's product SUM).
 * Returns 1 if a bound does not fit in int64.
 */
int or_sum_bounds(int64_t n, int npred, const uint32_t* const* pcols, const int* pks, const uint32_t* pbase,
                  const uint32_t* lo, const uint32_t* hi, const int* psgn, int nagg, const uint32_t* const* acols,
                  const int* aks, const uint32_t* abase, int64_t* out) {
    __int128 slo = 0, shi = 0;
    int64_t ndef = 0, ncand = 0;
    for (int64_t i = 0; i < n; ++i) {
        int cand = 1, def = 1;
        for (int p = 0; p < npred; ++p) {
            uint32_t flip = (psgn && psgn[p]) ? 0x80000000u : 0u;
            uint32_t d = pcols[p][i] ^ flip, dlo = lo[p] ^ flip, dhi = hi[p] ^ flip;
            uint64_t two_k = (uint64_t)1 << pks[p];
            uint64_t m = (uint64_t)(uint32_t)(d - pbase[p]) / two_k;
            uint64_t first = (uint64_t)pbase[p] + m * two_k;
            uint64_t last = first + two_k - 1;
            if (!(dlo <= dhi && first <= dhi && last >= dlo)) cand = 0;
            if (!(first >= dlo && last <= dhi)) def = 0;
        }
        if (!cand) continue;
        ++ncand;
        if (def) ++ndef;
        if (nagg == 0) continue;
        __int128 plo = 1, phi = 1;
        for (int a = 0; a < nagg; ++a) {
            uint64_t two_k = (uint64_t)1 << aks[a];
            uint64_t m = (uint64_t)(uint32_t)(acols[a][i] - abase[a]) / two_k;
            uint64_t first = (uint64_t)abase[a] + m * two_k;
            uint64_t last = first + two_k - 1;
            if (last > 0xffffffffull) last = 0xffffffffull;
            plo *= first;
            phi *= last;
        }
        shi += phi;
        if (def) slo += plo;
    }
    out[0] = (int64_t)slo;
    out[1] = (int64_t)shi;
    out[2] = ndef;
    out[3] = ncand;
    return shi > (__int128)INT64_MAX;
}

/* -------------------------------------------------------- MIN / MAX (Fig. 6) */

/*
 * Exact  select min(Y) / max(Y) from R where <conjunction>: the plain
 * definition (s IV-F).  mode 0 = MIN, 1 = MAX.  ysgn = 1
 * compares Y as int32.  out[0] = the aggregate (as int64; 0 when R is empty),
 * out[1] = |R|.
 */
void or_select_minmax(int64_t n, int npred, const uint32_t* const* pcols, const uint32_t* lo, const uint32_t* hi,
                      const int* sgn, const uint32_t* ycol, int ysgn, int mode, int64_t* out) {
    sel_ctx c;
    memset(&c, 0, sizeof(c));
    c.npred = npred; c.pcols = pcols; c.lo = lo; c.hi = hi; c.sgn = sgn;
    int64_t count = 0, best = 0;
    for (int64_t i = 0; i < n; ++i) {
        if (!row_qualifies(&c, i)) continue;
        int64_t v = ysgn ? (int64_t)(int32_t)ycol[i] : (int64_t)ycol[i];
        if (count == 0 || (mode == 0 ? v < best : v > best)) best = v;
        ++count;
    }
    out[0] = count ? best : 0;
    out[1] = count;
}

/*
 * A&R MIN / MAX, step by step as s IV-F describes it:
 *  1. approximate selection: candidate / definite rows of the conjunction by
 *     the bucket definition (or_bucket_flags);
 *  2. "the error bounds of the applied selections are propagated to the
 *     aggregation": with Y's majors m (key u = v ^ flip - b, m = u >> ky), a
 *     definite row is certainly in R, so for MIN the true minimum is at most
 *     the top of the bucket of the smallest definite major mD; every row whose
 *     major exceeds mD is larger than that definite row and cannot be the
 *     minimum.  The approximation of the minimum is therefore the set of
 *     candidates with m <= mD (all candidates when no row is definite), which
 *     "assuredly include[s] the tuple ID of the actual minimum" -- not merely
 *     the rows with the minimal approximation, which may be a false positive
 *     (Fig. 6).  MAX mirrors it (m >= the largest definite major MD).
 *     Approximate answer before refinement (bucket ends, key domain):
 *       MIN in [bmin(min_C m), D ? bmax(mD) : bmax(max_C m)]
 *       MAX in [D ? bmin(MD) : bmin(min_C m), bmax(max_C m)]
 *  3. refinement: "a join of the candidate set with the input residuals and
 *     the calculation of the minimum": the exact predicates
 *     and the exact Y on the set of step 2.
 * pks / pbase: k and base of each predicate column; ky / ybase: of Y.  psgn
 * (optional, NULL = all unsigned): psgn[p] = 1 marks an int32 predicate column,
 * compared -- approximately and exactly -- in the key domain d = v ^ 2^31
 * (DESIGN R8), in which its base and buckets are defined.  Bounds
 * and the result are values (int32 when ysgn).  out[0] = refined aggregate
 * (0 if no refined row survives), out[1] = survivors of the refinement (>= 1
 * iff R is not empty), out[2] / out[3] = approximate lower / upper bound
 * (0 / 0 when there is no candidate), out[4] = rows refined (|set of step 2|),
 * out[5] = |D|, out[6] = |C|.  refine_flag (optional, n bytes) marks the rows
 * of step 2.
 */
void or_minmax_ar(int64_t n, int npred, const uint32_t* const* pcols, const int* pks, const uint32_t* pbase,
                  const uint32_t* lo, const uint32_t* hi, const int* psgn, const uint32_t* ycol, int ky,
                  uint32_t ybase, int ysgn, int mode, int64_t* out, uint8_t* refine_flag) {
    uint32_t flip = ysgn ? 0x80000000u : 0u;
    uint64_t two_ky = (uint64_t)1 << ky;
    uint8_t* cand = (uint8_t*)calloc((size_t)(n > 0 ? n : 1), 1);
    uint8_t* def = (uint8_t*)calloc((size_t)(n > 0 ? n : 1), 1);
    /* 1. approximate selection */
    for (int64_t i = 0; i < n; ++i) {
        int c = 1, d = 1;
        for (int p = 0; p < npred; ++p) {
            uint32_t pf = (psgn && psgn[p]) ? 0x80000000u : 0u;
            uint32_t key = pcols[p][i] ^ pf, klo = lo[p] ^ pf, khi = hi[p] ^ pf;
            uint64_t two_k = (uint64_t)1 << pks[p];
            uint64_t m = (uint64_t)(uint32_t)(key - pbase[p]) / two_k;
            uint64_t first = (uint64_t)pbase[p] + m * two_k;
            uint64_t last = first + two_k - 1;
            if (!(klo <= khi && first <= khi && last >= klo)) c = 0;
            if (!(first >= klo && last <= khi)) d = 0;
        }
        cand[i] = (uint8_t)c;
        def[i] = (uint8_t)(c && d);
    }
    /* 2. propagate the selection's error bounds to the aggregation */
    int64_t nc = 0, nd = 0;
    uint64_t minC = 0, maxC = 0, minD = 0, maxD = 0;
    for (int64_t i = 0; i < n; ++i) {
        if (!cand[i]) continue;
        uint64_t m = (uint64_t)((ycol[i] ^ flip) - ybase) / two_ky;
        if (nc == 0 || m < minC) minC = m;
        if (nc == 0 || m > maxC) maxC = m;
        ++nc;
        if (def[i]) {
            if (nd == 0 || m < minD) minD = m;
            if (nd == 0 || m > maxD) maxD = m;
            ++nd;
        }
    }
    int64_t nref = 0, surv = 0, best = 0;
    int64_t blo = 0, bhi = 0;
    if (nc > 0) {
        uint64_t mlo = mode == 0 ? minC : (nd ? maxD : minC);   /* bucket whose bottom bounds the answer */
        uint64_t mhi = mode == 0 ? (nd ? minD : maxC) : maxC;   /* bucket whose top bounds the answer */
        uint64_t klo = (uint64_t)ybase + mlo * two_ky;
        uint64_t khi = (uint64_t)ybase + mhi * two_ky + two_ky - 1;
        if (khi > 0xffffffffull) khi = 0xffffffffull;
        uint32_t vlo = (uint32_t)klo ^ flip, vhi = (uint32_t)khi ^ flip;
        blo = ysgn ? (int64_t)(int32_t)vlo : (int64_t)vlo;
        bhi = ysgn ? (int64_t)(int32_t)vhi : (int64_t)vhi;
        /* 3. refine the rows that can hold the answer */
        uint64_t thr = mode == 0 ? (nd ? minD : maxC) : (nd ? maxD : minC);
        for (int64_t i = 0; i < n; ++i) {
            if (refine_flag) refine_flag[i] = 0;
            if (!cand[i]) continue;
            uint64_t m = (uint64_t)((ycol[i] ^ flip) - ybase) / two_ky;
            if (mode == 0 ? m > thr : m < thr) continue;
            if (refine_flag) refine_flag[i] = 1;
            ++nref;
            int ok = 1;
            for (int p = 0; p < npred; ++p) {
                uint32_t pf = (psgn && psgn[p]) ? 0x80000000u : 0u;
                uint32_t key = pcols[p][i] ^ pf;
                if (!((lo[p] ^ pf) <= key && key <= (hi[p] ^ pf))) ok = 0;
            }
            if (!ok) continue;
            int64_t v = ysgn ? (int64_t)(int32_t)ycol[i] : (int64_t)ycol[i];
            if (surv == 0 || (mode == 0 ? v < best : v > best)) best = v;
            ++surv;
        }
    } else if (refine_flag) {
        memset(refine_flag, 0, (size_t)n);
    }
    out[0] = surv ? best : 0;
    out[1] = surv;
    out[2] = blo;
    out[3] = bhi;
    out[4] = nref;
    out[5] = nd;
    out[6] = nc;
    free(cand);
    free(def);
}

/* ---------------------------------------------------- grouped SUM (s IV-E) */

/*
 * Exact  select key, count(*), sum(prod_a acols[a]) from R where <conjunction>
 * group by key  -- the plain definition of a grouped aggregation over the
 * selection (s IV-E/F; Fig. 4 "select count(*) from R where
 * A<5 groupby B").  Keys are small non-negative integers
 * (group id = key value, key < ngroups).  out_cnt[g] = rows of R with key g,
 * out_sum[g] = their product sum (0 if nagg == 0).  Returns 0, 1 on int64
 * overflow, 2 if a qualifying row has key >= ngroups.
 */
int or_select_group_sum(int64_t n, int npred, const uint32_t* const* pcols, const uint32_t* lo,
                        const uint32_t* hi, const uint32_t* key, int ngroups, int nagg,
                        const uint32_t* const* acols, int64_t* out_sum, int64_t* out_cnt) {
    sel_ctx c;
    memset(&c, 0, sizeof(c));
    c.npred = npred; c.pcols = pcols; c.lo = lo; c.hi = hi;
    __int128* s = (__int128*)calloc((size_t)(ngroups > 0 ? ngroups : 1), sizeof(__int128));
    for (int g = 0; g < ngroups; ++g) out_cnt[g] = 0;
    int rc = 0;
    for (int64_t i = 0; i < n; ++i) {
        if (!row_qualifies(&c, i)) continue;
        uint32_t g = key[i];
        if (g >= (uint32_t)ngroups) { rc = 2; break; }
        out_cnt[g] += 1;
        __int128 prod = 1;
        for (int a = 0; a < nagg; ++a) prod *= (__int128)acols[a][i];
        if (nagg > 0) s[g] += prod;
    }
    for (int g = 0; g < ngroups; ++g) {
        if (s[g] > (__int128)INT64_MAX) rc = rc ? rc : 1;
        out_sum[g] = (int64_t)s[g];
    }
    free(s);
    return rc;
}

/*
 * Exact  select key, count(*), sum(prod_a acols[a]) from R where <conjunction>
 * group by key  for ARBITRARY uint32 key values -- the plain definition of a
 * grouped aggregation (s IV-E/F), with the groups listed in
 * ascending key order.  Written plainly: the keys of the qualifying rows are
 * collected and sorted (qsort), duplicates dropped; each qualifying row then
 * finds its group by binary search and adds to it.  out_key / out_cnt /
 * out_sum have room for max_groups entries; *ngroups = number of distinct keys
 * among the qualifying rows.  Returns 0, 1 on int64 overflow of a sum, 2 if
 * there are more than max_groups groups (outputs then hold the first max_groups).
 */
static int or_cmp_u32(const void* a, const void* b) {
    uint32_t x = *(const uint32_t*)a, y = *(const uint32_t*)b;
    return x < y ? -1 : (x > y ? 1 : 0);
}

int or_select_group_sum_keys(int64_t n, int npred, const uint32_t* const* pcols, const uint32_t* lo,
                             const uint32_t* hi, const int* sgn, const uint32_t* key, int nagg,
                             const uint32_t* const* acols, int64_t max_groups, uint32_t* out_key,
                             int64_t* out_cnt, int64_t* out_sum, int64_t* ngroups) {
    sel_ctx c;
    memset(&c, 0, sizeof(c));
    c.npred = npred; c.pcols = pcols; c.lo = lo; c.hi = hi; c.sgn = sgn;
    uint32_t* keys = (uint32_t*)malloc((size_t)(n > 0 ? n : 1) * sizeof(uint32_t));
    int64_t m = 0;
    for (int64_t i = 0; i < n; ++i)
        if (row_qualifies(&c, i)) keys[m++] = key[i];
    qsort(keys, (size_t)m, sizeof(uint32_t), or_cmp_u32);
    int64_t g = 0;
    for (int64_t i = 0; i < m; ++i)
        if (i == 0 || keys[i] != keys[i - 1]) keys[g++] = keys[i];
    *ngroups = g;
    __int128* s = (__int128*)calloc((size_t)(g > 0 ? g : 1), sizeof(__int128));
    int64_t* cnt = (int64_t*)calloc((size_t)(g > 0 ? g : 1), sizeof(int64_t));
    for (int64_t i = 0; i < n; ++i) {
        if (!row_qualifies(&c, i)) continue;
        int64_t a = 0, b = g - 1;          /* binary search: keys[a..b] holds key[i] */
        while (a < b) {
            int64_t mid = a + (b - a) / 2;
            if (keys[mid] < key[i]) a = mid + 1; else b = mid;
        }
        cnt[a] += 1;
        __int128 prod = 1;
        for (int q = 0; q < nagg; ++q) prod *= (__int128)acols[q][i];
        if (nagg > 0) s[a] += prod;
    }
    int rc = 0;
    for (int64_t j = 0; j < g; ++j) {
        if (s[j] > (__int128)INT64_MAX) rc = 1;
        if (j < max_groups) {
            out_key[j] = keys[j];
            out_cnt[j] = cnt[j];
            out_sum[j] = (int64_t)s[j];
        }
    }
    if (g > max_groups) rc = 2;
    free(keys); free(s); free(cnt);
    return rc;
}

/*
 * datagen.c -- seeded, counter-based synthetic inputs shared by the oracle side
 * and the CUDA side.  This module holds NONE of the A&R / BWD arithmetic
 * (no decomposition, no relaxation, no predicate, no aggregate): it only
 * produces the columns the paper's workloads are made of, so that both sides
 * can be fed the same bytes.
 *
 * Generator: splitmix64 (Steele, Lea, Flood 2014).  Row i of stream s under
 * seed S is   mix(key(S,s) + (i+1)*GAMMA),   i.e. the i-th output of the
 * splitmix64 sequence seeded with key(S,s).  Because it is counter-based, any
 * row range [row0, row0+n) of any table can be regenerated independently,
 * which is what lets every rank of a row-sharded run build only its own shard.
 *
 * A uniform integer in [lo, hi] (span = hi-lo+1 <= 2^32) is
 *   lo + (((r >> 32) * span) >> 32)
 * (multiply-shift; deterministic, slightly biased for spans that are not
 * powers of two, which does not matter for synthetic data).
 *
 * Workload recipes:
 *  - uniform u32 column                                (configs C1, C3-A)
 *  - keyed bijection of [0, N): unique shuffled ints    (config C3-B; the
 *    paper's micro-benchmarks use "100 million unique, randomly shuffled
 *    integers (value range 0 to 100 million)", s VI-B)
 *  - TPC-H-lineitem-shaped Q6 columns                   (configs C2, C4, C5;
 *    value domains from PAPER.md:1294-1299, s VI-D-1: l_quantity 50 values /
 *    6 bits, l_discount 4 bits, l_shipdate 2526 values / 12 bits)
 *  - GPS-fix-shaped (lon, lat) pairs                     (config C6, the
 *    spatial range query of Table I, s VI-C: ~250 M
 *    fixes from navigation devices, decimal(8,5)/(7,5) degrees, lat
 *    27.09371..70.13643, lon -12.62427..29.64975)
 */
#include <stdint.h>
#include <stdlib.h>
#include <pthread.h>
#include <unistd.h>

#define GAMMA 0x9E3779B97F4A7C15ull

static inline uint64_t mix64(uint64_t z) {
    z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
    z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
    return z ^ (z >> 31);
}

uint64_t dg_key(uint64_t seed, uint32_t stream) {
    return mix64(seed * GAMMA + (uint64_t)stream * 0xD1B54A32D192ED03ull + 1ull);
}

static inline uint64_t draw(uint64_t key, uint64_t row) {
    return mix64(key + (row + 1ull) * GAMMA);
}

static inline uint32_t uniform_span(uint64_t r, uint64_t span) {
    return (uint32_t)(((r >> 32) * span) >> 32);
}

/* ---------------------------------------------------------------- threads */

typedef void (*chunk_fn)(void* ctx, int64_t begin, int64_t end);
typedef struct { chunk_fn fn; void* ctx; int64_t b, e; } job_t;

static void* run_job(void* p) { job_t* j = (job_t*)p; j->fn(j->ctx, j->b, j->e); return NULL; }

int dg_threads_default(void) {
    long c = sysconf(_SC_NPROCESSORS_ONLN);
    return c > 0 ? (int)c : 1;
}

static void parallel_for(int64_t n, int threads, chunk_fn fn, void* ctx) {
    if (threads <= 0) threads = dg_threads_default();
    if (threads > 256) threads = 256;
    if (n < 65536 || threads == 1) { fn(ctx, 0, n); return; }
    pthread_t tid[256]; job_t jobs[256];
    int64_t chunk = (n + threads - 1) / threads;
    int used = 0;
    for (int t = 0; t < threads; ++t) {
        int64_t b = (int64_t)t * chunk, e = b + chunk;
        if (b >= n) break;
        if (e > n) e = n;
        jobs[t] = (job_t){fn, ctx, b, e};
        if (pthread_create(&tid[t], NULL, run_job, &jobs[t]) != 0) { fn(ctx, b, e); jobs[t].fn = NULL; }
        used = t + 1;
    }
    for (int t = 0; t < used; ++t) if (jobs[t].fn) pthread_join(tid[t], NULL);
}

/* ------------------------------------------------------------ uniform u32 */

typedef struct { uint64_t key, row0, span; uint32_t lo; uint32_t* out; } uni_ctx;

static void uni_chunk(void* p, int64_t b, int64_t e) {
    uni_ctx* c = (uni_ctx*)p;
    for (int64_t i = b; i < e; ++i)
        c->out[i] = c->lo + uniform_span(draw(c->key, c->row0 + (uint64_t)i), c->span);
}

/* out[i] = U[lo, hi] for table rows row0 .. row0+n-1 of stream `stream`. */
void dg_uniform_u32(uint64_t seed, uint32_t stream, uint64_t row0, int64_t n,
                    uint32_t lo, uint32_t hi, uint32_t* out, int threads) {
    uni_ctx c = {dg_key(seed, stream), row0, (uint64_t)hi - lo + 1ull, lo, out};
    parallel_for(n, threads, uni_chunk, &c);
}

/* -------------------------------------------------------- keyed bijection */

typedef struct { uint64_t key, row0, N; int half; uint32_t* out; } bij_ctx;

static inline uint64_t feistel(uint64_t x, uint64_t key, int half) {
    uint64_t mask = (half >= 32) ? 0xFFFFFFFFull : ((1ull << half) - 1ull);
    uint64_t L = (x >> half) & mask, R = x & mask;
    for (int r = 0; r < 4; ++r) {
        uint64_t F = mix64(key + (uint64_t)r * GAMMA + R) & mask;
        uint64_t nl = R;
        R = L ^ F;
        L = nl;
    }
    return (L << half) | R;
}

static void bij_chunk(void* p, int64_t b, int64_t e) {
    bij_ctx* c = (bij_ctx*)p;
    for (int64_t i = b; i < e; ++i) {
        uint64_t x = c->row0 + (uint64_t)i;
        do { x = feistel(x, c->key, c->half); } while (x >= c->N); /* cycle walking */
        c->out[i] = (uint32_t)x;
    }
}

/* out[i] = perm(row0+i), perm a keyed bijection of [0, N), N <= 2^32. */
void dg_bijection_u32(uint64_t seed, uint32_t stream, uint64_t N, uint64_t row0, int64_t n,
                      uint32_t* out, int threads) {
    int bits = 2;
    while (bits < 64 && (1ull << bits) < N) bits += 2;
    bij_ctx c = {dg_key(seed, stream), row0, N, bits / 2, out};
    parallel_for(n, threads, bij_chunk, &c);
}

/* ----------------------------------------------------------- Q6 lineitem */

enum { S_ORDERDATE = 0, S_SHIPDELAY = 1, S_QUANTITY = 2, S_DISCOUNT = 3, S_PARTKEY = 4 };

typedef struct {
    uint64_t k_od, k_sd, k_q, k_d, k_pk, row0, n_parts;
    uint32_t *shipdate, *discount, *quantity, *extprice;
} q6_ctx;

/* TPC-H retail price of part pk in cents (TPC-H spec 4.2.3, [ext]). */
static inline uint32_t retail_cents(uint64_t pk) {
    return (uint32_t)(90000ull + ((pk / 10ull) % 20001ull) + 100ull * (pk % 1000ull));
}

static void q6_chunk(void* p, int64_t b, int64_t e) {
    q6_ctx* c = (q6_ctx*)p;
    for (int64_t i = b; i < e; ++i) {
        uint64_t row = c->row0 + (uint64_t)i;
        uint32_t od = uniform_span(draw(c->k_od, row), 2406);          /* U[0,2405]   */
        uint32_t sd = 1u + uniform_span(draw(c->k_sd, row), 121);      /* U[1,121]    */
        uint32_t q  = 1u + uniform_span(draw(c->k_q, row), 50);        /* U[1,50]     */
        uint32_t d  = uniform_span(draw(c->k_d, row), 11);             /* U[0,10]     */
        uint64_t pk = 1ull + uniform_span(draw(c->k_pk, row), c->n_parts); /* U[1,P]   */
        if (c->shipdate) c->shipdate[i] = od + sd;       /* days since 1992-01-01: 1..2526 */
        if (c->discount) c->discount[i] = d;             /* hundredths                     */
        if (c->quantity) c->quantity[i] = q;
        if (c->extprice) c->extprice[i] = q * retail_cents(pk); /* cents, < 2^24          */
    }
}

/*
 * Lineitem-shaped columns for table rows row0 .. row0+n-1 of a table whose
 * part table has n_parts = 200000*SF rows.  Any output pointer may be NULL.
 */
void dg_q6(uint64_t seed, uint64_t n_parts, uint64_t row0, int64_t n,
           uint32_t* shipdate, uint32_t* discount, uint32_t* quantity, uint32_t* extprice,
           int threads) {
    q6_ctx c = {dg_key(seed, S_ORDERDATE), dg_key(seed, S_SHIPDELAY), dg_key(seed, S_QUANTITY),
                dg_key(seed, S_DISCOUNT), dg_key(seed, S_PARTKEY), row0, n_parts,
                shipdate, discount, quantity, extprice};
    parallel_for(n, threads, q6_chunk, &c);
}

/* ------------------------------------------------------------ spatial C6 */

/*
 * GPS fixes as int32 in 1e-5 degree units (decimal(8,5) / decimal(7,5) scaled),
 * inside the paper's bounding box.  Fixes come in trips of
 * SP_TRIP consecutive rows: trip t starts near one of SP_CITIES city centres
 * (city = floor(SP_CITIES * u^2): a skewed, Zipf-like popularity; city 0 sits
 * at the centre of Table I's query box), offset by a
 * triangular U[-R,R] + U[-R,R] displacement, and moves by a constant per-fix
 * step (dx, dy) in U[-SP_STEP, SP_STEP]^2 with U[-SP_JIT, SP_JIT] jitter on
 * every fix.  Coordinates are clamped to the bounding box.  Row-addressable
 * (counter-based), so every shard regenerates its own rows.
 */
#define SP_LON_MIN (-1262427)
#define SP_LON_MAX 2964975
#define SP_LAT_MIN 2709371
#define SP_LAT_MAX 7013643
#define SP_TRIP 128
#define SP_CITIES 32
#define SP_R 10000
#define SP_STEP 30
#define SP_JIT 3
#define SP_BOX_LON 269258   /* centre of lon BETWEEN 2.68288 AND 2.70228 */
#define SP_BOX_LAT 5043535  /* centre of lat BETWEEN 50.4222 AND 50.4485  */

enum { S_CITY_LON = 10, S_CITY_LAT = 11, S_TRIP_CITY = 12, S_TRIP_DLON = 13, S_TRIP_DLAT = 14,
       S_TRIP_SLON = 15, S_TRIP_SLAT = 16, S_FIX_JLON = 17, S_FIX_JLAT = 18, S_TRIP_DLON2 = 19, S_TRIP_DLAT2 = 20 };

typedef struct { uint64_t seed, row0; int32_t *lon, *lat; } sp_ctx;

static inline int64_t sp_uni(uint64_t seed, uint32_t stream, uint64_t row, int64_t lo, int64_t hi) {
    return lo + (int64_t)uniform_span(draw(dg_key(seed, stream), row), (uint64_t)(hi - lo + 1));
}

static inline int64_t sp_clamp(int64_t x, int64_t lo, int64_t hi) { return x < lo ? lo : (x > hi ? hi : x); }

static void sp_chunk(void* p, int64_t b, int64_t e) {
    sp_ctx* c = (sp_ctx*)p;
    for (int64_t i = b; i < e; ++i) {
        uint64_t row = c->row0 + (uint64_t)i, trip = row / SP_TRIP, j = row % SP_TRIP;
        uint64_t u = (uint64_t)uniform_span(draw(dg_key(c->seed, S_TRIP_CITY), trip), 1ull << 16);
        uint64_t city = (SP_CITIES * u * u) >> 32;                       /* floor(C * (u/2^16)^2) */
        int64_t clon = city == 0 ? SP_BOX_LON : sp_uni(c->seed, S_CITY_LON, city, SP_LON_MIN, SP_LON_MAX);
        int64_t clat = city == 0 ? SP_BOX_LAT : sp_uni(c->seed, S_CITY_LAT, city, SP_LAT_MIN, SP_LAT_MAX);
        int64_t slon = clon + sp_uni(c->seed, S_TRIP_DLON, trip, -SP_R, SP_R) + sp_uni(c->seed, S_TRIP_DLON2, trip, -SP_R, SP_R);
        int64_t slat = clat + sp_uni(c->seed, S_TRIP_DLAT, trip, -SP_R, SP_R) + sp_uni(c->seed, S_TRIP_DLAT2, trip, -SP_R, SP_R);
        int64_t dx = sp_uni(c->seed, S_TRIP_SLON, trip, -SP_STEP, SP_STEP);
        int64_t dy = sp_uni(c->seed, S_TRIP_SLAT, trip, -SP_STEP, SP_STEP);
        int64_t lon = slon + (int64_t)j * dx + sp_uni(c->seed, S_FIX_JLON, row, -SP_JIT, SP_JIT);
        int64_t lat = slat + (int64_t)j * dy + sp_uni(c->seed, S_FIX_JLAT, row, -SP_JIT, SP_JIT);
        if (c->lon) c->lon[i] = (int32_t)sp_clamp(lon, SP_LON_MIN, SP_LON_MAX);
        if (c->lat) c->lat[i] = (int32_t)sp_clamp(lat, SP_LAT_MIN, SP_LAT_MAX);
    }
}

/* GPS-fix columns (int32, 1e-5 degrees) for rows row0 .. row0+n-1; either output may be NULL. */
void dg_spatial(uint64_t seed, uint64_t row0, int64_t n, int32_t* lon, int32_t* lat, int threads) {
    sp_ctx c = {seed, row0, lon, lat};
    parallel_for(n, threads, sp_chunk, &c);
}

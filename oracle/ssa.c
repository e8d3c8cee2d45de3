/*
 * ORACLE — test infrastructure only.  Plain, slow, obviously-correct CPU reference of the
 * CWC ensemble-SSA hot path.  Only tests/, __graft_entry__.smoke() and bench.py's
 * cpu_baseline / --impl reference legs may load this library.  It shares no code, header,
 * table or constant generator with the product (paper_conf_icdcsw_aldinuccidpmtt14_b200/).
 *
 * What it computes (PAPER.md = /root/reference/PAPER.md):
 *   - Monte Carlo ensemble of independent instances            P:L47-52 (§I)
 *   - Gillespie's algorithm (direct method, reading R2) on the
 *     flat reaction network of a static CWC term                P:L216-217 (§IV), ref [1] P:L698-699
 *   - the state of every instance at fixed simulation times
 *     ("cuts", trajectory alignment)                            P:L244-251 (§IV.A.1-2)
 * Readings R1-R15 fix what the paper leaves open: propensity convention,
 * RNG stream, the portable log, FP evaluation order, tie rules, sampling convention,
 * absorbing/overflow handling.  This file follows the SURVEY.md §8(c) pseudo-code line by
 * line.  Build with -O2 -ffp-contract=off (no FMA contraction; explicit fma() only where
 * the CWC-log spec says so).
 *
 * Pins (tests/test_oracle_*.py): Random123 Philox KAT vectors, CWC-log vs mpmath (<= 1 ulp),
 * closed forms (Poisson / Binomial laws), exact CME (scipy expm), first-step laws,
 * conservation invariants, brute-force propensities.
 */
#include <math.h>
#include <pthread.h>
#include <stdint.h>
#include <stdlib.h>
#include <string.h>

/* ---------------------------------------------------------------------------------------
 * Philox4x32-10 (Salmon et al., SC'11; Random123).  Reading R3: one block per SSA step,
 * ctr = (lo32(step), hi32(step), lo32(instance), hi32(instance)), key = (lo32(seed), hi32(seed)).
 * Pinned by the Random123 known-answer vectors in tests/golden/philox4x32_10_kat.txt.
 * ------------------------------------------------------------------------------------- */
static void philox_round(uint32_t ctr[4], const uint32_t key[2]) {
    uint64_t p0 = (uint64_t)0xD2511F53u * ctr[0];
    uint64_t p1 = (uint64_t)0xCD9E8D57u * ctr[2];
    uint32_t hi0 = (uint32_t)(p0 >> 32), lo0 = (uint32_t)p0;
    uint32_t hi1 = (uint32_t)(p1 >> 32), lo1 = (uint32_t)p1;
    uint32_t n0 = hi1 ^ ctr[1] ^ key[0];
    uint32_t n1 = lo1;
    uint32_t n2 = hi0 ^ ctr[3] ^ key[1];
    uint32_t n3 = lo0;
    ctr[0] = n0; ctr[1] = n1; ctr[2] = n2; ctr[3] = n3;
}

void oracle_philox4x32_10(const uint32_t in_ctr[4], const uint32_t in_key[2], uint32_t out[4]) {
    uint32_t ctr[4] = {in_ctr[0], in_ctr[1], in_ctr[2], in_ctr[3]};
    uint32_t key[2] = {in_key[0], in_key[1]};
    for (int r = 0; r < 10; ++r) {
        philox_round(ctr, key);
        key[0] += 0x9E3779B9u;
        key[1] += 0xBB67AE85u;
    }
    out[0] = ctr[0]; out[1] = ctr[1]; out[2] = ctr[2]; out[3] = ctr[3];
}

/* 52-bit uniform in (0,1): u = (2*m + 1) * 2^-53 with m = (hi<<32 | lo) >> 12 (reading R3). */
double oracle_u01(uint32_t lo, uint32_t hi) {
    uint64_t m = ((((uint64_t)hi) << 32) | lo) >> 12;
    return (double)(2 * m + 1) * 0x1p-53;
}

/* ---------------------------------------------------------------------------------------
 * CWC-log (reading R4): a fixed, division-free natural log built only from correctly
 * rounded IEEE operations, so any two faithful implementations agree bit for bit.
 *   x = 2^k * z, z in [0.6875, 1.375), table index i = 7 bits after OFF = 0x3fe6000000000000
 *   log x = k*ln2 + log(c_i) + log1p(r),  r = fma(z, 1/c_i, -1),  log1p by degree-8 Taylor.
 * Table (computed here, independently of the product): c_i = midpoint of the z-range of i,
 * invc_i = 1/c_i (i = 79, 80 -> 1.0 exactly), L = -logl(invc_i) in x87 long double,
 * logc_i = (double)L, logclo_i = (double)(L - logc_i)  (a double-double log(c_i)).
 * Pinned: |CWC-log(u) - log(u)| <= 1 ulp against mpmath at 60 digits (tests).
 * ------------------------------------------------------------------------------------- */
#define CWCLOG_N 128
#define CWCLOG_OFF 0x3fe6000000000000ULL
static double cwclog_invc[CWCLOG_N];
static double cwclog_logc[CWCLOG_N];
static double cwclog_logclo[CWCLOG_N];
static pthread_once_t cwclog_once = PTHREAD_ONCE_INIT;

static double as_double(uint64_t b) { double d; memcpy(&d, &b, 8); return d; }
static uint64_t as_bits(double d) { uint64_t b; memcpy(&b, &d, 8); return b; }

static void cwclog_init(void) {
    for (int i = 0; i < CWCLOG_N; ++i) {
        double zlo = as_double(CWCLOG_OFF + ((uint64_t)i << 45));
        double zhi = as_double(CWCLOG_OFF + ((uint64_t)(i + 1) << 45));
        double c = (zlo + zhi) / 2.0;
        double invc = (i == 79 || i == 80) ? 1.0 : 1.0 / c;
        cwclog_invc[i] = invc;
        long double l = -logl((long double)invc);
        cwclog_logc[i] = (double)l;
        cwclog_logclo[i] = (double)(l - (long double)cwclog_logc[i]);
    }
}

void oracle_cwclog_table(double* invc, double* logc, double* logclo) {
    pthread_once(&cwclog_once, cwclog_init);
    for (int i = 0; i < CWCLOG_N; ++i) {
        invc[i] = cwclog_invc[i]; logc[i] = cwclog_logc[i]; logclo[i] = cwclog_logclo[i];
    }
}

static const double LN2HI = 6.93147180369123816490e-01; /* 0x3fe62e42fee00000: k*LN2HI exact */
static const double LN2LO = 1.90821492927058770002e-10; /* 0x3dea39ef35793c76 */

double oracle_cwclog(double x) {
    pthread_once(&cwclog_once, cwclog_init);
    uint64_t ix = as_bits(x);
    uint64_t tmp = ix - CWCLOG_OFF;
    int i = (int)((tmp >> 45) & (CWCLOG_N - 1));
    int64_t k = ((int64_t)tmp) >> 52;
    uint64_t iz = ix - (tmp & (0xfffULL << 52));
    double z = as_double(iz);
    double r = fma(z, cwclog_invc[i], -1.0);
    double kd = (double)k;
    double p = kd * LN2HI;                 /* exact */
    double w = p + cwclog_logc[i];
    double e1 = (p - w) + cwclog_logc[i];  /* Fast2Sum error of w */
    double hi = w + r;
    double e2 = (w - hi) + r;              /* Fast2Sum error of hi */
    /* log1p(r) - r = r^2 * (-1/2 + r/3 - r^2/4 + r^3/5 - r^4/6 + r^5/7 - r^6/8) */
    double q = fma(r, -0.125, 1.0 / 7.0);
    q = fma(r, q, -1.0 / 6.0);
    q = fma(r, q, 0.2);
    q = fma(r, q, -0.25);
    q = fma(r, q, 1.0 / 3.0);
    q = fma(r, q, -0.5);
    double r2 = r * r;
    double t1 = (e1 + e2) + cwclog_logclo[i];
    double t2 = fma(kd, LN2LO, t1);
    double lo = fma(r2, q, t2);
    return hi + lo;
}

/* ---------------------------------------------------------------------------------------
 * Flat model (the oracle's own flattening is oracle/cwc_terms.py).
 * ------------------------------------------------------------------------------------- */
typedef struct {
    int32_t S, M;
    const int32_t* x0;       /* [S] */
    const double* k;         /* [M] rate constants */
    const int32_t* n_react;  /* [M] number of (species, order) reactant entries */
    const int32_t* react_s;  /* [M*ORACLE_RMAX] reactant species */
    const int32_t* react_r;  /* [M*ORACLE_RMAX] reactant orders (stoichiometric coefficient) */
    const int32_t* delta;    /* [M*S] dense net change nu_j */
    int64_t x_cap;           /* reading R9 */
    const int32_t* law;      /* [M] 0 mass action, 1 mm, 2 hill, 3 hillr (reading R16') */
    const int32_t* law_s;    /* [M] species the law reads */
    const double* law_K;     /* [M] */
    const int32_t* law_n;    /* [M] Hill exponent */
    /* reading R20 (dynamic compartments in bounded pools); all may be NULL for static models */
    const int32_t* gate_s;   /* [M] species gating the reaction, -1 none */
    const int32_t* gate_k;   /* [M] 1: enabled while x >= 1, 2: enabled while x == 0 */
    const int32_t* place_off;    /* [M+1] candidate slots of a creation: place_alive[off[j]..off[j+1]) */
    const int32_t* place_alive;  /* [P] occupancy flag species of each candidate slot */
    const int32_t* add_off;      /* [P+1] additions of a slot: add_s/add_n[add_off[p]..add_off[p+1]) */
    const int32_t* add_s;
    const int32_t* add_n;
    const int32_t* xfer_off;     /* [M+1] moves of a destruction: xfer_src/dst[xfer_off[j]..) */
    const int32_t* xfer_src;
    const int32_t* xfer_dst;     /* -1: removed */
    int32_t sentinel;            /* species "#full" (> 0 = a pool overflowed), -1 none */
} oracle_model;

#define ORACLE_RMAX 8   /* reactant entries per flat reaction */
#define ORACLE_SMAX 512 /* species */
#define ORACLE_MMAX 4096 /* flat reactions */

enum { ORACLE_FLAG_ABSORBED = 1, ORACLE_FLAG_OVERFLOWED = 2 };

/* C(x, r): number of distinct r-subsets of x molecules (reading R1, Gillespie 1977). Exact;
 * the caller guarantees (X_cap validation) that every product stays below 2^53. */
static uint64_t binom(int64_t x, int r) {
    if (x < r) return 0;
    uint64_t c = 1;
    for (int i = 0; i < r; ++i) c = c * (uint64_t)(x - i) / (uint64_t)(i + 1);
    return c;
}

/* a_j of one flat reaction.  Mass action (R1): fl(k_j * h_j).  Functional rate laws (reading
 * R16') apply only when the lhs is available (h_j > 0); with X = (double)x_s of
 * the law's species and Y^n = fl(...fl(fl(Y*Y)*Y)...) (n-1 left-to-right products):
 *   mm:    fl(fl(k*X) / fl(K + X))            Michaelis-Menten
 *   hill:  fl(fl(k*X^n) / fl(K^n + X^n))      Hill activation
 *   hillr: fl(fl(k*K^n) / fl(K^n + X^n))      Hill repression */
static double ipow(double y, int n) {
    double r = y;
    for (int i = 1; i < n; ++i) r = r * y;
    return r;
}

static double propensity(const oracle_model* m, int32_t j, const int32_t* x, uint64_t h) {
    const int law = m->law ? m->law[j] : 0;
    /* reading R20: a creation is enabled while its pool has a free slot (gate x >= 1), the
     * pool-full reaction while it has none (gate x == 0) */
    if (m->gate_s && m->gate_s[j] >= 0) {
        const int32_t g = x[m->gate_s[j]];
        if (m->gate_k[j] == 1 ? g < 1 : g != 0) h = 0;
    }
    if (law == 0) return m->k[j] * (double)h;
    if (h == 0) return 0.0;
    const double X = (double)x[m->law_s[j]], K = m->law_K[j];
    if (law == 1) return (m->k[j] * X) / (K + X);
    const double Xn = ipow(X, m->law_n[j]), Kn = ipow(K, m->law_n[j]);
    if (law == 2) return (m->k[j] * Xn) / (Kn + Xn);
    return (m->k[j] * Kn) / (Kn + Xn);
}

typedef struct {
    const oracle_model* m;
    int64_t first, count;     /* instance range [first, first+count) */
    int64_t K;
    double dt;
    uint64_t seed;
    int32_t* raw;             /* [K+1][S][count] or NULL; -1 = missing */
    uint8_t* flags;           /* [count] or NULL */
    int64_t* reactions;       /* [count] or NULL */
    int32_t tid, nthreads;
} job_t;

static void emit(const job_t* jb, int64_t li, int64_t k, const int32_t* x) {
    if (!jb->raw) return;
    int32_t S = jb->m->S;
    for (int32_t s = 0; s < S; ++s) jb->raw[(k * S + s) * jb->count + li] = x[s];
}

static void emit_missing(const job_t* jb, int64_t li, int64_t k) {
    if (!jb->raw) return;
    int32_t S = jb->m->S;
    for (int32_t s = 0; s < S; ++s) jb->raw[(k * S + s) * jb->count + li] = -1;
}

/* One direct-method step of instance li from state (x, *t, *k) with the draw (u_tau, u_sel),
 * SURVEY.md §8(c) pseudo-code from "propensities" to "x += nu_{j*}", in that order:
 *   ORACLE_STEP_ABSORBED   a0 == 0 (R8): cuts k..K hold x, the draw is not consumed
 *   ORACLE_STEP_HORIZON    the next jump lies beyond t_K: cuts up to K emitted, no jump
 *   ORACLE_STEP_OVERFLOWED the jump was applied and a count exceeds X_cap (R9): cuts k..K missing
 *   ORACLE_STEP_JUMP       the jump was applied (cuts strictly before it emitted, R7)
 * *js_out (optional) = the selected reaction j* (-1 when no jump was applied). */
enum { ORACLE_STEP_JUMP = 0, ORACLE_STEP_ABSORBED = 1, ORACLE_STEP_OVERFLOWED = 2, ORACLE_STEP_HORIZON = 3 };

static int ssa_step(const job_t* jb, int64_t li, int32_t* x, double* t, int64_t* k, double u_tau, double u_sel,
                    int32_t* js_out) {
    const oracle_model* m = jb->m;
    const int32_t S = m->S, M = m->M;
    const int64_t K = jb->K;
    static __thread double a[ORACLE_MMAX], cum[ORACLE_MMAX];
    if (js_out) *js_out = -1;
    /* propensities a_j = fl(k_j * (double)h_j), h_j = prod_s C(x_s, r_js) (R1) */
    for (int32_t j = 0; j < M; ++j) {
        uint64_t h = 1;
        for (int32_t e = 0; e < m->n_react[j]; ++e)
            h *= binom(x[m->react_s[j * ORACLE_RMAX + e]], m->react_r[j * ORACLE_RMAX + e]);
        a[j] = propensity(m, j, x, h);
    }
    /* a0 as a left-to-right running sum (R5) */
    double c = 0.0;
    for (int32_t j = 0; j < M; ++j) { c = c + a[j]; cum[j] = c; }
    double a0 = c;
    if (a0 == 0.0) {                          /* absorbing state (R8): hold to t_K, no draw */
        for (; *k <= K; ++*k) emit(jb, li, *k, x);
        return ORACLE_STEP_ABSORBED;
    }
    double tau = -oracle_cwclog(u_tau) / a0;
    double t_next = *t + tau;
    /* cuts at t_k = fl(k*dt) strictly before the next jump: cadlag sampling (R7) */
    while (*k <= K && (double)*k * jb->dt < t_next) { emit(jb, li, *k, x); ++*k; }
    if (*k > K) return ORACLE_STEP_HORIZON;
    /* rule selection (R6): j* = min{ j : cum_j > u_sel*a0 }, else last positive a_j */
    double target = u_sel * a0;
    int32_t js = -1;
    for (int32_t j = 0; j < M; ++j) if (cum[j] > target) { js = j; break; }
    if (js < 0) for (int32_t j = M - 1; j >= 0; --j) if (a[j] > 0.0) { js = j; break; }
    if (js_out) *js_out = js;
    /* multiset rewrite: x += nu_{j*} */
    for (int32_t s = 0; s < S; ++s) x[s] += m->delta[js * S + s];
    /* reading R20: a creation fills the first free slot of its pool; a destruction moves the
     * rest of the dissolved compartment to the context (or removes it) */
    if (m->place_off)
        for (int32_t p = m->place_off[js]; p < m->place_off[js + 1]; ++p)
            if (x[m->place_alive[p]] == 0) {
                for (int32_t e = m->add_off[p]; e < m->add_off[p + 1]; ++e) x[m->add_s[e]] += m->add_n[e];
                break;
            }
    if (m->xfer_off)
        for (int32_t e = m->xfer_off[js]; e < m->xfer_off[js + 1]; ++e) {
            if (m->xfer_dst[e] >= 0) x[m->xfer_dst[e]] += x[m->xfer_src[e]];
            x[m->xfer_src[e]] = 0;
        }
    *t = t_next;
    int over = 0;
    for (int32_t s = 0; s < S; ++s) if (x[s] > m->x_cap) over = 1;
    if (m->sentinel >= 0 && x[m->sentinel] > 0) over = 1;
    if (over) {                               /* R9: freeze, remaining samples missing */
        for (; *k <= K; ++*k) emit_missing(jb, li, *k);
        return ORACLE_STEP_OVERFLOWED;
    }
    return ORACLE_STEP_JUMP;
}

/* One instance: the draw of step n is Philox4x32-10 block (ctr = (n, i), key = seed) (R3),
 * mapped to two 52-bit uniforms; steps until absorption, overflow or the horizon. */
static void simulate_instance(const job_t* jb, int64_t li) {
    const oracle_model* m = jb->m;
    const int32_t S = m->S;
    const uint64_t i = (uint64_t)(jb->first + li);
    int32_t x[ORACLE_SMAX];
    for (int32_t s = 0; s < S; ++s) x[s] = m->x0[s];
    double t = 0.0;
    uint64_t step = 0;
    int64_t k = 0, reactions = 0;
    uint8_t flag = 0;
    const uint32_t key[2] = {(uint32_t)jb->seed, (uint32_t)(jb->seed >> 32)};
    for (;;) {
        uint32_t ctr[4] = {(uint32_t)step, (uint32_t)(step >> 32), (uint32_t)i, (uint32_t)(i >> 32)};
        uint32_t w[4];
        oracle_philox4x32_10(ctr, key, w);
        double u_tau = oracle_u01(w[0], w[1]);
        double u_sel = oracle_u01(w[2], w[3]);
        int st = ssa_step(jb, li, x, &t, &k, u_tau, u_sel, NULL);
        if (st == ORACLE_STEP_ABSORBED) { flag = ORACLE_FLAG_ABSORBED; break; }
        if (st == ORACLE_STEP_HORIZON) break;
        step += 1;                            /* the draw was consumed: one reaction applied */
        reactions += 1;
        if (st == ORACLE_STEP_OVERFLOWED) { flag = ORACLE_FLAG_OVERFLOWED; break; }
    }
    if (jb->flags) jb->flags[li] = flag;
    if (jb->reactions) jb->reactions[li] = reactions;
}

/* Injected-draw trajectory (pins of R6/R7 with crafted uniforms; the device counterpart is
 * cwc_selftest_step): from state (x, *t, *k), apply up to n_draws steps of ssa_step with the
 * draws (u_tau[d], u_sel[d]), stopping at the first step that is not a jump.  Cuts emitted go to
 * cuts[k][s] ([K+1][S], caller-initialised; -1 = missing after an overflow); js[d] (optional)
 * receives the selected reactions.  Returns the status of the last step taken (ORACLE_STEP_*)
 * and *n_done the number of steps taken (draws consumed + a final non-jump step). */
int oracle_step_with_draws(const oracle_model* m, int32_t* x, double* t, int64_t* k, int64_t K, double dt,
                           int32_t n_draws, const double* u_tau, const double* u_sel, int32_t* cuts, int32_t* js,
                           int32_t* n_done) {
    if (!m || m->S <= 0 || m->S > ORACLE_SMAX || m->M < 0 || m->M > ORACLE_MMAX || K < 0 || !(dt > 0) ||
        n_draws < 0 || *k < 0 || *k > K + 1)
        return -1;
    pthread_once(&cwclog_once, cwclog_init);
    job_t jb = {m, 0, 1, K, dt, 0, cuts, NULL, NULL, 0, 1};
    int st = ORACLE_STEP_JUMP;
    int32_t d = 0;
    for (; d < n_draws; ++d) {
        st = ssa_step(&jb, 0, x, t, k, u_tau[d], u_sel[d], js ? js + d : NULL);
        if (st != ORACLE_STEP_JUMP) { ++d; break; }
    }
    if (n_done) *n_done = d;
    return st;
}

static void* worker(void* arg) {
    const job_t* jb = (const job_t*)arg;
    for (int64_t li = jb->tid; li < jb->count; li += jb->nthreads) simulate_instance(jb, li);
    return NULL;
}

/* Simulate instances [first, first+count) with nthreads POSIX threads (static interleave).
 * Returns 0 on success, -1 on invalid arguments. */
int oracle_simulate(const oracle_model* m, int64_t first, int64_t count, int64_t K, double dt,
                    uint64_t seed, int32_t nthreads, int32_t* raw, uint8_t* flags,
                    int64_t* reactions) {
    if (!m || m->S <= 0 || m->S > ORACLE_SMAX || m->M < 0 || m->M > ORACLE_MMAX || count < 0 || K < 0 || !(dt > 0))
        return -1;
    pthread_once(&cwclog_once, cwclog_init);
    if (nthreads < 1) nthreads = 1;
    job_t* jobs = (job_t*)calloc((size_t)nthreads, sizeof(job_t));
    pthread_t* th = (pthread_t*)calloc((size_t)nthreads, sizeof(pthread_t));
    for (int32_t t = 0; t < nthreads; ++t) {
        job_t j = {m, first, count, K, dt, seed, raw, flags, reactions, t, nthreads};
        jobs[t] = j;
    }
    for (int32_t t = 1; t < nthreads; ++t) pthread_create(&th[t], NULL, worker, &jobs[t]);
    worker(&jobs[0]);
    for (int32_t t = 1; t < nthreads; ++t) pthread_join(th[t], NULL);
    free(jobs);
    free(th);
    return 0;
}

/* Propensities and cumulative sums of one state (exposed for brute-force pin tests). */
void oracle_propensities(const oracle_model* m, const int32_t* x, double* a, double* cum) {
    double c = 0.0;
    for (int32_t j = 0; j < m->M; ++j) {
        uint64_t h = 1;
        for (int32_t e = 0; e < m->n_react[j]; ++e)
            h *= binom(x[m->react_s[j * ORACLE_RMAX + e]], m->react_r[j * ORACLE_RMAX + e]);
        a[j] = propensity(m, j, x, h);
        c = c + a[j];
        cum[j] = c;
    }
}

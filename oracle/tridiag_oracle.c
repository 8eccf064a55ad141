/*
 * tridiag_oracle.c -- TEST INFRASTRUCTURE ONLY.
 *
 * Plain, slow, obviously-correct CPU implementations of what the paper
 * "Fast Tridiagonal Solvers on the GPU" (Zhang, Cohen, Owens, PPoPP'10;
 * /root/reference/PAPER.md, cited as P:L<line>) computes.  Only tests/,
 * __graft_entry__.smoke() and bench.py's cpu_baseline / --impl reference legs
 * may load this library.  It shares no code, header or table with the CUDA
 * path (paper_conf_ppopp_zhangco10_b200/csrc) and never includes it.
 *
 * Every routine is written once as a macro body over the element type T and
 * instantiated for double (suffix _f64, the parity oracle) and float (suffix
 * _f32, used only to model the paper's fp32 behaviour, e.g. the RD overflow
 * onset of P:L1219-1221).
 *
 * Conventions (DESIGN.md "Readings" R1-R22 = SURVEY.md 8(c) items 1-22):
 *   - 0-based.  Equation i of system s:  a_i x_{i-1} + b_i x_i + c_i x_{i+1} = d_i,
 *     element i of system s at ptr[s*n + i] for each of a, b, c, d, x.
 *   - a_0 and c_{n-1} are not matrix entries (the matrix at P:L166-181 has no
 *     a_1 and no c_n): every routine copies the system and sets them to 0
 *     before use, so any value (including NaN) in the caller's arrays is
 *     ignored (reading R1).
 *   - Absent neighbours contribute 0 (reading R3).
 *   - n must be a power of two >= 2 for CR, PCR, RD and the hybrids;
 *     Thomas accepts any n >= 1.
 *
 * Step counting: *steps receives the number of parallel algorithmic steps of
 * ONE system as the paper counts them (CR 2log2n-1 P:L311, PCR log2n
 * P:L384-385, RD log2n+2 P:L420-421, hybrids per reading R13).
 *
 * Event log (for the Fig 1-4 dataflow pins): when log != NULL, the events of
 * system 0 are appended as rows of 5 int64 {step, kind, i, p, q}:
 *   kind 0 CR forward update of equation i from neighbours p=i-h, q=i+h (-1 absent)
 *   kind 1 2x2 solve of unknowns (p, q) (i = -1)
 *   kind 2 CR backward substitution of x_i from x_p, x_q (-1 absent)
 *   kind 3 PCR update of equation i from p=i-s, q=i+s (-1 absent)
 *   kind 4 RD matrix setup of B_i
 *   kind 5 RD scan: after this step C_i is the product of matrices p..q
 *   kind 6 RD evaluation of x_i
 * Indices in the log are the ones of the (sub)system the algorithm runs on.
 */
#include <math.h>
#include <pthread.h>
#include <stdint.h>
#include <stdlib.h>
#include <string.h>

#define ORACLE_ABI_VERSION 1

int oracle_abi_version(void) { return ORACLE_ABI_VERSION; }

typedef struct {
    int64_t* buf;
    int64_t cap;  /* rows */
    int64_t len;  /* rows written (may exceed cap: then truncated) */
} evlog_t;

static void ev(evlog_t* L, int64_t step, int64_t kind, int64_t i, int64_t p, int64_t q) {
    if (!L || !L->buf) return;
    if (L->len < L->cap) {
        int64_t* r = L->buf + 5 * L->len;
        r[0] = step; r[1] = kind; r[2] = i; r[3] = p; r[4] = q;
    }
    L->len++;
}

static int is_pow2(int64_t n) { return n >= 1 && (n & (n - 1)) == 0; }
static int ilog2(int64_t n) { int l = 0; while ((1LL << l) < n) ++l; return l; }

/* ---------------------------------------------------------------------- */
/* Thomas algorithm = Gaussian elimination without pivoting.   */
/* 0-based restatement of P:L186-205 (with the d' index range typo of      */
/* P:L193-199 read as i = 2..n, reading R2):                                */
/*   c'_0 = c_0/b_0, d'_0 = d_0/b_0                                         */
/*   c'_i = c_i/(b_i - c'_{i-1} a_i),  d'_i = (d_i - d'_{i-1} a_i)/(b_i - c'_{i-1} a_i)  */
/*   x_{n-1} = d'_{n-1},  x_i = d'_i - c'_i x_{i+1}.                        */
/* ---------------------------------------------------------------------- */
#define DEFINE_THOMAS(T, SFX)                                                          \
int oracle_thomas_##SFX(const T* a, const T* b, const T* c, const T* d, T* x,          \
                        int64_t n, int64_t S) {                                        \
    if (n < 1 || S < 0) return -1;                                                     \
    T* cp = (T*)malloc(sizeof(T) * (size_t)n);                                         \
    T* dp = (T*)malloc(sizeof(T) * (size_t)n);                                         \
    if (!cp || !dp) { free(cp); free(dp); return -2; }                                 \
    for (int64_t s = 0; s < S; ++s) {                                                  \
        const T* A = a + s * n; const T* B = b + s * n;                                \
        const T* C = c + s * n; const T* D = d + s * n; T* X = x + s * n;              \
        /* c_{n-1} is not a matrix entry: c'_{n-1} is never formed (reading R1). */    \
        cp[0] = (n > 1) ? C[0] / B[0] : (T)0;                                          \
        dp[0] = D[0] / B[0];                                                           \
        for (int64_t i = 1; i < n; ++i) {                                              \
            T den = B[i] - cp[i - 1] * A[i];                                           \
            cp[i] = (i < n - 1) ? C[i] / den : (T)0;                                   \
            dp[i] = (D[i] - dp[i - 1] * A[i]) / den;                                   \
        }                                                                              \
        X[n - 1] = dp[n - 1];                                                          \
        for (int64_t i = n - 2; i >= 0; --i) X[i] = dp[i] - cp[i] * X[i + 1];          \
    }                                                                                  \
    free(cp); free(dp);                                                                \
    return 0;                                                                          \
}

/* ---------------------------------------------------------------------- */
/* Shared building blocks of CR (Fig 1) used by CR and the      */
/* hybrids (Fig 4).  w = working copy of one system (a,b,c,d).  */
/* ---------------------------------------------------------------------- */
/* One CR forward-reduction level with stride h: every equation
 * i with i = 2h-1 (mod 2h) is replaced by the linear combination of
 * equations i-h, i, i+h that eliminates x_{i-h} and x_{i+h}:
 *   k1 = a_i/b_{i-h}, k2 = c_i/b_{i+h}
 *   a'_i = -a_{i-h} k1, b'_i = b_i - c_{i-h} k1 - a_{i+h} k2,
 *   c'_i = -c_{i+h} k2, d'_i = d_i - d_{i-h} k1 - d_{i+h} k2.
 * The neighbours i+-h are not themselves updated at this level, so updating
 * in place reads pre-step values.  An absent neighbour
 * (i+h >= n) contributes nothing (reading R3). */
#define DEFINE_CR_LEVELS(T, SFX)                                                       \
static void cr_forward_level_##SFX(T* A, T* B, T* C, T* D, int64_t n, int64_t h,       \
                                   evlog_t* L, int64_t step) {                         \
    for (int64_t i = 2 * h - 1; i < n; i += 2 * h) {                                   \
        int64_t lo = i - h, hi = i + h;                                                \
        T k1 = A[i] / B[lo];                                                           \
        T a_new = -A[lo] * k1;                                                         \
        T b_new = B[i] - C[lo] * k1;                                                   \
        T d_new = D[i] - D[lo] * k1;                                                   \
        T c_new = (T)0;                                                                \
        if (hi < n) {                                                                  \
            T k2 = C[i] / B[hi];                                                       \
            b_new -= A[hi] * k2;                                                       \
            d_new -= D[hi] * k2;                                                       \
            c_new = -C[hi] * k2;                                                       \
        }                                                                              \
        A[i] = a_new; B[i] = b_new; C[i] = c_new; D[i] = d_new;                        \
        ev(L, step, 0, i, lo, hi < n ? hi : -1);                                       \
    }                                                                                  \
}                                                                                      \
/* One CR backward-substitution level with stride h:             \
 *   x_i = (d'_i - a'_i x_{i-h} - c'_i x_{i+h}) / b'_i  for i = h-1 (mod 2h),  \
 * with x_{i-h} := 0 when i < h (the "first unknown", reading R3).  The        \
 * coefficients are the ones equation i had when it was last updated, i.e.     \
 * at level log2(h) -- exactly what the in-place arrays hold. */               \
static void cr_backward_level_##SFX(const T* A, const T* B, const T* C, const T* D,    \
                                    T* X, int64_t n, int64_t h, evlog_t* L,            \
                                    int64_t step) {                                    \
    for (int64_t i = h - 1; i < n; i += 2 * h) {                                       \
        T xl = (i - h >= 0) ? X[i - h] : (T)0;                                         \
        T xh = (i + h < n) ? X[i + h] : (T)0;                                          \
        X[i] = (D[i] - A[i] * xl - C[i] * xh) / B[i];                                  \
        ev(L, step, 2, i, i - h >= 0 ? i - h : -1, i + h < n ? i + h : -1);            \
    }                                                                                  \
}                                                                                      \
/* 2-unknown solve (formula not printed -> Cramer's rule,           \
 * reading R5):  b_p x_p + c_p x_q = d_p,  a_q x_p + b_q x_q = d_q. */          \
static void solve2_##SFX(T bp, T cp, T dp, T aq, T bq, T dq, T* xp, T* xq) {           \
    T det = bp * bq - cp * aq;                                                         \
    *xp = (dp * bq - cp * dq) / det;                                                   \
    *xq = (bp * dq - dp * aq) / det;                                                   \
}

/* Copy one system into a zero-cornered working copy (reading R1). */
#define DEFINE_LOAD(T, SFX)                                                            \
static void load_sys_##SFX(const T* a, const T* b, const T* c, const T* d, int64_t n,  \
                           T* A, T* B, T* C, T* D) {                                   \
    memcpy(A, a, sizeof(T) * (size_t)n); memcpy(B, b, sizeof(T) * (size_t)n);          \
    memcpy(C, c, sizeof(T) * (size_t)n); memcpy(D, d, sizeof(T) * (size_t)n);          \
    A[0] = (T)0; C[n - 1] = (T)0;                                                      \
}

/* ---------------------------------------------------------------------- */
/* Cyclic reduction, serial textbook form (Fig 1):               */
/* log2n-1 forward levels (h = 1, 2, ..., n/4), a 2-unknown solve of         */
/* (n/2-1, n-1), log2n-1 backward levels (h = n/4, ..., 1).                  */
/* ---------------------------------------------------------------------- */
#define DEFINE_CR(T, SFX)                                                              \
int oracle_cr_##SFX(const T* a, const T* b, const T* c, const T* d, T* x,              \
                    int64_t n, int64_t S, int64_t* steps,                              \
                    int64_t* log, int64_t log_cap, int64_t* log_len) {                 \
    if (!is_pow2(n) || n < 2 || S < 0) return -1;                                      \
    T* w = (T*)malloc(sizeof(T) * 4 * (size_t)n);                                      \
    if (!w) return -2;                                                                 \
    T *A = w, *B = w + n, *C = w + 2 * n, *D = w + 3 * n;                              \
    evlog_t Lg = {log, log_cap, 0};                                                    \
    int64_t st = 0;                                                                    \
    for (int64_t s = 0; s < S; ++s) {                                                  \
        evlog_t* L = (s == 0) ? &Lg : NULL;                                            \
        T* X = x + s * n;                                                              \
        load_sys_##SFX(a + s * n, b + s * n, c + s * n, d + s * n, n, A, B, C, D);     \
        st = 0;                                                                        \
        for (int64_t h = 1; h < n / 2; h *= 2)                                         \
            cr_forward_level_##SFX(A, B, C, D, n, h, L, ++st);                         \
        int64_t p = n / 2 - 1, q = n - 1;                                              \
        solve2_##SFX(B[p], C[p], D[p], A[q], B[q], D[q], &X[p], &X[q]);                \
        ev(L, ++st, 1, -1, p, q);                                                      \
        for (int64_t h = n / 4; h >= 1; h /= 2)                                        \
            cr_backward_level_##SFX(A, B, C, D, X, n, h, L, ++st);                     \
    }                                                                                  \
    if (steps) *steps = st;                                                            \
    if (log_len) *log_len = Lg.len;                                                    \
    free(w);                                                                           \
    return 0;                                                                          \
}

/* ---------------------------------------------------------------------- */
/* PCR on one m-equation system held in (A,B,C,D), solution into X           */
/* (Fig 2).  Steps s = 1, 2, ..., m/4: every equation is reduced */
/* simultaneously from the PRE-step values (the reduction formula of CR with */
/* neighbours i-s, i+s; absent neighbours contribute nothing), splitting     */
/* each system into two of half size.  Final step: solve the m/2 2-unknown   */
/* systems (i, i+m/2) (Fig 2 "Solve the 4 2-unknown systems", reading R6).   */
/* Returns the number of steps (log2 m).                                     */
/* ---------------------------------------------------------------------- */
#define DEFINE_PCR_CORE(T, SFX)                                                        \
static int64_t pcr_core_##SFX(T* A, T* B, T* C, T* D, T* X, int64_t m, T* tmp,         \
                              evlog_t* L, int64_t step0) {                             \
    T *A2 = tmp, *B2 = tmp + m, *C2 = tmp + 2 * m, *D2 = tmp + 3 * m;                  \
    int64_t st = step0;                                                                \
    for (int64_t s = 1; s <= m / 4; s *= 2) {                                          \
        ++st;                                                                          \
        for (int64_t i = 0; i < m; ++i) {                                              \
            int64_t lo = i - s, hi = i + s;                                            \
            T a_new = (T)0, b_new = B[i], c_new = (T)0, d_new = D[i];                  \
            if (lo >= 0) {                                                             \
                T k1 = A[i] / B[lo];                                                   \
                a_new = -A[lo] * k1;                                                   \
                b_new -= C[lo] * k1;                                                   \
                d_new -= D[lo] * k1;                                                   \
            }                                                                          \
            if (hi < m) {                                                              \
                T k2 = C[i] / B[hi];                                                   \
                c_new = -C[hi] * k2;                                                   \
                b_new -= A[hi] * k2;                                                   \
                d_new -= D[hi] * k2;                                                   \
            }                                                                          \
            A2[i] = a_new; B2[i] = b_new; C2[i] = c_new; D2[i] = d_new;                \
            ev(L, st, 3, i, lo >= 0 ? lo : -1, hi < m ? hi : -1);                      \
        }                                                                              \
        memcpy(A, A2, sizeof(T) * (size_t)m); memcpy(B, B2, sizeof(T) * (size_t)m);    \
        memcpy(C, C2, sizeof(T) * (size_t)m); memcpy(D, D2, sizeof(T) * (size_t)m);    \
    }                                                                                  \
    ++st;                                                                              \
    for (int64_t i = 0; i < m / 2; ++i) {                                              \
        int64_t p = i, q = i + m / 2;                                                  \
        solve2_##SFX(B[p], C[p], D[p], A[q], B[q], D[q], &X[p], &X[q]);                \
        ev(L, st, 1, -1, p, q);                                                        \
    }                                                                                  \
    return st - step0;                                                                 \
}

/* ---------------------------------------------------------------------- */
/* Recursive doubling, Egecioglu's scan form of Stone's algorithm            */
/* (Fig 3), on one m-equation system, solution into X.           */
/* Readings R7-R10: B_i = [[-b_i/c_i, -a_i/c_i, d_i/c_i],[1,0,0],[0,0,1]]    */
/* maps X_i = [x_i, x_{i-1}, 1]^T to X_{i+1}; for the last equation c is     */
/* replaced by 1 and x_m := 0 is imposed; a_0 := 0 (x_{-1} absent).          */
/* Hillis-Steele inclusive scan: for s = 1, 2, ..., m/2, from   */
/* pre-step values, C_i <- C_i * C_{i-s} for i >= s (later matrix on the     */
/* left, reading R10), so that C_i = B_i ... B_1 B_0.  Then                  */
/* x_0 = -C_{m-1}[0][2] / C_{m-1}[0][0] and                         */
/* x_i = C_{i-1}[0][0] x_0 + C_{i-1}[0][2] (reading R9).         */
/* The full 3x3 products are formed (no 2-row shortcut): plain definition.   */
/* Returns the number of steps (setup + log2 m scan steps + evaluation).     */
/* ---------------------------------------------------------------------- */
#define DEFINE_RD_CORE(T, SFX)                                                         \
static void mat3_mul_##SFX(const T* P, const T* Q, T* R) { /* R = P*Q, row-major */    \
    for (int r = 0; r < 3; ++r)                                                        \
        for (int col = 0; col < 3; ++col) {                                            \
            T acc = (T)0;                                                              \
            for (int k = 0; k < 3; ++k) acc += P[3 * r + k] * Q[3 * k + col];          \
            R[3 * r + col] = acc;                                                      \
        }                                                                              \
}                                                                                      \
static int64_t rd_core_##SFX(const T* A, const T* B, const T* C, const T* D, T* X,     \
                             int64_t m, T* Cm, T* Cm2, int64_t* lo_idx,                \
                             int64_t* lo_idx2, evlog_t* L, int64_t step0) {            \
    int64_t st = step0 + 1;                                                            \
    for (int64_t i = 0; i < m; ++i) {                                                  \
        T ci = (i < m - 1) ? C[i] : (T)1;                                              \
        T ai = (i > 0) ? A[i] : (T)0;                                                  \
        T* M = Cm + 9 * i;                                                             \
        M[0] = -B[i] / ci; M[1] = -ai / ci; M[2] = D[i] / ci;                          \
        M[3] = (T)1;       M[4] = (T)0;     M[5] = (T)0;                               \
        M[6] = (T)0;       M[7] = (T)0;     M[8] = (T)1;                               \
        lo_idx[i] = i;                                                                 \
        ev(L, st, 4, i, i, i);                                                         \
    }                                                                                  \
    for (int64_t s = 1; s < m; s *= 2) {                                               \
        ++st;                                                                          \
        memcpy(Cm2, Cm, sizeof(T) * 9 * (size_t)m);                                    \
        memcpy(lo_idx2, lo_idx, sizeof(int64_t) * (size_t)m);                          \
        for (int64_t i = 0; i < m; ++i) {                                              \
            if (i >= s) {                                                              \
                mat3_mul_##SFX(Cm2 + 9 * i, Cm2 + 9 * (i - s), Cm + 9 * i);            \
                lo_idx[i] = lo_idx2[i - s];                                            \
            }                                                                          \
            ev(L, st, 5, i, lo_idx[i], i);                                             \
        }                                                                              \
    }                                                                                  \
    ++st;                                                                              \
    const T* Cl = Cm + 9 * (m - 1);                                                    \
    T x0 = -Cl[2] / Cl[0];                                                             \
    X[0] = x0;                                                                         \
    ev(L, st, 6, 0, m - 1, -1);                                                        \
    for (int64_t i = 1; i < m; ++i) {                                                  \
        const T* Ci = Cm + 9 * (i - 1);                                                \
        X[i] = Ci[0] * x0 + Ci[2];                                                     \
        ev(L, st, 6, i, i - 1, -1);                                                    \
    }                                                                                  \
    return st - step0;                                                                 \
}

/* ---------------------------------------------------------------------- */
/* Stand-alone PCR and RD (whole system), and the hybrids CR+PCR / CR+RD     */
/* (Fig 4): k = log2(n/m) CR forward levels; copy the m          */
/* surviving equations i_j = (j+1) 2^k - 1, j = 0..m-1, into a contiguous    */
/* m-system; solve it with PCR or RD; scatter x; k CR backward  */
/* levels.  inner: 0 = PCR, 1 = RD.  m = n gives the plain PCR / RD.         */
/* ---------------------------------------------------------------------- */
#define DEFINE_HYBRID(T, SFX)                                                          \
int oracle_hybrid_##SFX(const T* a, const T* b, const T* c, const T* d, T* x,          \
                        int64_t n, int64_t S, int inner, int64_t m, int64_t* steps,    \
                        int64_t* log, int64_t log_cap, int64_t* log_len) {             \
    if (!is_pow2(n) || n < 2 || S < 0) return -1;                                      \
    if (!is_pow2(m) || m < 2 || m > n) return -3;                                      \
    if (inner != 0 && inner != 1) return -4;                                           \
    size_t nn = (size_t)n, mm = (size_t)m;                                             \
    T* w = (T*)malloc(sizeof(T) * (4 * nn + 5 * mm + 4 * mm + 18 * mm));               \
    int64_t* li = (int64_t*)malloc(sizeof(int64_t) * 2 * mm);                          \
    if (!w || !li) { free(w); free(li); return -2; }                                   \
    T *A = w, *B = w + nn, *C = w + 2 * nn, *D = w + 3 * nn;                           \
    T *mA = w + 4 * nn, *mB = mA + mm, *mC = mB + mm, *mD = mC + mm, *mX = mD + mm;    \
    T *tmp = mX + mm, *Cm = tmp + 4 * mm, *Cm2 = Cm + 9 * mm;                          \
    evlog_t Lg = {log, log_cap, 0};                                                    \
    int64_t st = 0;                                                                    \
    int64_t k = ilog2(n / m);                                                          \
    for (int64_t s = 0; s < S; ++s) {                                                  \
        evlog_t* L = (s == 0) ? &Lg : NULL;                                            \
        T* X = x + s * n;                                                              \
        load_sys_##SFX(a + s * n, b + s * n, c + s * n, d + s * n, n, A, B, C, D);     \
        st = 0;                                                                        \
        int64_t h = 1;                                                                 \
        for (int64_t l = 0; l < k; ++l, h *= 2)                                        \
            cr_forward_level_##SFX(A, B, C, D, n, h, L, ++st);                         \
        int64_t stride = (int64_t)1 << k;                                              \
        for (int64_t j = 0; j < m; ++j) {                                              \
            int64_t i = (j + 1) * stride - 1;                                          \
            mA[j] = A[i]; mB[j] = B[i]; mC[j] = C[i]; mD[j] = D[i];                    \
        }                                                                              \
        mA[0] = (T)0; mC[m - 1] = (T)0;                                                \
        if (inner == 0) st += pcr_core_##SFX(mA, mB, mC, mD, mX, m, tmp, L, st);       \
        else st += rd_core_##SFX(mA, mB, mC, mD, mX, m, Cm, Cm2, li, li + m, L, st);   \
        for (int64_t j = 0; j < m; ++j) X[(j + 1) * stride - 1] = mX[j];               \
        for (h = stride / 2; h >= 1; h /= 2)                                           \
            cr_backward_level_##SFX(A, B, C, D, X, n, h, L, ++st);                     \
    }                                                                                  \
    if (steps) *steps = st;                                                            \
    if (log_len) *log_len = Lg.len;                                                    \
    free(w); free(li);                                                                 \
    return 0;                                                                          \
}                                                                                      \
int oracle_pcr_##SFX(const T* a, const T* b, const T* c, const T* d, T* x, int64_t n,  \
                     int64_t S, int64_t* steps, int64_t* log, int64_t log_cap,         \
                     int64_t* log_len) {                                               \
    return oracle_hybrid_##SFX(a, b, c, d, x, n, S, 0, n, steps, log, log_cap, log_len);\
}                                                                                      \
int oracle_rd_##SFX(const T* a, const T* b, const T* c, const T* d, T* x, int64_t n,   \
                    int64_t S, int64_t* steps, int64_t* log, int64_t log_cap,          \
                    int64_t* log_len) {                                                \
    return oracle_hybrid_##SFX(a, b, c, d, x, n, S, 1, n, steps, log, log_cap, log_len);\
}

/* ---------------------------------------------------------------------- */
/* Overflow-free recursive doubling in LU form (the  */
/* paper names the overflow problem of its RD, and cites      */
/* Stone [27] for the method).  Three Hillis-Steele scans:     */
/*  1. pivots of A = LU: u_0 = b_0, u_i = b_i - a_i c_{i-1} / u_{i-1}, via    */
/*     the continuant [q_i, q_{i-1}] = M_i [q_{i-1}, q_{i-2}],               */
/*     M_i = [[b_i, -a_i c_{i-1}], [1, 0]], q_{-1} = 1, q_{-2} = 0:           */
/*     P_i = M_i ... M_0 (later matrix on the left), u_i = P_i[0][0] /       */
/*     P_i[1][0]; every product is rescaled by a power of two (exact) so     */
/*     that its largest entry lies in [1, 2): no overflow, same ratios;      */
/*  2. L y = d, l_i = a_i / u_{i-1}: affine maps y -> -l_i y + d_i composed  */
/*     from the left (y_0 = d_0);                                           */
/*  3. U x = y: affine maps x -> -(c_i/u_i) x + y_i/u_i composed from the    */
/*     right (x_{n-1} = y_{n-1}/u_{n-1}).                                    */
/* Steps: 3 log2 n scan steps + 3 setup steps + 1 evaluation.               */
/* ---------------------------------------------------------------------- */
#define DEFINE_STONE(T, SFX)                                                           \
static void stone_rescale_##SFX(T* M) { /* M[4] = [[m0 m1],[m2 m3]] */                  \
    T mx = 0;                                                                          \
    for (int e = 0; e < 4; ++e) { T v = M[e] < 0 ? -M[e] : M[e]; if (v > mx) mx = v; } \
    if (mx > 0 && mx == mx && mx < (T)INFINITY) {                                      \
        int ex; frexp((double)mx, &ex);                                                \
        for (int e = 0; e < 4; ++e) M[e] = (T)ldexp((double)M[e], 1 - ex);             \
    }                                                                                  \
}                                                                                      \
int oracle_rd_stone_##SFX(const T* a, const T* b, const T* c, const T* d, T* x,        \
                          int64_t n, int64_t S, int64_t* steps, int64_t* log,          \
                          int64_t log_cap, int64_t* log_len) {                         \
    if (!is_pow2(n) || n < 2 || S < 0) return -1;                                      \
    size_t nn = (size_t)n;                                                             \
    T* w = (T*)malloc(sizeof(T) * (4 * nn + 8 * nn + 4 * nn + 3 * nn));                \
    if (!w) return -2;                                                                 \
    T *A = w, *B = w + nn, *C = w + 2 * nn, *D = w + 3 * nn;                           \
    T *Pm = w + 4 * nn, *Pm2 = Pm + 4 * nn;      /* 2x2 products (4 per eq) */        \
    T *F = Pm2 + 4 * nn, *F2 = F + 2 * nn;       /* affine maps (alpha, beta) */       \
    T *U = F2 + 2 * nn, *Y = U + nn;                                                   \
    evlog_t Lg = {log, log_cap, 0};                                                    \
    int64_t st = 0;                                                                    \
    (void)Y;                                                                           \
    for (int64_t s = 0; s < S; ++s) {                                                  \
        evlog_t* L = (s == 0) ? &Lg : NULL;                                            \
        (void)L;                                                                       \
        T* X = x + s * n;                                                              \
        load_sys_##SFX(a + s * n, b + s * n, c + s * n, d + s * n, n, A, B, C, D);     \
        st = 1; /* setup of M_i */                                                     \
        for (int64_t i = 0; i < n; ++i) {                                              \
            T* M = Pm + 4 * i;                                                         \
            M[0] = B[i]; M[1] = (i > 0) ? -A[i] * C[i - 1] : (T)0; M[2] = 1; M[3] = 0;  \
        }                                                                              \
        for (int64_t sh = 1; sh < n; sh *= 2) {                                        \
            ++st;                                                                      \
            memcpy(Pm2, Pm, sizeof(T) * 4 * nn);                                       \
            for (int64_t i = sh; i < n; ++i) {                                         \
                const T* P = Pm2 + 4 * i; const T* Q = Pm2 + 4 * (i - sh);             \
                T* R = Pm + 4 * i;                                                     \
                R[0] = P[0] * Q[0] + P[1] * Q[2]; R[1] = P[0] * Q[1] + P[1] * Q[3];    \
                R[2] = P[2] * Q[0] + P[3] * Q[2]; R[3] = P[2] * Q[1] + P[3] * Q[3];    \
                stone_rescale_##SFX(R);                                                \
            }                                                                          \
        }                                                                              \
        for (int64_t i = 0; i < n; ++i) U[i] = Pm[4 * i] / Pm[4 * i + 2];              \
        ++st; /* setup of the forward maps */                                          \
        for (int64_t i = 0; i < n; ++i) {                                              \
            F[2 * i] = (i > 0) ? -(A[i] / U[i - 1]) : (T)0; F[2 * i + 1] = D[i];        \
        }                                                                              \
        for (int64_t sh = 1; sh < n; sh *= 2) {                                        \
            ++st;                                                                      \
            memcpy(F2, F, sizeof(T) * 2 * nn);                                         \
            for (int64_t i = sh; i < n; ++i) {   /* F_i o F_{i-sh} */                  \
                F[2 * i] = F2[2 * i] * F2[2 * (i - sh)];                               \
                F[2 * i + 1] = F2[2 * i] * F2[2 * (i - sh) + 1] + F2[2 * i + 1];       \
            }                                                                          \
        }                                                                              \
        ++st; /* setup of the backward maps from y_i = F_i.beta */                     \
        for (int64_t i = 0; i < n; ++i) {                                              \
            T yi = F[2 * i + 1];                                                       \
            F2[2 * i] = (i < n - 1) ? -(C[i] / U[i]) : (T)0;                           \
            F2[2 * i + 1] = yi / U[i];                                                 \
        }                                                                              \
        memcpy(F, F2, sizeof(T) * 2 * nn);                                             \
        for (int64_t sh = 1; sh < n; sh *= 2) {                                        \
            ++st;                                                                      \
            memcpy(F2, F, sizeof(T) * 2 * nn);                                         \
            for (int64_t i = 0; i + sh < n; ++i) {  /* G_i o G_{i+sh} */               \
                F[2 * i] = F2[2 * i] * F2[2 * (i + sh)];                               \
                F[2 * i + 1] = F2[2 * i] * F2[2 * (i + sh) + 1] + F2[2 * i + 1];       \
            }                                                                          \
        }                                                                              \
        ++st; /* evaluation: x_i = G_i.beta (the last map is constant) */              \
        for (int64_t i = 0; i < n; ++i) X[i] = F[2 * i + 1];                           \
    }                                                                                  \
    if (steps) *steps = st;                                                            \
    if (log_len) *log_len = Lg.len;                                                    \
    free(w);                                                                           \
    return 0;                                                                          \
}

#define DEFINE_ALL(T, SFX)  \
    DEFINE_THOMAS(T, SFX)   \
    DEFINE_CR_LEVELS(T, SFX) \
    DEFINE_LOAD(T, SFX)     \
    DEFINE_CR(T, SFX)       \
    DEFINE_PCR_CORE(T, SFX) \
    DEFINE_RD_CORE(T, SFX)  \
    DEFINE_HYBRID(T, SFX)   \
    DEFINE_STONE(T, SFX)

DEFINE_ALL(double, f64)
DEFINE_ALL(float, f32)

/* ---------------------------------------------------------------------- */
/* MT: the paper's multi-threaded CPU solver: several threads,  */
/* each solving whole systems with Thomas.  Contiguous system ranges.        */
/* Used only as bench.py's timed cpu_baseline.                               */
/* ---------------------------------------------------------------------- */
typedef struct {
    const void *a, *b, *c, *d;
    void* x;
    int64_t n, s0, s1;
    int f64;
} mt_job_t;

static void* mt_worker(void* p) {
    mt_job_t* j = (mt_job_t*)p;
    int64_t off = j->s0 * j->n, cnt = j->s1 - j->s0;
    if (j->f64)
        oracle_thomas_f64((const double*)j->a + off, (const double*)j->b + off,
                          (const double*)j->c + off, (const double*)j->d + off,
                          (double*)j->x + off, j->n, cnt);
    else
        oracle_thomas_f32((const float*)j->a + off, (const float*)j->b + off,
                          (const float*)j->c + off, (const float*)j->d + off,
                          (float*)j->x + off, j->n, cnt);
    return NULL;
}

static int thomas_mt(const void* a, const void* b, const void* c, const void* d, void* x,
                     int64_t n, int64_t S, int nthreads, int f64) {
    if (n < 1 || S < 0 || nthreads < 1) return -1;
    if (nthreads > 1024) nthreads = 1024;
    pthread_t th[1024];
    mt_job_t jobs[1024];
    for (int t = 0; t < nthreads; ++t) {
        jobs[t].a = a; jobs[t].b = b; jobs[t].c = c; jobs[t].d = d; jobs[t].x = x;
        jobs[t].n = n; jobs[t].f64 = f64;
        jobs[t].s0 = S * t / nthreads;
        jobs[t].s1 = S * (t + 1) / nthreads;
    }
    for (int t = 1; t < nthreads; ++t) pthread_create(&th[t], NULL, mt_worker, &jobs[t]);
    mt_worker(&jobs[0]);
    for (int t = 1; t < nthreads; ++t) pthread_join(th[t], NULL);
    return 0;
}

int oracle_thomas_mt_f64(const double* a, const double* b, const double* c,
                         const double* d, double* x, int64_t n, int64_t S, int nthreads) {
    return thomas_mt(a, b, c, d, x, n, S, nthreads, 1);
}
int oracle_thomas_mt_f32(const float* a, const float* b, const float* c, const float* d,
                         float* x, int64_t n, int64_t S, int nthreads) {
    return thomas_mt(a, b, c, d, x, n, S, nthreads, 0);
}

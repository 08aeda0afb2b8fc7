/*
 * oracle/thomas.c -- CPU fp64 Thomas algorithm.  TEST INFRASTRUCTURE ONLY.
 *
 * Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline /
 * --impl reference legs may load this library.  It shares no code, header,
 * table or helper with the CUDA path (paper_conf_ipps_davidsonzo11_b200/csrc).
 *
 * What it computes: the exact solution (up to fp64 rounding) of each of m
 * independent tridiagonal systems
 *      a_i x_{i-1} + b_i x_i + c_i x_{i+1} = d_i,   i = 0..n-1,
 * with a_0 and c_{n-1} ignored (taken as 0; reading R3).
 *
 * Source: the paper uses the Thomas algorithm as its serial O(n) stage
 * ("The Thomas algorithm is serial, requiring only O(n) total work, but with
 * O(n) steps", §III-A; stage 4 P:L511-512) without
 * printing it; this is the textbook form (Hockney & Jesshope [11]):
 *
 *   c'_0 = c_0 / b_0 ;  d'_0 = d_0 / b_0
 *   for i = 1..n-1:  w = b_i - a_i c'_{i-1};  c'_i = c_i / w;
 *                    d'_i = (d_i - a_i d'_{i-1}) / w
 *   x_{n-1} = d'_{n-1};  for i = n-2..0:  x_i = d'_i - c'_i x_{i+1}
 *
 * Compiled with -O2 -ffp-contract=off so every operation rounds as written.
 * Systems are independent; OpenMP runs one system per thread (the paper's MKL
 * baseline setup).  No pivoting: the precondition is a nonsingular
 * diagonally dominant system, as for the method under test.
 * Layout: element i of system s at ptr[s*stride + i].
 */
#include <stdint.h>
#include <stdlib.h>
#ifdef _OPENMP
#include <omp.h>
#endif

static void thomas_one(int64_t n, const double *a, const double *b, const double *c,
                       const double *d, double *x, double *cp, double *dp) {
    cp[0] = (n > 1 ? c[0] : 0.0) / b[0];
    dp[0] = d[0] / b[0];
    for (int64_t i = 1; i < n; ++i) {
        double ci = (i < n - 1) ? c[i] : 0.0;
        double w = b[i] - a[i] * cp[i - 1];
        cp[i] = ci / w;
        dp[i] = (d[i] - a[i] * dp[i - 1]) / w;
    }
    x[n - 1] = dp[n - 1];
    for (int64_t i = n - 2; i >= 0; --i) x[i] = dp[i] - cp[i] * x[i + 1];
}

/* Returns 0 on success, -1 on bad arguments, -2 on allocation failure. */
int oracle_thomas_f64(int64_t n, int64_t m, int64_t stride, const double *a,
                      const double *b, const double *c, const double *d, double *x,
                      int threads) {
    if (n < 1 || m < 0 || stride < n || !a || !b || !c || !d || !x) return -1;
    int status = 0;
#ifdef _OPENMP
    if (threads <= 0) threads = omp_get_max_threads();
#pragma omp parallel num_threads(threads)
#endif
    {
        double *cp = (double *)malloc(sizeof(double) * (size_t)n);
        double *dp = (double *)malloc(sizeof(double) * (size_t)n);
        int ok = (cp && dp);
        if (!ok) {
#ifdef _OPENMP
#pragma omp atomic write
#endif
            status = -2;
        }
#ifdef _OPENMP
#pragma omp for schedule(dynamic, 1)
#endif
        for (int64_t s = 0; s < m; ++s) {
            if (!ok) continue;
            int64_t o = s * stride;
            thomas_one(n, a + o, b + o, c + o, d + o, x + o, cp, dp);
        }
        free(cp);
        free(dp);
    }
    (void)threads;
    return status;
}

int oracle_num_threads(void) {
#ifdef _OPENMP
    return omp_get_max_threads();
#else
    return 1;
#endif
}

/* plan_and_solve.c -- the C ABI (include/tds.h) from plain C.
 *
 *   gcc -std=c11 -O2 examples/plan_and_solve.c -Iinclude -I/usr/local/cuda/include \
 *       -Lpaper_conf_ipps_davidsonzo11_b200 -ltds -L/usr/local/cuda/lib64 -lcudart -lm \
 *       -Wl,-rpath,$PWD/paper_conf_ipps_davidsonzo11_b200 -o plan_and_solve
 *   ./plan_and_solve
 *
 * Part 1 needs no GPU: STATIC plans for B200 properties (tds_plan_from_props)
 * and the canonical subsystem order of a small plan (Fig. 3a).
 * Part 2 runs when a CUDA device is present: m diagonally dominant systems
 * built on the host, copied to the device, tuned and solved with
 * tds_solve_batched, and the relative residual ||Ax - d|| / ||d|| checked on
 * the host in double precision.
 */
#include <cuda_runtime_api.h>
#include <math.h>
#include <stdint.h>
#include <stdio.h>
#include <stdlib.h>

#include "tds.h"

#define CHECK(call)                                                                      \
    do {                                                                                 \
        tds_status s_ = (call);                                                          \
        if (s_ != TDS_OK) {                                                              \
            fprintf(stderr, "%s: %s (%s)\n", #call, tds_status_string(s_), tds_last_error()); \
            return 1;                                                                    \
        }                                                                                \
    } while (0)

static int part1_plans(void) {
    /* B200: 148 SMs, 227 KB opt-in shared memory per block */
    const tds_device_props b200 = {148, 232448, 233472, 65536, 1024, 32, 10, 0, 126LL << 20, 180LL << 30};
    const int64_t shapes[4][2] = {{1024, 1}, {65536, 256}, {1 << 20, 16}, {16384, 4096}};
    for (int i = 0; i < 4; ++i) {
        tds_plan_t p;
        tds_plan_info info;
        CHECK(tds_plan_from_props(&p, &b200, TDS_F32, shapes[i][0], shapes[i][1], 0, TDS_PARAMS_STATIC));
        CHECK(tds_plan_info_get(p, &info));
        printf("STATIC n=%lld m=%lld: k=%d passes=%d n_sub=%lld subsystems=%lld workspace=%zu launches=%d\n",
               (long long)info.n, (long long)info.m, info.params.k, info.params.passes, (long long)info.n_sub,
               (long long)info.num_subsystems, info.workspace_bytes, info.launches);
        CHECK(tds_plan_destroy(p));
    }
    /* canonical order after k = 2 levels of an 8-row system: [0 4 1 5 2 6 3 7] */
    tds_plan_t p;
    tds_params prm;
    tds_plan_info info;
    int64_t perm[8];
    CHECK(tds_plan_from_props(&p, &b200, TDS_F32, 8, 1, 0, TDS_PARAMS_STATIC));
    CHECK(tds_plan_info_get(p, &info));
    prm = info.params;
    prm.k = 2;
    prm.passes = 1;
    prm.k_pass[0] = 2;
    CHECK(tds_plan_set_params(p, &prm));
    CHECK(tds_plan_permutation(p, perm, 8));
    printf("permutation n=8 k=2:");
    for (int i = 0; i < 8; ++i) printf(" %lld", (long long)perm[i]);
    printf("\n");
    CHECK(tds_plan_destroy(p));
    return 0;
}

static int part2_solve(void) {
    int ndev = 0;
    if (cudaGetDeviceCount(&ndev) != cudaSuccess || ndev < 1) {
        printf("no CUDA device: solve skipped\n");
        return 0;
    }
    const int64_t n = 100003, m = 3, N = n * m; /* ragged n: uneven subsystems */
    float *h[5];
    for (int q = 0; q < 5; ++q) h[q] = (float *)malloc(sizeof(float) * N);
    uint64_t z = 12345;
    for (int64_t e = 0; e < N; ++e) { /* diagonally dominant random rows, a_0 = c_{n-1} = 0 */
        float v[3];
        for (int q = 0; q < 3; ++q) {
            z = z * 6364136223846793005ULL + 1442695040888963407ULL;
            v[q] = (float)((double)(z >> 40) / (double)(1ULL << 24) * 2.0 - 1.0);
        }
        const int64_t i = e % n;
        h[0][e] = i > 0 ? v[0] : 0.f;
        h[2][e] = i < n - 1 ? v[1] : 0.f;
        h[3][e] = v[2];
        h[1][e] = fabsf(h[0][e]) + fabsf(h[2][e]) + 1.f;
    }
    void *d[5], *ws = NULL;
    for (int q = 0; q < 5; ++q) {
        if (cudaMalloc(&d[q], sizeof(float) * N) != cudaSuccess) return 1;
        if (q < 4) cudaMemcpy(d[q], h[q], sizeof(float) * N, cudaMemcpyHostToDevice);
    }
    tds_plan_t p;
    tds_plan_info info;
    CHECK(tds_plan(&p, 0, TDS_F32, n, m, 0, TDS_PARAMS_STATIC));
    CHECK(tds_tune(p, NULL, NULL)); /* optional: the self-tuned plan */
    CHECK(tds_plan_info_get(p, &info));
    if (info.workspace_bytes && cudaMalloc(&ws, info.workspace_bytes) != cudaSuccess) return 1;
    CHECK(tds_solve_batched(p, d[0], d[1], d[2], d[3], d[4], ws, info.workspace_bytes, NULL));
    if (cudaDeviceSynchronize() != cudaSuccess) return 1;
    cudaMemcpy(h[4], d[4], sizeof(float) * N, cudaMemcpyDeviceToHost);
    double rmax = 0, dmax = 0;
    for (int64_t e = 0; e < N; ++e) {
        const int64_t i = e % n;
        double r = (double)h[1][e] * h[4][e] - h[3][e];
        if (i > 0) r += (double)h[0][e] * h[4][e - 1];
        if (i < n - 1) r += (double)h[2][e] * h[4][e + 1];
        rmax = fmax(rmax, fabs(r));
        dmax = fmax(dmax, fabs((double)h[3][e]));
    }
    printf("tuned plan k=%d passes=%d onchip_form=%d; relative residual %.2e %s\n", info.params.k,
           info.params.passes, info.onchip_form, rmax / dmax, rmax / dmax <= 1e-5 ? "ok" : "FAILED");
    CHECK(tds_plan_destroy(p));
    for (int q = 0; q < 5; ++q) {
        cudaFree(d[q]);
        free(h[q]);
    }
    if (ws) cudaFree(ws);
    return rmax / dmax <= 1e-5 ? 0 : 1;
}

int main(void) {
    if (part1_plans()) return 1;
    return part2_solve();
}

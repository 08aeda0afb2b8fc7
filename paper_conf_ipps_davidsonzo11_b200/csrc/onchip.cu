// onchip.cu -- G2: the on-chip hybrid solver for one (sub)system per CTA.
//
// Paper: the base kernel is a hybrid PCR-Thomas solver that fetches each
// system into shared memory, splits it with PCR until there are enough
// independent subsystems, then solves each with the Thomas algorithm in one
// thread (§III-A, Fig. 3b; stages 3 and 4, §III-D
// P:L505-512).  The north_star asks for a hybrid CR/PCR solver; Zhang et
// al.'s CR-PCR hybrid is the paper's comparison point.
//
// B200 form: thread t owns R = 2^c CONSECUTIVE rows
// in registers.
//   A. load + normalise (b = 1) -- rows beyond the subsystem are identity rows;
//   B. c CR forward levels entirely in registers (stride 2^(l-1) within the
//      thread; only the last kept row needs one row of thread t+1, exchanged
//      through shared memory) -> one reduced row per thread;
//   C. the reduced system (blockDim rows, coupling stride R) in shared memory:
//      log2(T) PCR levels until T independent chains, then Thomas on each
//      chain by one thread (the paper's stage 3 -> 4 switch point T);
//   D. CR back substitution in registers, x written to original rows
//      r + 2^K j (index placement A4).
// c = 0 (R = 1) is exactly the paper's PCR-Thomas base kernel.
#include "common.cuh"

namespace tds {


template <typename T, int R, bool RAW>
__global__ void __launch_bounds__(R >= 8 ? 512 : 1024) onchip_kernel(const OnchipArgs<T> A) {
    extern __shared__ __align__(16) unsigned char smem_raw[];
    const int NT = blockDim.x;
    const int t = threadIdx.x;
    T *xch = reinterpret_cast<T *>(smem_raw);  // [2][3][NT+1]
    T *za = xch + 6 * (NT + 1);                // reduced system [3][NT]
    T *zc = za + NT;
    T *zd = zc + NT;

    const int64_t sigma = blockIdx.x;
    int64_t sys, r, L, in_base;
    if (RAW) {
        sys = sigma;
        r = 0;
        L = A.n;
        in_base = sys * A.batch_stride;
    } else {
        sys = sigma >> A.K;
        r = slot_residue(sigma & ((int64_t(1) << A.K) - 1), A.geom.npass, A.geom.kpass);
        if (r >= A.n) return;  // empty slot (2^K > n): uniform per CTA
        L = (A.n - r + (int64_t(1) << A.K) - 1) >> A.K;
        in_base = sigma * A.slot;
    }
    const int64_t out_base = sys * A.batch_stride + r;

    // ---- A. load R consecutive rows per thread, normalise
    T ra[R], rc[R], rd[R];
#pragma unroll
    for (int v = 0; v < R; ++v) {
        const int64_t j = int64_t(t) * R + v;
        ra[v] = T(0);
        rc[v] = T(0);
        rd[v] = T(0);
        if (j < L) {
            const int64_t o = in_base + j;
            if (RAW) {
                const T rb = rcp(A.b[o]);
                ra[v] = (j > 0 ? A.a[o] : T(0)) * rb;
                rc[v] = (j < L - 1 ? A.c[o] : T(0)) * rb;
                rd[v] = A.d[o] * rb;
            } else {
                ra[v] = A.a[o];
                rc[v] = A.c[o];
                rd[v] = A.d[o];
            }
        }
    }

    // ---- B. CR forward levels in registers
#pragma unroll
    for (int l = 1; (1 << l) <= R; ++l) {
        const int s = 1 << (l - 1);
        T *xb = xch + (l & 1) * 3 * (NT + 1);
        // publish row s-1 (kept at level l-1) for thread t-1
        xb[t] = ra[s - 1];
        xb[(NT + 1) + t] = rc[s - 1];
        xb[2 * (NT + 1) + t] = rd[s - 1];
        if (t == 0) {
            xb[NT] = T(0);
            xb[(NT + 1) + NT] = T(0);
            xb[2 * (NT + 1) + NT] = T(0);
        }
        __syncthreads();
        const T na = xb[t + 1], nc = xb[(NT + 1) + t + 1], nd = xb[2 * (NT + 1) + t + 1];
#pragma unroll
        for (int v = (1 << l) - 1; v < R; v += (1 << l)) {
            const T ar = (v + s < R) ? ra[(v + s) % R] : na;
            const T cr = (v + s < R) ? rc[(v + s) % R] : nc;
            const T dr = (v + s < R) ? rd[(v + s) % R] : nd;
            row_update(ra[v], rc[v], rd[v], ra[v - s], rc[v - s], rd[v - s], ar, cr, dr);
        }
    }

    // ---- C. reduced system: PCR until T chains, then Thomas per chain
    za[t] = ra[R - 1];
    zc[t] = rc[R - 1];
    zd[t] = rd[R - 1];
    __syncthreads();
    for (int j = 0; j < A.log2T; ++j) {
        const int s = 1 << j;
        T a = za[t], c = zc[t], d = zd[t];
        const T al = t >= s ? za[t - s] : T(0), cl = t >= s ? zc[t - s] : T(0), dl = t >= s ? zd[t - s] : T(0);
        const T ar = t + s < NT ? za[t + s] : T(0), cr = t + s < NT ? zc[t + s] : T(0),
                dr = t + s < NT ? zd[t + s] : T(0);
        row_update(a, c, d, al, cl, dl, ar, cr, dr);
        __syncthreads();
        za[t] = a;
        zc[t] = c;
        zd[t] = d;
        __syncthreads();
    }
    const int TC = 1 << A.log2T;
    if (t < TC && t < NT) {
        // Thomas on rows t, t+T, t+2T, ... (b = 1 after normalisation)
        T cp = zc[t], dp = zd[t];
        int q = t;
        for (int qn = t + TC; qn < NT; qn += TC) {
            const T aq = za[qn];
            const T w = rcp(fma(-aq, cp, T(1)));
            cp = zc[qn] * w;
            dp = (zd[qn] - aq * dp) * w;
            zc[qn] = cp;
            zd[qn] = dp;
            q = qn;
        }
        T xv = dp;  // x of the last chain row
        for (int qp = q - TC; qp >= t; qp -= TC) {
            xv = zd[qp] - zc[qp] * xv;
            zd[qp] = xv;
        }
    }
    __syncthreads();

    // ---- D. CR back substitution in registers, then write x
    T xs[R];
    xs[R - 1] = zd[t];
    const T xleft = t > 0 ? zd[t - 1] : T(0);
#pragma unroll
    for (int l = ilog2c(R); l >= 1; --l) {
        const int s = 1 << (l - 1);
#pragma unroll
        for (int v = s - 1; v < R - 1; v += 2 * s) {
            const T xl = (v >= s) ? xs[(v - s + R) % R] : xleft;
            xs[v] = rd[v] - ra[v] * xl - rc[v] * xs[(v + s) % R];
        }
    }
#pragma unroll
    for (int v = 0; v < R; ++v) {
        const int64_t j = int64_t(t) * R + v;
        if (j < L) A.x[out_base + (j << A.K)] = xs[v];
    }
}

template <typename T, int R>
static cudaError_t launch_r(const OnchipArgs<T> &A, bool raw, int64_t grid, int threads, size_t smem,
                            cudaStream_t st) {
    auto kern = raw ? onchip_kernel<T, R, true> : onchip_kernel<T, R, false>;
    cudaError_t e = cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    if (e != cudaSuccess) return e;
    kern<<<(unsigned)grid, threads, smem, st>>>(A);
    return cudaGetLastError();
}

template <typename T>
cudaError_t launch_onchip(const OnchipArgs<T> &A, int cr_levels, bool raw, int64_t grid, int threads,
                          size_t smem, cudaStream_t st) {
    switch (cr_levels) {
        case 0: return launch_r<T, 1>(A, raw, grid, threads, smem, st);
        case 1: return launch_r<T, 2>(A, raw, grid, threads, smem, st);
        case 2: return launch_r<T, 4>(A, raw, grid, threads, smem, st);
        case 3: return launch_r<T, 8>(A, raw, grid, threads, smem, st);
        case 4:
            if constexpr (sizeof(T) == 4) return launch_r<T, 16>(A, raw, grid, threads, smem, st);
            return cudaErrorInvalidConfiguration;
        default: return cudaErrorInvalidConfiguration;
    }
}

template cudaError_t launch_onchip<float>(const OnchipArgs<float> &, int, bool, int64_t, int, size_t, cudaStream_t);
template cudaError_t launch_onchip<double>(const OnchipArgs<double> &, int, bool, int64_t, int, size_t, cudaStream_t);

}  // namespace tds

// simt_chol.cuh — SIMT building blocks of the potrf and trsm tile tasks (reading R5).
//
// potrf (in place, lower):  A = L L^T.  Blocked right-looking:
//   for each nb-wide panel k0:  (1) potrf_diag: unblocked factorisation of the nb x nb
//   diagonal block in shared memory (IEEE sqrt / div), first non-positive pivot ->
//   *info (1-based, within the tile; R9);  (2) trsm_panel on the rows below;
//   (3) lower-only NT GEMM update of the trailing matrix (simt_gemm / tc kernels).
// trsm (right, lower, transposed, non-unit):  X L^T = B, X overwrites B.  Rows are
//   independent; column panels J: (1) trsm_panel: per-row forward substitution
//   x_j = (b_j - sum_{k<j} x_k L_jk) / L_jj  with L_JJ in shared memory; (2) NT GEMM
//   update of the remaining columns.
#pragma once
#include <cuda_runtime.h>
#include <stdint.h>

#include "kernels.hpp"

namespace vsk {

// Unblocked right-looking Cholesky of an NB x NB diagonal block at A (leading dim lda),
// computed in Tacc, lower triangle only.  One CTA.  k_base = global column of the block
// (for info).  Writes back only j <= i.
template <typename Tin, typename Tacc, int NB>
__global__ void __launch_bounds__(256) potrf_diag_kernel(Tin *A, int lda, int k_base, int *info)
{
    __shared__ Tacc a[NB][NB + 1];
    __shared__ int bad;
    const int tid = threadIdx.x;
    for (int e = tid; e < NB * NB; e += blockDim.x) {
        const int i = e / NB, j = e % NB;
        a[i][j] = j <= i ? (Tacc)A[(int64_t)i * lda + j] : (Tacc)0;
    }
    if (tid == 0) bad = 0;
    __syncthreads();
    for (int k = 0; k < NB; k++) {
        if (tid == 0) {
            const Tacc d = a[k][k];
            if (!(d > (Tacc)0)) {
                if (!bad) {
                    bad = 1;
                    if (info) atomicCAS(info, 0, k_base + k + 1);
                }
            }
            a[k][k] = sqrt(d);
        }
        __syncthreads();
        const Tacc lkk = a[k][k];
        for (int i = k + 1 + tid; i < NB; i += blockDim.x) a[i][k] = a[i][k] / lkk;
        __syncthreads();
        // trailing update a_ij -= a_ik * a_jk, k < j <= i
        const int rem = NB - k - 1;
        for (int e = tid; e < rem * rem; e += blockDim.x) {
            const int i = k + 1 + e / rem, j = k + 1 + e % rem;
            if (j <= i) a[i][j] = fma(-a[i][k], a[j][k], a[i][j]);
        }
        __syncthreads();
    }
    for (int e = tid; e < NB * NB; e += blockDim.x) {
        const int i = e / NB, j = e % NB;
        if (j <= i) A[(int64_t)i * lda + j] = (Tin)a[i][j];
    }
}

// Forward substitution of `rows` rows of X (leading dim ldx) against the NB x NB lower
// block L (leading dim ldl):  X <- X L^{-T}.  Each CTA owns 64 rows staged in smem.
template <typename Tin, typename Tacc, int NB>
__global__ void __launch_bounds__(64) trsm_panel_kernel(const Tin *L, int ldl, Tin *X, int ldx, int rows)
{
    __shared__ Tacc l[NB][NB + 1];
    __shared__ Tacc x[64][NB + 1];
    const int tid = threadIdx.x;
    const int r0 = blockIdx.x * 64;
    for (int e = tid; e < NB * NB; e += 64) {
        const int i = e / NB, j = e % NB;
        l[i][j] = j <= i ? (Tacc)L[(int64_t)i * ldl + j] : (Tacc)0;
    }
    for (int e = tid; e < 64 * NB; e += 64) {
        const int i = e / NB, j = e % NB;
        x[i][j] = (r0 + i < rows) ? (Tacc)X[(int64_t)(r0 + i) * ldx + j] : (Tacc)0;
    }
    __syncthreads();
    for (int j = 0; j < NB; j++) {
        Tacc s = x[tid][j];
        for (int k = 0; k < j; k++) s = fma(-x[tid][k], l[j][k], s);
        x[tid][j] = s / l[j][j];
    }
    __syncthreads();
    for (int e = tid; e < 64 * NB; e += 64) {
        const int i = e / NB, j = e % NB;
        if (r0 + i < rows) X[(int64_t)(r0 + i) * ldx + j] = (Tin)x[i][j];
    }
}

template <typename Tin, typename Tacc, int NB>
inline void potrf_diag(Tin *A, int lda, int k_base, int *info, cudaStream_t s)
{
    count_launch();
    potrf_diag_kernel<Tin, Tacc, NB><<<1, 256, 0, s>>>(A, lda, k_base, info);
}

template <typename Tin, typename Tacc, int NB>
inline void trsm_panel(const Tin *L, int ldl, Tin *X, int ldx, int rows, cudaStream_t s)
{
    if (rows <= 0) return;
    count_launch();
    trsm_panel_kernel<Tin, Tacc, NB><<<(rows + 63) / 64, 64, 0, s>>>(L, ldl, X, ldx, rows);
}

}  // namespace vsk

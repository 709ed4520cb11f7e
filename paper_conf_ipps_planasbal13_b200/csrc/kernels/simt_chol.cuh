// simt_chol.cuh — SIMT building blocks of the potrf and trsm tile tasks (reading R5).
//
// potrf_diag: unblocked right-looking Cholesky of an NB x NB
//   diagonal block, one CTA of NB threads; thread i keeps row i of the block in
//   registers; per column k: thread k publishes l_kk = sqrt(a_kk) (first non-positive
//   pivot -> *info, 1-based within the tile, R9), every thread i > k scales
//   l_ik = a_ik / l_kk and publishes it, then updates its row a_ij -= l_ik l_jk
//   (k < j <= i) from the published column: one barrier per column, IEEE sqrt/div.
// trsm_panel: X <- X L^{-T} for an NB-wide column panel (right, lower, transposed,
//   non-unit): each thread owns one row, forward substitution
//   x_j = (b_j - sum_{k<j} x_k L_jk) / L_jj with L_JJ staged in shared memory.
// Both stage their global tiles with fully unrolled, batched loads.
#pragma once
#include <cuda_runtime.h>
#include <stdint.h>

#include "kernels.hpp"
#include "task_ctx.cuh"

namespace vsk {

template <typename Tin, typename Tacc, int NB>
__global__ void __launch_bounds__(NB) potrf_diag_kernel(Tin *A, int lda, int k_base, int *info, TaskCtx ctx)
{
    ctx_begin(ctx);
    __shared__ Tacc col[2][NB];   // published column k (double-buffered by parity)
    __shared__ int bad;
    const int i = threadIdx.x;
    Tacc a[NB];
    // row i, lower part only (j <= i); batched loads
#pragma unroll
    for (int j = 0; j < NB; j++) a[j] = (j <= i) ? (Tacc)A[(int64_t)i * lda + j] : (Tacc)0;
    if (i == 0) bad = 0;
    __syncthreads();
#pragma unroll
    for (int k = 0; k < NB; k++) {
        if (i == k) {
            const Tacc d = a[k];
            if (!(d > (Tacc)0) && !bad) {
                bad = 1;
                if (info) atomicCAS(info, 0, k_base + k + 1);
            }
            a[k] = sqrt(d);
            col[k & 1][k] = a[k];
        }
        __syncthreads();
        const Tacc lkk = col[k & 1][k];
        if (i > k) {
            a[k] = a[k] / lkk;
            col[k & 1][i] = a[k];
        }
        __syncthreads();
        if (i > k) {
#pragma unroll
            for (int j = k + 1; j < NB; j++)
                if (j <= i) a[j] = fma(-a[k], col[k & 1][j], a[j]);
        }
        // buffer k&1 is rewritten at k+2, after every thread passed iteration k+1's barriers
    }
#pragma unroll
    for (int j = 0; j < NB; j++)
        if (j <= i) A[(int64_t)i * lda + j] = (Tin)a[j];
    ctx_end(ctx);
}

// Forward substitution of `rows` rows of X (leading dim ldx) against the NB x NB lower
// block L (leading dim ldl):  X <- X L^{-T}.  Each CTA owns 64 rows staged in smem.
template <typename Tin, typename Tacc, int NB>
__global__ void __launch_bounds__(64) trsm_panel_kernel(const Tin *L, int ldl, Tin *X, int ldx, int rows, TaskCtx ctx)
{
    ctx_begin(ctx);
    __shared__ Tacc l[NB][NB + 1];
    __shared__ Tacc x[64][NB + 1];
    const int tid = threadIdx.x;
    const int r0 = blockIdx.x * 64;
    constexpr int PER = NB * NB / 64;
    Tin tmp[PER];
#pragma unroll
    for (int q = 0; q < PER; q++) {
        const int e = tid + 64 * q, i = e / NB, j = e % NB;
        tmp[q] = j <= i ? L[(int64_t)i * ldl + j] : (Tin)0;
    }
#pragma unroll
    for (int q = 0; q < PER; q++) {
        const int e = tid + 64 * q, i = e / NB, j = e % NB;
        l[i][j] = (Tacc)tmp[q];
    }
    constexpr int PERX = NB;   // 64 rows x NB columns over 64 threads
    Tin tmx[PERX];
#pragma unroll
    for (int q = 0; q < PERX; q++) {
        const int e = tid + 64 * q, i = e / NB, j = e % NB;
        tmx[q] = (r0 + i < rows) ? X[(int64_t)(r0 + i) * ldx + j] : (Tin)0;
    }
#pragma unroll
    for (int q = 0; q < PERX; q++) {
        const int e = tid + 64 * q, i = e / NB, j = e % NB;
        x[i][j] = (Tacc)tmx[q];
    }
    __syncthreads();
    for (int j = 0; j < NB; j++) {
        Tacc s = x[tid][j];
        for (int k = 0; k < j; k++) s = fma(-x[tid][k], l[j][k], s);
        x[tid][j] = s / l[j][j];
    }
    __syncthreads();
#pragma unroll
    for (int q = 0; q < PERX; q++) {
        const int e = tid + 64 * q, i = e / NB, j = e % NB;
        if (r0 + i < rows) X[(int64_t)(r0 + i) * ldx + j] = (Tin)x[i][j];
    }
    ctx_end(ctx);
}

template <typename Tin, typename Tacc, int NB>
inline void potrf_diag(Tin *A, int lda, int k_base, int *info, cudaStream_t s, const TaskCtx &ctx)
{
    count_launch();
    potrf_diag_kernel<Tin, Tacc, NB><<<1, NB, 0, s>>>(A, lda, k_base, info, ctx);
}

template <typename Tin, typename Tacc, int NB>
inline void trsm_panel(const Tin *L, int ldl, Tin *X, int ldx, int rows, cudaStream_t s, const TaskCtx &ctx)
{
    if (rows <= 0) return;
    count_launch();
    auto kern = trsm_panel_kernel<Tin, Tacc, NB>;
    kern<<<(rows + 63) / 64, 64, 0, s>>>(L, ldl, X, ldx, rows, ctx_for(ctx, kern, 64, 0));
}

}  // namespace vsk

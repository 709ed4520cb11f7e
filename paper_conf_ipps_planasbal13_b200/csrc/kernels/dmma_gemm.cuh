// dmma_gemm.cuh — FP64 tensor-core tile GEMM (mma.sync.aligned.m8n8k4 .f64, "DMMA") for the
// dmma_f64 version (fp64 tiles) and the f64in_f32io version (fp32 tiles upcast to fp64 in
// shared memory, fp64 products and sums, ONE rounding to fp32 on store).
//
//   C[M x N] (ldc) = C + s * A[M x K] (lda) * op(B)      s = +1 / -1, op(B) = B or B^T
//
// tcgen05 has no f64 kind on sm_100a (ptxas rejects .kind::f64); the legacy
// DMMA path is the tensor-core FP64 route.  CTA tile 64 x 64, 4 warps (2 x 2), warp tile
// 32 x 32 = 4 x 4 m8n8 fragments, BK = 16; the accumulators start from C_in (converted to
// fp64) so the fp32 variant rounds once.  Fragment layouts of m8n8k4.f64 (row.col):
//   A (8x4): lane holds A[lane/4][lane%4];  B (4x8): B[lane%4][lane/4];
//   C (8x8): C[lane/4][2*(lane%4) + {0,1}].
// LOWER: tiles strictly above the diagonal exit; diagonal tiles store only j <= i.
#pragma once
#include <cuda_runtime.h>
#include <stdint.h>

#include "kernels.hpp"
#include "task_ctx.cuh"

namespace vsk {

__device__ __forceinline__ void dmma_8x8x4(double &d0, double &d1, double a, double b)
{
    asm volatile("mma.sync.aligned.m8n8k4.row.col.f64.f64.f64.f64 {%0,%1}, {%2}, {%3}, {%0,%1};"
                 : "+d"(d0), "+d"(d1)
                 : "d"(a), "d"(b));
}

template <typename Tin, bool NT, bool NEG, bool LOWER>
__global__ void __launch_bounds__(128) dmma_gemm_kernel(int M, int N, int K, const Tin *__restrict__ A, int lda,
                                                        const Tin *__restrict__ B, int ldb, Tin *__restrict__ C,
                                                        int ldc, TaskCtx ctx)
{
    ctx_begin(ctx);
    constexpr int BM = 64, BN = 64, BK = 16;
    __shared__ double As[BM][BK + 1];
    __shared__ double Bs[BK][BN + 1];
    const int m0 = blockIdx.y * BM, n0 = blockIdx.x * BN;
    if (LOWER && n0 >= m0 + BM) {
        ctx_end(ctx);
        return;
    }
    const int tid = threadIdx.x, warp = tid >> 5, lane = tid & 31;
    const int wm = (warp >> 1) * 32, wn = (warp & 1) * 32;
    const int g = lane >> 2, t = lane & 3;

    double acc[4][4][2];
#pragma unroll
    for (int i = 0; i < 4; i++)
#pragma unroll
        for (int j = 0; j < 4; j++)
#pragma unroll
            for (int e = 0; e < 2; e++) {
                const int r = m0 + wm + 8 * i + g, c = n0 + wn + 8 * j + 2 * t + e;
                acc[i][j][e] = (r < M && c < N) ? (double)C[(int64_t)r * ldc + c] : 0.0;
            }

    for (int k0 = 0; k0 < K; k0 += BK) {
        // stage A (BM x BK) and B (as BK x BN) in fp64
        for (int e = tid; e < BM * BK; e += 128) {
            const int r = e / BK, k = e % BK;
            As[r][k] = (m0 + r < M) ? (double)A[(int64_t)(m0 + r) * lda + k0 + k] : 0.0;
        }
        for (int e = tid; e < BN * BK; e += 128) {
            if (NT) {
                const int n = e / BK, k = e % BK;
                Bs[k][n] = (n0 + n < N) ? (double)B[(int64_t)(n0 + n) * ldb + k0 + k] : 0.0;
            } else {
                const int k = e / BN, n = e % BN;
                Bs[k][n] = (n0 + n < N) ? (double)B[(int64_t)(k0 + k) * ldb + n0 + n] : 0.0;
            }
        }
        __syncthreads();
#pragma unroll
        for (int kk = 0; kk < BK; kk += 4) {
            double a[4], b[4];
#pragma unroll
            for (int i = 0; i < 4; i++) a[i] = NEG ? -As[wm + 8 * i + g][kk + t] : As[wm + 8 * i + g][kk + t];
#pragma unroll
            for (int j = 0; j < 4; j++) b[j] = Bs[kk + t][wn + 8 * j + g];
#pragma unroll
            for (int i = 0; i < 4; i++)
#pragma unroll
                for (int j = 0; j < 4; j++) dmma_8x8x4(acc[i][j][0], acc[i][j][1], a[i], b[j]);
        }
        __syncthreads();
    }
#pragma unroll
    for (int i = 0; i < 4; i++)
#pragma unroll
        for (int j = 0; j < 4; j++)
#pragma unroll
            for (int e = 0; e < 2; e++) {
                const int r = m0 + wm + 8 * i + g, c = n0 + wn + 8 * j + 2 * t + e;
                if (r < M && c < N && (!LOWER || c <= r)) C[(int64_t)r * ldc + c] = (Tin)acc[i][j][e];
            }
    ctx_end(ctx);
}

template <typename Tin, bool NT, bool NEG, bool LOWER>
inline void dmma_gemm(int M, int N, int K, const Tin *A, int lda, const Tin *B, int ldb, Tin *C, int ldc,
                      cudaStream_t s, const TaskCtx &ctx)
{
    if (M <= 0 || N <= 0) return;
    dim3 grid((N + 63) / 64, (M + 63) / 64);
    count_launch();
    auto kern = dmma_gemm_kernel<Tin, NT, NEG, LOWER>;
    kern<<<grid, 128, 0, s>>>(M, N, K, A, lda, B, ldb, C, ldc, ctx_for(ctx, kern, 128, 0));
}

}  // namespace vsk

// simt_gemm.cuh — SIMT tile GEMM for the simt_f32 / f64in_f32io / dfma_f64 versions.
//
//   C[M x N] (ldc) = C -/+ A[M x K] (lda) * op(B)      op(B) = B (NN) or B^T (NT)
//
// Each output element is accumulated by ONE thread with a fused multiply-add in
// ascending k, starting from C_in: c = fma(+/-a_ik, b_kj, c).  In fp32 this is the
// per-element order of Fig 1's matmul_tile taken with fmaf,
// i.e. bit-identical to oracle_matmul_tiled_fmaf_f32 (pin P6).  Negating a is
// exact, so the "-=" forms are fma(-a, b, c) = round(c - a*b).
//
// Tin = storage type, Tacc = arithmetic type (f64in_f32io: float in, double math,
// one rounding on store).  Operand tiles are staged through shared memory with
// register double buffering (next k-tile loaded while the current one is consumed);
// A (and B in NT form) is transposed into k-major smem so each thread reads its
// TM rows / TN cols as 16-byte vectors; same-row threads of a warp read the same
// address (hardware broadcast).  LOWER: SYRK form — tiles strictly above the
// diagonal exit, diagonal tiles store only j <= i (strict upper untouched, R7).
#pragma once
#include <cuda_runtime.h>
#include <stdint.h>

#include "kernels.hpp"
#include "task_ctx.cuh"

namespace vsk {

template <typename T> struct Vec16;
template <> struct Vec16<float> { using type = float4; static constexpr int n = 4; };
template <> struct Vec16<double> { using type = double2; static constexpr int n = 2; };

template <typename Tin, typename Tacc, int BM, int BN, int BK, int TM, int TN, bool NT, bool NEG, bool LOWER>
__global__ void __launch_bounds__((BM / TM) * (BN / TN))
simt_gemm_kernel(int M, int N, int K, const Tin *__restrict__ A, int lda, const Tin *__restrict__ B, int ldb,
                 Tin *__restrict__ C, int ldc, TaskCtx ctx)
{
    ctx_begin(ctx);
    constexpr int NTH = (BM / TM) * (BN / TN);
    using V = typename Vec16<Tin>::type;
    constexpr int VN = Vec16<Tin>::n;
    constexpr int A_VECS = BM * BK / VN;             // vectors per A tile
    constexpr int B_VECS = BN * BK / VN;
    constexpr int A_PER = (A_VECS + NTH - 1) / NTH;
    constexpr int B_PER = (B_VECS + NTH - 1) / NTH;
    static_assert(A_VECS % NTH == 0 && B_VECS % NTH == 0, "tile/threads mismatch");

    __shared__ __align__(16) Tacc As[BK][BM + 4];
    __shared__ __align__(16) Tacc Bs[BK][BN + 4];

    const int m0 = blockIdx.y * BM, n0 = blockIdx.x * BN;
    if (LOWER && n0 >= m0 + BM) {                     // tile strictly above the diagonal
        ctx_end(ctx);
        return;
    }
    const int tid = threadIdx.x;
    const int tx = tid % (BN / TN), ty = tid / (BN / TN);

    // accumulators start from C_in (per-element order: C_in, then k = 0, 1, ...)
    Tacc acc[TM][TN];
#pragma unroll
    for (int i = 0; i < TM; i++)
#pragma unroll
        for (int j = 0; j < TN; j++) {
            const int r = m0 + ty * TM + i, c = n0 + tx * TN + j;
            acc[i][j] = (r < M && c < N) ? (Tacc)C[(int64_t)r * ldc + c] : (Tacc)0;
        }

    V ra[A_PER], rb[B_PER];
    auto load = [&](int k0) {
#pragma unroll
        for (int p = 0; p < A_PER; p++) {          // A tile: BM rows x BK (k contiguous)
            const int v = tid + p * NTH;
            const int r = v / (BK / VN), kc = (v % (BK / VN)) * VN;
            const int gr = m0 + r;
            if (gr < M) ra[p] = *reinterpret_cast<const V *>(A + (int64_t)gr * lda + k0 + kc);
            else ra[p] = V{};
        }
#pragma unroll
        for (int p = 0; p < B_PER; p++) {
            const int v = tid + p * NTH;
            if (NT) {                                // B stored N x K: rows n, k contiguous
                const int r = v / (BK / VN), kc = (v % (BK / VN)) * VN;
                const int gn = n0 + r;
                if (gn < N) rb[p] = *reinterpret_cast<const V *>(B + (int64_t)gn * ldb + k0 + kc);
                else rb[p] = V{};
            } else {                                 // B stored K x N: rows k, n contiguous
                const int kr = v / (BN / VN), nc = (v % (BN / VN)) * VN;
                const int gn = n0 + nc;
                if (gn < N) rb[p] = *reinterpret_cast<const V *>(B + (int64_t)(k0 + kr) * ldb + gn);
                else rb[p] = V{};
            }
        }
    };
    auto store = [&]() {
#pragma unroll
        for (int p = 0; p < A_PER; p++) {
            const int v = tid + p * NTH;
            const int r = v / (BK / VN), kc = (v % (BK / VN)) * VN;
            const Tin *e = reinterpret_cast<const Tin *>(&ra[p]);
#pragma unroll
            for (int q = 0; q < VN; q++) As[kc + q][r] = (Tacc)e[q];
        }
#pragma unroll
        for (int p = 0; p < B_PER; p++) {
            const int v = tid + p * NTH;
            const Tin *e = reinterpret_cast<const Tin *>(&rb[p]);
            if (NT) {
                const int r = v / (BK / VN), kc = (v % (BK / VN)) * VN;
#pragma unroll
                for (int q = 0; q < VN; q++) Bs[kc + q][r] = (Tacc)e[q];
            } else {
                const int kr = v / (BN / VN), nc = (v % (BN / VN)) * VN;
#pragma unroll
                for (int q = 0; q < VN; q++) Bs[kr][nc + q] = (Tacc)e[q];
            }
        }
    };

    load(0);
    for (int k0 = 0; k0 < K; k0 += BK) {
        store();
        __syncthreads();
        if (k0 + BK < K) load(k0 + BK);              // prefetch next k-tile into registers
#pragma unroll
        for (int kk = 0; kk < BK; kk++) {
            Tacc a[TM], b[TN];
#pragma unroll
            for (int i = 0; i < TM; i++) a[i] = As[kk][ty * TM + i];
#pragma unroll
            for (int j = 0; j < TN; j++) b[j] = Bs[kk][tx * TN + j];
#pragma unroll
            for (int i = 0; i < TM; i++)
#pragma unroll
                for (int j = 0; j < TN; j++) acc[i][j] = fma(NEG ? -a[i] : a[i], b[j], acc[i][j]);
        }
        __syncthreads();
    }

#pragma unroll
    for (int i = 0; i < TM; i++)
#pragma unroll
        for (int j = 0; j < TN; j++) {
            const int r = m0 + ty * TM + i, c = n0 + tx * TN + j;
            if (r < M && c < N && (!LOWER || c <= r)) C[(int64_t)r * ldc + c] = (Tin)acc[i][j];
        }
    ctx_end(ctx);
}

// Host launcher.  K must be a multiple of BK (16); lda/ldb and the k offsets must keep
// 16-byte alignment (tile sizes are multiples of 32 elements).
template <typename Tin, typename Tacc, bool NT, bool NEG, bool LOWER>
inline void simt_gemm(int M, int N, int K, const Tin *A, int lda, const Tin *B, int ldb, Tin *C, int ldc,
                      cudaStream_t s, const TaskCtx &ctx)
{
    if (M <= 0 || N <= 0) return;
    constexpr bool WIDE = sizeof(Tacc) == 4;           // fp32 math: 128x128 tiles, 8x8 per thread
    constexpr int BM = WIDE ? 128 : 64, BN = WIDE ? 128 : 64, BK = 16, TM = WIDE ? 8 : 4, TN = WIDE ? 8 : 4;
    dim3 grid((N + BN - 1) / BN, (M + BM - 1) / BM);
    count_launch();
    auto kern = simt_gemm_kernel<Tin, Tacc, BM, BN, BK, TM, TN, NT, NEG, LOWER>;
    constexpr int threads = (BM / TM) * (BN / TN);
    kern<<<grid, threads, 0, s>>>(M, N, K, A, lda, B, ldb, C, ldc, ctx_for(ctx, kern, threads, 0));
}

}  // namespace vsk

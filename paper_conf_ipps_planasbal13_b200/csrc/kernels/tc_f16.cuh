// tc_f16.cuh — tcgen05 3xFP16 tile GEMM on pre-split operands (version tc_3xf16), sm_100a.
//
//   C[M x N] (ldc) = C + s * A[M x K] * B'[N x K]^T,  s = +1 (matmul) or -1 (Cholesky gemm /
//   syrk), where A and B' are given in the SPLIT FORM below (B' = B^T for the matmul's NN
//   operand, = B for the NT operands of gemm / syrk).
//
// Split form of an R x K fp32 operand X (one row = one K-major vector, reading R30):
//   every row r is scaled by a power of two 2^e_r that brings max_k |x_rk| into
//   [2^14, 2^15) (e_r = 0 for an all-zero or non-finite row), and each scaled element
//   x' = x * 2^e_r is written as two fp16 halves: big = rn_f16(x'), small = rn_f16(x' - big).
//   |x' - big - small| <= 2^-22 |x'| + 2^-25 (the absolute term is fp16's subnormal
//   spacing, i.e. <= 2^-39 of the row maximum), so the pair carries ~22 significant bits,
//   the same as 3xTF32's big/small, and fp16's range problem is removed by the row scale.
//   D = Ab*Bb + Ab*Bs + As*Bb is accumulated by three tcgen05.mma.kind::f16 per 16-wide
//   k-step (the dropped As*Bs term is < 2^-22 |a||b|), and the epilogue multiplies by
//   2^-e_A(i) * 2^-e_B(j) (exact) and adds C_in in fp32 round-to-nearest.
//   kind::f16 runs at twice the tf32 rate, so the 3-product scheme has twice the
//   tensor-pipe ceiling of 3xTF32.
//
// Byte layout (Rp = R rounded up to 256, rows >= R are zero; K a multiple of 64):
//   for each k-block kb of 64 columns: [big: Rp rows x 128 B][small: Rp rows x 128 B], each
//   part in the UMMA canonical K-major SWIZZLE_128B layout (8-row atoms of 1024 B, 16-byte
//   chunk index XOR (row & 7)); after the Rp*K*4 bytes: float inv_scale[Rp] = 2^-e_r.
//   A 128-row slice of one part for one k-block is therefore one contiguous 16 KB block, so
//   the GEMM feeds shared memory with plain bulk copies (cp.async.bulk, the TMA engine's 1-D
//   mode): no tensor map, no register traffic, no per-task conversion.
//
// GEMM structure (one 128 x 256 output tile per CTA, cta_group::1, UMMA M=128, N=256):
//   warp 0      lane 0 issues the bulk copies of a stage (A big/small 16 KB each, B
//               big/small 32 KB each) onto the stage's full barrier (expect_tx).
//   warp 1      TMEM allocator (512 columns) + MMA issuer: 4 k-steps x 3 MMAs per stage,
//               tcgen05.commit -> empty[s]; after the last stage -> acc_full.
//   warps 2-9   C_in staged into TMEM columns [256, 512) during the main loop; epilogue:
//               tcgen05.ld acc and C_in, C = C_in + acc * 2^-eA(i) * 2^-eB(j), vector stores.
// LOWER (syrk): CTAs strictly above the diagonal exit; diagonal tiles store only j <= i.
#pragma once
#include <cuda_fp16.h>
#include <cuda_runtime.h>
#include <stdint.h>
#include <stdlib.h>

#include "kernels.hpp"
#include "task_ctx.cuh"
#include "tc_gemm.cuh"

namespace vsk {
namespace tcf {

using tc::fence_proxy_async;
using tc::make_desc;
using tc::mbar_arrive;
using tc::mbar_init;
using tc::mbar_wait;
using tc::smem_u32;
using tc::tc_fence_after;
using tc::tc_fence_before;
using tc::tmem_ld32;
using tc::tmem_st32;

constexpr int BM = 128, BN = 256, BK = 64;   // BK in fp16 elements (one 128-byte swizzled row)
constexpr int STAGES = 2;
constexpr int A_BYTES = BM * BK * 2;          // 16 KB per part
constexpr int B_BYTES = BN * BK * 2;          // 32 KB per part
constexpr int STAGE = 2 * A_BYTES + 2 * B_BYTES;
constexpr int NEPI = 256;                     // epilogue threads (warps 2-9)
constexpr int NTHREADS = 64 + NEPI;
constexpr int SMEM = STAGES * STAGE + 1024 /*align*/ + 256 /*barriers*/;

__host__ __device__ inline int split_rows_padded(int R) { return (R + 255) / 256 * 256; }
__host__ __device__ inline size_t split_bytes(int R, int K)
{
    const size_t Rp = (size_t)split_rows_padded(R);
    return Rp * (size_t)K * 4 + Rp * 4;
}
// byte offset of the 16-byte chunk holding elements (r, 8c .. 8c+7) of the big part
__host__ __device__ inline size_t split_chunk_off(int Rp, int r, int c)
{
    const int kb = c >> 3, kc = c & 7;
    return (size_t)kb * Rp * 256 + (size_t)(r >> 3) * 1024 + (r & 7) * 128 + ((kc ^ (r & 7)) << 4);
}

// Row scale exponent: max * 2^e in [2^14, 2^15).
__device__ __forceinline__ int row_exponent(float m)
{
    if (!(m > 0.f) || !isfinite(m)) return 0;
    int x;
    frexpf(m, &x);   // m = f * 2^x, f in [0.5, 1)
    int e = 15 - x;
    return e > 126 ? 126 : e;
}

__device__ __forceinline__ uint32_t pack_h2(__half lo, __half hi)
{
    return (uint32_t)__half_as_ushort(lo) | ((uint32_t)__half_as_ushort(hi) << 16);
}

// 8 scaled values -> (big chunk, small chunk)
__device__ __forceinline__ void split8(const float (&v)[8], float sc, uint4 &big, uint4 &small)
{
    __half hb[8], hs[8];
#pragma unroll
    for (int i = 0; i < 8; i++) {
        const float s = v[i] * sc;   // sc = 2^e, exact
        hb[i] = __float2half_rn(s);
        hs[i] = __float2half_rn(s - __half2float(hb[i]));
    }
    big = make_uint4(pack_h2(hb[0], hb[1]), pack_h2(hb[2], hb[3]), pack_h2(hb[4], hb[5]), pack_h2(hb[6], hb[7]));
    small = make_uint4(pack_h2(hs[0], hs[1]), pack_h2(hs[2], hs[3]), pack_h2(hs[4], hs[5]), pack_h2(hs[6], hs[7]));
}

// Row form of an R x K row-major fp32 matrix (ld): one warp per (padded) row.
__global__ void __launch_bounds__(256) split_rows_kernel(const float *__restrict__ X, int R, int K, int ld,
                                                         uint8_t *__restrict__ out)
{
    const int Rp = split_rows_padded(R);
    const int r = blockIdx.x * 8 + (threadIdx.x >> 5), lane = threadIdx.x & 31;
    if (r >= Rp) return;
    const float *row = X + (int64_t)r * ld;
    float m = 0.f;
    if (r < R) {
        for (int k = 8 * lane; k < K; k += 256) {
            const float4 a = __ldg(reinterpret_cast<const float4 *>(row + k));
            const float4 b = __ldg(reinterpret_cast<const float4 *>(row + k + 4));
            m = fmaxf(m, fmaxf(fmaxf(fabsf(a.x), fabsf(a.y)), fmaxf(fabsf(a.z), fabsf(a.w))));
            m = fmaxf(m, fmaxf(fmaxf(fabsf(b.x), fabsf(b.y)), fmaxf(fabsf(b.z), fabsf(b.w))));
        }
#pragma unroll
        for (int o = 16; o; o >>= 1) m = fmaxf(m, __shfl_xor_sync(0xffffffffu, m, o));
    }
    const int e = row_exponent(m);
    const float sc = ldexpf(1.f, e);
    const size_t half = (size_t)Rp * 128;
    for (int k = 8 * lane; k < K; k += 256) {
        float v[8] = {0.f, 0.f, 0.f, 0.f, 0.f, 0.f, 0.f, 0.f};
        if (r < R) {
            const float4 a = __ldg(reinterpret_cast<const float4 *>(row + k));
            const float4 b = __ldg(reinterpret_cast<const float4 *>(row + k + 4));
            v[0] = a.x; v[1] = a.y; v[2] = a.z; v[3] = a.w; v[4] = b.x; v[5] = b.y; v[6] = b.z; v[7] = b.w;
        }
        uint4 big, small;
        split8(v, sc, big, small);
        const size_t off = split_chunk_off(Rp, r, k >> 3);
        *reinterpret_cast<uint4 *>(out + off) = big;
        *reinterpret_cast<uint4 *>(out + off + half) = small;
    }
    if (lane == 0) reinterpret_cast<float *>(out + (size_t)Rp * K * 4)[r] = ldexpf(1.f, -e);
}

// Row form of X^T for a K x R row-major fp32 matrix X (ld): form row r = column r of X.
// One CTA per 32 columns: pass 1 = column maxima, pass 2 = 64 x 32 blocks transposed
// through shared memory, 16-byte stores of 8 consecutive k per thread.
__global__ void __launch_bounds__(256) split_cols_kernel(const float *__restrict__ X, int K, int R, int ld,
                                                         uint8_t *__restrict__ out)
{
    __shared__ float tile[64][33];
    __shared__ float cmax[8][32];
    __shared__ int cexp[32];
    const int Rp = split_rows_padded(R);
    const int r0 = blockIdx.x * 32, w = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int col = r0 + lane;
    float m = 0.f;
    if (col < R)
        for (int k = w; k < K; k += 8) m = fmaxf(m, fabsf(__ldg(X + (int64_t)k * ld + col)));
    cmax[w][lane] = m;
    __syncthreads();
    if (w == 0) {
        float mm = cmax[0][lane];
#pragma unroll
        for (int i = 1; i < 8; i++) mm = fmaxf(mm, cmax[i][lane]);
        const int e = row_exponent(mm);
        cexp[lane] = e;
        if (col < Rp) reinterpret_cast<float *>(out + (size_t)Rp * K * 4)[col] = ldexpf(1.f, -e);
    }
    __syncthreads();
    const size_t half = (size_t)Rp * 128;
    const int rr = threadIdx.x >> 3, kc = threadIdx.x & 7;   // form row r0+rr, chunk kc of the block
    const float sc = ldexpf(1.f, cexp[rr]);
    for (int k0 = 0; k0 < K; k0 += 64) {
#pragma unroll
        for (int i = 0; i < 8; i++) {
            const int k = k0 + w * 8 + i;
            tile[w * 8 + i][lane] = (col < R) ? __ldg(X + (int64_t)k * ld + col) : 0.f;
        }
        __syncthreads();
        if (r0 + rr < Rp) {
            float v[8];
#pragma unroll
            for (int i = 0; i < 8; i++) v[i] = tile[kc * 8 + i][rr];
            uint4 big, small;
            split8(v, sc, big, small);
            const size_t off = split_chunk_off(Rp, r0 + rr, (k0 >> 3) + kc);
            *reinterpret_cast<uint4 *>(out + off) = big;
            *reinterpret_cast<uint4 *>(out + off + half) = small;
        }
        __syncthreads();
    }
}

__device__ __forceinline__ void mbar_expect_tx(uint64_t *bar, uint32_t bytes)
{
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes) : "memory");
}
__device__ __forceinline__ void bulk_g2s(uint32_t dst, const void *src, uint32_t bytes, uint64_t *bar)
{
    asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(dst),
                 "l"(src), "r"(bytes), "r"(smem_u32(bar))
                 : "memory");
}

// Instruction descriptor, kind::f16: D f32 (bit 4), A/B f16 (format 0), negate A (bit 13),
// K-major A and B, N>>3 at 17, M>>4 at 24.
__host__ __device__ constexpr uint32_t make_idesc_f16(int M, int N, bool negA)
{
    return (1u << 4) | ((negA ? 1u : 0u) << 13) | ((uint32_t)(N >> 3) << 17) | ((uint32_t)(M >> 4) << 24);
}

__device__ __forceinline__ void mma_f16(uint32_t tmem_d, uint64_t adesc, uint64_t bdesc, uint32_t idesc, uint32_t acc)
{
    asm volatile(
        "{\n\t.reg .pred p;\n\t"
        "setp.ne.b32 p, %4, 0;\n\t"
        "tcgen05.mma.cta_group::1.kind::f16 [%0], %1, %2, %3, p;\n\t}" ::"r"(tmem_d),
        "l"(adesc), "l"(bdesc), "r"(idesc), "r"(acc));
}

template <bool NEG, bool LOWER>
__global__ void __launch_bounds__(NTHREADS, 1)
tcf_gemm_kernel(int M, int N, int K, const uint8_t *__restrict__ As, const uint8_t *__restrict__ Bs,
                float *__restrict__ C, int ldc, TaskCtx ctx)
{
    ctx_begin(ctx);
    extern __shared__ uint8_t smem_raw[];
    uint8_t *smem = smem_raw + ((1024u - (smem_u32(smem_raw) & 1023u)) & 1023u);
    uint64_t *full = (uint64_t *)(smem + STAGES * STAGE);
    uint64_t *empty = full + STAGES;
    uint64_t *acc_full = empty + STAGES;
    uint32_t *tmem_slot = (uint32_t *)(acc_full + 1);

    const int m0 = blockIdx.y * BM, n0 = blockIdx.x * BN;
    if (LOWER && n0 >= m0 + BM) {
        ctx_end(ctx);
        return;
    }
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int nk = K / BK;
    const int RA = split_rows_padded(M), RB = split_rows_padded(N);

    if (threadIdx.x == 0) {
        for (int s = 0; s < STAGES; s++) {
            mbar_init(&full[s], 1);
            mbar_init(&empty[s], 1);
        }
        mbar_init(acc_full, 1);
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    if (warp == 1) {
        asm volatile("tcgen05.alloc.cta_group::1.sync.aligned.shared::cta.b32 [%0], %1;" ::"r"(smem_u32(tmem_slot)),
                     "r"(512u));
        asm volatile("tcgen05.relinquish_alloc_permit.cta_group::1.sync.aligned;");
    }
    tc_fence_before();
    __syncthreads();
    tc_fence_after();
    const uint32_t tmem = *tmem_slot;

    if (warp == 0) {
        // ------------------------------------------------------------ bulk-copy producer
        if (lane == 0) {
            for (int kb = 0; kb < nk; kb++) {
                const int s = kb % STAGES;
                if (kb >= STAGES) mbar_wait(&empty[s], ((kb / STAGES) - 1) & 1);
                const uint32_t st = smem_u32(smem + s * STAGE);
                mbar_expect_tx(&full[s], STAGE);
                const uint8_t *a = As + (size_t)kb * RA * 256 + (size_t)m0 * 128;
                const uint8_t *b = Bs + (size_t)kb * RB * 256 + (size_t)n0 * 128;
                bulk_g2s(st, a, A_BYTES, &full[s]);
                bulk_g2s(st + A_BYTES, a + (size_t)RA * 128, A_BYTES, &full[s]);
                bulk_g2s(st + 2 * A_BYTES, b, B_BYTES, &full[s]);
                bulk_g2s(st + 2 * A_BYTES + B_BYTES, b + (size_t)RB * 128, B_BYTES, &full[s]);
            }
        }
        __syncwarp();
    } else if (warp == 1) {
        // ------------------------------------------------------------ MMA issuer
        constexpr uint32_t idesc = make_idesc_f16(BM, BN, NEG);
        for (int kb = 0; kb < nk; kb++) {
            const int s = kb % STAGES;
            mbar_wait(&full[s], (kb / STAGES) & 1);
            tc_fence_after();
            if (lane == 0) {
                const uint32_t a_big = smem_u32(smem + s * STAGE), a_small = a_big + A_BYTES;
                const uint32_t b_big = a_big + 2 * A_BYTES, b_small = b_big + B_BYTES;
#pragma unroll
                for (int kk = 0; kk < BK / 16; kk++) {
                    const uint32_t o = kk * 32;   // 16 fp16 = 32 B inside the 128 B swizzled row
                    const uint64_t dAb = make_desc(a_big + o, 16, 1024), dAs = make_desc(a_small + o, 16, 1024);
                    const uint64_t dBb = make_desc(b_big + o, 16, 1024), dBs = make_desc(b_small + o, 16, 1024);
                    const uint32_t first = (kb == 0 && kk == 0) ? 0u : 1u;
                    mma_f16(tmem, dAb, dBb, idesc, first);
                    mma_f16(tmem, dAb, dBs, idesc, 1u);
                    mma_f16(tmem, dAs, dBb, idesc, 1u);
                }
                tc::mma_commit(&empty[s]);
                if (kb == nk - 1) tc::mma_commit(acc_full);
            }
            __syncwarp();
        }
    } else {
        // ------------------------------------------------------------ C_in staging + epilogue
        const int eq = warp & 3, eh = (warp - 2) >> 2;   // TMEM lane quarter, column half
        const int erow = m0 + eq * 32 + lane;
        const float4 z4 = make_float4(0.f, 0.f, 0.f, 0.f);
#pragma unroll 1
        for (int c = 0; c < BN / 64; c++) {
            const int col0 = eh * (BN / 2) + c * 32;
            float v[32];
            const float *crow = C + (int64_t)erow * ldc + n0 + col0;
#pragma unroll
            for (int j = 0; j < 8; j++) {
                const float4 x = (erow < M && n0 + col0 + 4 * j < N) ? *reinterpret_cast<const float4 *>(crow + 4 * j) : z4;
                v[4 * j] = x.x; v[4 * j + 1] = x.y; v[4 * j + 2] = x.z; v[4 * j + 3] = x.w;
            }
            tmem_st32(tmem + ((uint32_t)(eq * 32) << 16) + (uint32_t)(BN + col0), v);
        }
        asm volatile("tcgen05.wait::st.sync.aligned;" ::: "memory");
        const float sa = erow < RA ? __ldg(reinterpret_cast<const float *>(As + (size_t)RA * K * 4) + erow) : 0.f;
        const float *sbv = reinterpret_cast<const float *>(Bs + (size_t)RB * K * 4) + n0;

        mbar_wait(acc_full, 0);
        tc_fence_after();
#pragma unroll 1
        for (int c = 0; c < BN / 64; c++) {
            const int col0 = eh * (BN / 2) + c * 32;
            float v[32], cv[32];
            tmem_ld32(tmem + ((uint32_t)(eq * 32) << 16) + (uint32_t)col0, v);
            tmem_ld32(tmem + ((uint32_t)(eq * 32) << 16) + (uint32_t)(BN + col0), cv);
#pragma unroll
            for (int j = 0; j < 8; j++) {
                const float4 sb = __ldg(reinterpret_cast<const float4 *>(sbv + col0) + j);
                v[4 * j + 0] = cv[4 * j + 0] + (v[4 * j + 0] * sa) * sb.x;
                v[4 * j + 1] = cv[4 * j + 1] + (v[4 * j + 1] * sa) * sb.y;
                v[4 * j + 2] = cv[4 * j + 2] + (v[4 * j + 2] * sa) * sb.z;
                v[4 * j + 3] = cv[4 * j + 3] + (v[4 * j + 3] * sa) * sb.w;
            }
            if (erow < M) {
                float *crow = C + (int64_t)erow * ldc + n0 + col0;
#pragma unroll
                for (int j = 0; j < 8; j++) {
                    const int col = n0 + col0 + 4 * j;
                    if (col >= N) break;
                    if (LOWER && col + 3 > erow) {
                        if (col + 0 <= erow) crow[4 * j + 0] = v[4 * j + 0];
                        if (col + 1 <= erow) crow[4 * j + 1] = v[4 * j + 1];
                        if (col + 2 <= erow) crow[4 * j + 2] = v[4 * j + 2];
                    } else {
                        *reinterpret_cast<float4 *>(crow + 4 * j) =
                            make_float4(v[4 * j + 0], v[4 * j + 1], v[4 * j + 2], v[4 * j + 3]);
                    }
                }
            }
        }
    }

    tc_fence_before();
    __syncthreads();
    if (warp == 1) {
        tc_fence_after();
        asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, %1;" ::"r"(tmem), "r"(512u));
    }
    ctx_end(ctx);
}

// ---------------------------------------------------------------- CTA-pair variant
// A cluster of two CTAs computes a 256 x 256 output tile with UMMA M=256, N=256
// (cta_group::2): CTA r stages rows [128r, 128r+128) of A and rows [128r, 128r+128) of the
// pair's B' slice in ITS shared memory (bulk copies onto its own full[s]); a relay thread
// of each CTA then arrives on the LEADER's pfull[s] (count 2); the leader issues the MMAs,
// which read both CTAs' operands, and tcgen05.commit multicasts empty[s] to both CTAs.
// Per SM and per 64-wide k-block this stages 64 KB (vs 96 KB for one CTA at 128 x 256):
// 42 B/clk of L2 traffic at the MMA rate instead of 64 (the L2 delivers ~42 B/clk/SM).
constexpr int P_STAGES = 3;
constexpr int P_A_BYTES = 128 * BK * 2;    // 16 KB per part (this CTA's 128 rows of A)
constexpr int P_B_BYTES = 128 * BK * 2;    // 16 KB per part (this CTA's 128 rows of B')
constexpr int P_STAGE = 2 * P_A_BYTES + 2 * P_B_BYTES;
constexpr int P_SMEM = P_STAGES * P_STAGE + 1024 + 256;

__device__ __forceinline__ uint32_t cluster_rank()
{
    uint32_t r;
    asm volatile("mov.u32 %0, %%cluster_ctarank;" : "=r"(r));
    return r;
}
__device__ __forceinline__ void cluster_sync()
{
    asm volatile("barrier.cluster.arrive.release.aligned;\n\tbarrier.cluster.wait.acquire.aligned;" ::: "memory");
}
__device__ __forceinline__ void mbar_arrive_cluster(uint64_t *bar, uint32_t target)
{
    uint32_t remote;
    asm volatile("mapa.shared::cluster.u32 %0, %1, %2;" : "=r"(remote) : "r"(smem_u32(bar)), "r"(target));
    asm volatile("mbarrier.arrive.release.cluster.shared::cluster.b64 _, [%0];" ::"r"(remote) : "memory");
}
__device__ __forceinline__ void mbar_wait_cluster(uint64_t *bar, uint32_t parity)
{
    asm volatile(
        "{\n\t.reg .pred P1;\n"
        "WAIT_%=:\n\t"
        "mbarrier.try_wait.parity.acquire.cluster.shared::cta.b64 P1, [%0], %1;\n\t"
        "@P1 bra DONE_%=;\n\t"
        "bra WAIT_%=;\n"
        "DONE_%=:\n\t}" ::"r"(smem_u32(bar)),
        "r"(parity)
        : "memory");
}
__device__ __forceinline__ void mma_f16_pair(uint32_t tmem_d, uint64_t adesc, uint64_t bdesc, uint32_t idesc, uint32_t acc)
{
    asm volatile(
        "{\n\t.reg .pred p;\n\t"
        "setp.ne.b32 p, %4, 0;\n\t"
        "tcgen05.mma.cta_group::2.kind::f16 [%0], %1, %2, %3, p;\n\t}" ::"r"(tmem_d),
        "l"(adesc), "l"(bdesc), "r"(idesc), "r"(acc));
}
__device__ __forceinline__ void mma_commit_pair(uint64_t *bar)
{
    asm volatile(
        "tcgen05.commit.cta_group::2.mbarrier::arrive::one.shared::cluster.multicast::cluster.b64 [%0], %1;" ::"r"(
            smem_u32(bar)),
        "h"((uint16_t)0x3)
        : "memory");
}

template <bool NEG, bool LOWER>
__global__ void __cluster_dims__(2, 1, 1) __launch_bounds__(NTHREADS, 1)
tcf_gemm2_kernel(int M, int N, int K, const uint8_t *__restrict__ As, const uint8_t *__restrict__ Bs,
                 float *__restrict__ C, int ldc, TaskCtx ctx)
{
    ctx_begin(ctx);
    extern __shared__ uint8_t smem_raw[];
    uint8_t *smem = smem_raw + ((1024u - (smem_u32(smem_raw) & 1023u)) & 1023u);
    uint64_t *full = (uint64_t *)(smem + P_STAGES * P_STAGE);
    uint64_t *pfull = full + P_STAGES;
    uint64_t *empty = pfull + P_STAGES;
    uint64_t *acc_full = empty + P_STAGES;
    uint32_t *tmem_slot = (uint32_t *)(acc_full + 1);

    const uint32_t crank = cluster_rank();
    const int pair_m0 = (blockIdx.x & ~1) * 128;
    const int m0 = pair_m0 + (int)crank * 128;
    const int n0 = blockIdx.y * 256;
    const int nb0 = n0 + (int)crank * 128;
    if (LOWER && n0 >= pair_m0 + 256) {
        ctx_end(ctx);
        return;
    }
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int nk = K / BK;
    const int RA = split_rows_padded(M), RB = split_rows_padded(N);

    if (threadIdx.x == 0) {
        for (int s = 0; s < P_STAGES; s++) {
            mbar_init(&full[s], 1);
            mbar_init(&pfull[s], 2);
            mbar_init(&empty[s], 1);
        }
        mbar_init(acc_full, 1);
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    if (warp == 1) {
        asm volatile("tcgen05.alloc.cta_group::2.sync.aligned.shared::cta.b32 [%0], %1;" ::"r"(smem_u32(tmem_slot)),
                     "r"(512u));
        asm volatile("tcgen05.relinquish_alloc_permit.cta_group::2.sync.aligned;");
    }
    tc_fence_before();
    cluster_sync();
    tc_fence_after();
    const uint32_t tmem = *tmem_slot;

    if (warp == 0) {
        // ------------------------------------------------------------ bulk-copy producer
        if (lane == 0) {
            for (int kb = 0; kb < nk; kb++) {
                const int s = kb % P_STAGES;
                if (kb >= P_STAGES) mbar_wait(&empty[s], ((kb / P_STAGES) - 1) & 1);
                const uint32_t st = smem_u32(smem + s * P_STAGE);
                mbar_expect_tx(&full[s], P_STAGE);
                const uint8_t *a = As + (size_t)kb * RA * 256 + (size_t)m0 * 128;
                const uint8_t *b = Bs + (size_t)kb * RB * 256 + (size_t)nb0 * 128;
                bulk_g2s(st, a, P_A_BYTES, &full[s]);
                bulk_g2s(st + P_A_BYTES, a + (size_t)RA * 128, P_A_BYTES, &full[s]);
                bulk_g2s(st + 2 * P_A_BYTES, b, P_B_BYTES, &full[s]);
                bulk_g2s(st + 2 * P_A_BYTES + P_B_BYTES, b + (size_t)RB * 128, P_B_BYTES, &full[s]);
            }
        }
        __syncwarp();
    } else if (warp == 1) {
        // ------------------------------------------------------------ relay (+ MMA issue in the leader)
        constexpr uint32_t idesc = make_idesc_f16(256, 256, NEG);
        for (int kb = 0; kb < nk; kb++) {
            const int s = kb % P_STAGES;
            const uint32_t par = (kb / P_STAGES) & 1;
            if (lane == 0) {
                mbar_wait(&full[s], par);            // this CTA's operands landed
                mbar_arrive_cluster(&pfull[s], 0);   // tell the leader
            }
            if (crank == 0) {
                mbar_wait_cluster(&pfull[s], par);   // both CTAs' operands landed
                tc_fence_after();
                if (lane == 0) {
                    const uint32_t a_big = smem_u32(smem + s * P_STAGE), a_small = a_big + P_A_BYTES;
                    const uint32_t b_big = a_big + 2 * P_A_BYTES, b_small = b_big + P_B_BYTES;
#pragma unroll
                    for (int kk = 0; kk < BK / 16; kk++) {
                        const uint32_t o = kk * 32;
                        const uint64_t dAb = make_desc(a_big + o, 16, 1024), dAs = make_desc(a_small + o, 16, 1024);
                        const uint64_t dBb = make_desc(b_big + o, 16, 1024), dBs = make_desc(b_small + o, 16, 1024);
                        const uint32_t first = (kb == 0 && kk == 0) ? 0u : 1u;
                        mma_f16_pair(tmem, dAb, dBb, idesc, first);
                        mma_f16_pair(tmem, dAb, dBs, idesc, 1u);
                        mma_f16_pair(tmem, dAs, dBb, idesc, 1u);
                    }
                    mma_commit_pair(&empty[s]);
                    if (kb == nk - 1) mma_commit_pair(acc_full);
                }
            }
            __syncwarp();
        }
    } else {
        // ------------------------------------------------------------ C_in staging + epilogue
        const int eq = warp & 3, eh = (warp - 2) >> 2;
        const int erow = m0 + eq * 32 + lane;
        const float4 z4 = make_float4(0.f, 0.f, 0.f, 0.f);
#pragma unroll 1
        for (int c = 0; c < 4; c++) {
            const int col0 = eh * 128 + c * 32;
            float v[32];
            const float *crow = C + (int64_t)erow * ldc + n0 + col0;
#pragma unroll
            for (int j = 0; j < 8; j++) {
                const float4 x = (erow < M && n0 + col0 + 4 * j < N) ? *reinterpret_cast<const float4 *>(crow + 4 * j) : z4;
                v[4 * j] = x.x; v[4 * j + 1] = x.y; v[4 * j + 2] = x.z; v[4 * j + 3] = x.w;
            }
            tmem_st32(tmem + ((uint32_t)(eq * 32) << 16) + (uint32_t)(256 + col0), v);
        }
        asm volatile("tcgen05.wait::st.sync.aligned;" ::: "memory");
        const float sa = __ldg(reinterpret_cast<const float *>(As + (size_t)RA * K * 4) + erow);
        const float *sbv = reinterpret_cast<const float *>(Bs + (size_t)RB * K * 4) + n0;

        mbar_wait(acc_full, 0);
        tc_fence_after();
#pragma unroll 1
        for (int c = 0; c < 4; c++) {
            const int col0 = eh * 128 + c * 32;
            float v[32], cv[32];
            tmem_ld32(tmem + ((uint32_t)(eq * 32) << 16) + (uint32_t)col0, v);
            tmem_ld32(tmem + ((uint32_t)(eq * 32) << 16) + (uint32_t)(256 + col0), cv);
#pragma unroll
            for (int j = 0; j < 8; j++) {
                const float4 sb = __ldg(reinterpret_cast<const float4 *>(sbv + col0) + j);
                v[4 * j + 0] = cv[4 * j + 0] + (v[4 * j + 0] * sa) * sb.x;
                v[4 * j + 1] = cv[4 * j + 1] + (v[4 * j + 1] * sa) * sb.y;
                v[4 * j + 2] = cv[4 * j + 2] + (v[4 * j + 2] * sa) * sb.z;
                v[4 * j + 3] = cv[4 * j + 3] + (v[4 * j + 3] * sa) * sb.w;
            }
            if (erow < M) {
                float *crow = C + (int64_t)erow * ldc + n0 + col0;
#pragma unroll
                for (int j = 0; j < 8; j++) {
                    const int col = n0 + col0 + 4 * j;
                    if (col >= N) break;
                    if (LOWER && col + 3 > erow) {
                        if (col + 0 <= erow) crow[4 * j + 0] = v[4 * j + 0];
                        if (col + 1 <= erow) crow[4 * j + 1] = v[4 * j + 1];
                        if (col + 2 <= erow) crow[4 * j + 2] = v[4 * j + 2];
                    } else {
                        *reinterpret_cast<float4 *>(crow + 4 * j) =
                            make_float4(v[4 * j + 0], v[4 * j + 1], v[4 * j + 2], v[4 * j + 3]);
                    }
                }
            }
        }
    }

    tc_fence_before();
    cluster_sync();
    if (warp == 1) {
        tc_fence_after();
        asm volatile("tcgen05.dealloc.cta_group::2.sync.aligned.b32 %0, %1;" ::"r"(tmem), "r"(512u));
    }
    ctx_end(ctx);
}

// ---------------------------------------------------------------- host launchers
// Split forms: X is R x K row-major (ld) -> row form; X is K x R row-major -> row form of X^T.
inline int split_rows(const float *X, int R, int K, int ld, void *out, cudaStream_t s)
{
    if (R <= 0 || K <= 0 || K % 64 || ld % 4) return -1;
    const int Rp = split_rows_padded(R);
    count_launch();
    split_rows_kernel<<<(Rp + 7) / 8, 256, 0, s>>>(X, R, K, ld, (uint8_t *)out);
    return 0;
}
inline int split_cols(const float *X, int K, int R, int ld, void *out, cudaStream_t s)
{
    if (R <= 0 || K <= 0 || K % 64) return -1;
    const int Rp = split_rows_padded(R);
    count_launch();
    split_cols_kernel<<<Rp / 32, 256, 0, s>>>(X, K, R, ld, (uint8_t *)out);
    return 0;
}

// CTA-pair launcher (VS_TCF_PAIR=0 selects the single-CTA kernel).
template <bool NEG, bool LOWER>
inline int tcf_gemm2(int M, int N, int K, const void *As, const void *Bs, float *C, int ldc, cudaStream_t s,
                     const TaskCtx &ctx)
{
    auto kern = tcf_gemm2_kernel<NEG, LOWER>;
    static bool attr[64] = {};
    int dev = 0;
    cudaGetDevice(&dev);
    if (!attr[dev & 63]) {
        cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, P_SMEM);
        attr[dev & 63] = true;
    }
    int gx = (M + 127) / 128;
    gx += gx & 1;
    dim3 grid(gx, (N + 255) / 256);
    count_launch();
    kern<<<grid, NTHREADS, P_SMEM, s>>>(M, N, K, (const uint8_t *)As, (const uint8_t *)Bs, C, ldc, ctx);
    return 0;
}

inline bool tcf_pair_enabled()
{
    static int v = [] {
        const char *e = getenv("VS_TCF_PAIR");
        return e ? atoi(e) : 1;
    }();
    return v != 0;
}

// C (M x N, ldc) += s * A * B'^T with A, B' in split form (K a multiple of 64).
template <bool NEG, bool LOWER>
inline int tcf_gemm(int M, int N, int K, const void *As, const void *Bs, float *C, int ldc, cudaStream_t s,
                    const TaskCtx &ctx = TaskCtx())
{
    if (M <= 0 || N <= 0) return 0;
    if (K % BK || ldc % 4) return -1;
    if (tcf_pair_enabled()) return tcf_gemm2<NEG, LOWER>(M, N, K, As, Bs, C, ldc, s, ctx);
    auto kern = tcf_gemm_kernel<NEG, LOWER>;
    static bool attr[64] = {};
    int dev = 0;
    cudaGetDevice(&dev);
    if (!attr[dev & 63]) {
        cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, SMEM);
        attr[dev & 63] = true;
    }
    dim3 grid((N + BN - 1) / BN, (M + BM - 1) / BM);
    count_launch();
    kern<<<grid, NTHREADS, SMEM, s>>>(M, N, K, (const uint8_t *)As, (const uint8_t *)Bs, C, ldc, ctx);
    return 0;
}

}  // namespace tcf
}  // namespace vsk

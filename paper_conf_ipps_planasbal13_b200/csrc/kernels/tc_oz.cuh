// tc_oz.cuh — fp64 tile GEMM on the tcgen05 INT8 tensor cores (Ozaki scheme), version
// oz_i8_f64, sm_100a.  The tcgen05 MMA has no f64 kind; this is the
// "tcgen05 FP64 variant" of the north star / NEXT-4.
//
//   C[M x N] (ldc, fp64) = C + s * A[M x K] * B'[N x K]^T,  s = +1 (matmul) or -1 (Cholesky
//   gemm / syrk); A and B' are given in the SLICE FORM below (B' = B^T for the matmul's NN
//   operand, = B for the NT operands of gemm / syrk).
//
// Slice form of an R x K fp64 operand X (one row = one K-major vector):
//   row r gets the power of two sc_r = 2^e_r with max_k |x_rk| / sc_r in [1/2, 1) (sc_r = 1
//   for an all-zero row); t = x / sc_r (exact), and for s = 1..S (S = 7):
//       t <- 128 t (exact),  d_s = trunc(t) in [-127, 127],  t <- t - d_s (exact)
//   so x = sc_r (sum_s d_s 2^-7s + t_S 2^-7S) with |t_S| < 1: S int8 slices carry 49 bits,
//   |x - sc_r sum_s d_s 2^-7s| < 2^-49 sc_r <= 2^-48 max_k |x_rk|.
// Product: a.b = sA sB sum_{i,j} (sum_k dA_ik dB_jk) 2^-7(i+j).  The pairs with i + j <= S+1
// are kept (28 of 49): every pair of one diagonal q = i + j shares the scale 2^-7q, so its
// integer products are accumulated by the tensor core into ONE int32 TMEM accumulator
// (exact: K * 127^2 * (q-1) < 2^31 for K <= 4096), 7 accumulators in all.  The dropped pairs
// and the slice remainders perturb each product by < (S + 3) 2^-7S |max a_row| |max b_row|
// = 10 * 2^-49 ~ 1.8e-14 of the row maxima (the fp64-class gate is relF <= 1e-12).
// Epilogue: C = C_in + s * sA_i sB_j * sum_q acc_q 2^-7q in fp64 (acc_q -> fp64 exact, the
// 2^-7q and sA sB scalings exact; the 7-term sum is the only rounding besides C_in + .).
//
// Form byte layout, row-group size G = 128 (A role) or 64 (B role of an NT / NN product)
// (Rp = R rounded up to 128, rows >= R are zero; K a multiple of 64; KB = 32):
//   [kb = k / KB][row group r / G][slice s][row r % G][KB bytes], each row in the UMMA
//   canonical K-major SWIZZLE_32B layout (8-row atoms of 256 B, 16-byte chunk index XOR
//   ((r >> 2) & 1)), then double sc[Rp] at byte S * Rp * K.  The 7 slices of one row group
//   for one k-block are one contiguous block (28 KB for G = 128, 14 KB for G = 64), so a
//   stage is filled by two bulk copies.
//
// GEMM (one 128 x 64 output tile per CTA, cta_group::1, UMMA M=128 N=64 K=32 kind::i8):
//   warp 0     lane 0: per 32-wide k-block, the bulk copies of the stage (A: one 28 KB block;
//              B: one 14 KB block, or 7 x 2 KB when B's form has G = 128, SYRK) onto the
//              stage's full barrier (expect_tx); 5 stages (210 KB) in flight.
//   warp 1     TMEM allocator (512 columns; accumulator q at columns 64(q-2)) + MMA issuer:
//              per 32-wide k-step 28 tcgen05.mma.kind::i8 (i = 1..7, j = 1..8-i),
//              tcgen05.commit -> empty[s]; after the last k-block -> acc_full.
//   warps 2-5  epilogue (TMEM lane quarter = warp % 4).
// LOWER (syrk): CTA tiles strictly above the diagonal exit; tiles crossing it store j <= i.
#pragma once
#include <cuda_runtime.h>
#include <stdint.h>

#include "kernels.hpp"
#include "task_ctx.cuh"
#include "tc_gemm.cuh"

namespace vsk {
namespace oz {

using tc::mbar_init;
using tc::mbar_wait;
using tc::smem_u32;
using tc::tc_fence_after;
using tc::tc_fence_before;
using tc::tmem_ld32;

constexpr int S = 7;                     // slices
// k-block = one KB-byte row of int8 per slice: 32 (SWIZZLE_32B rows, one MMA k-step per
// stage, 42 KB stages, 5 in flight) or 64 (SWIZZLE_64B, 84 KB stages, 2 in flight: measured
// load-latency bound)
constexpr int BM = 128, BN = 64, KB = 32;   // CTA tile
constexpr int SLA = BM * KB;             // one A slice of a stage
constexpr int SLB = BN * KB;             // one B slice
constexpr int STAGE = S * (SLA + SLB);
constexpr int STAGES = KB == 64 ? 2 : 5;
__host__ __device__ constexpr int swz(int r) { return KB == 64 ? ((r >> 1) & 3) : ((r >> 2) & 1); }
constexpr int NTHREADS = 192;
constexpr int EPI_LD = 33;               // padded row (doubles) of the epilogue staging
constexpr int SMEM = STAGES * STAGE + 1024 + 256;
static_assert(4 * 32 * EPI_LD * 8 <= STAGES * STAGE, "epilogue staging fits in the stages");

__host__ __device__ inline int rows_padded(int R) { return (R + 127) / 128 * 128; }
__host__ __device__ inline size_t form_bytes(int R, int K) { return (size_t)S * rows_padded(R) * K + (size_t)rows_padded(R) * 8; }
__host__ __device__ inline size_t slice_off(int Rp, int G, int kb, int s, int r, int chunk)
{
    return (((size_t)kb * (Rp / G) + r / G) * S + s) * G * KB + (size_t)(r % G) * KB + ((chunk ^ swz(r)) << 4);
}
// byte offset of the 7-slice block of row group r0 / G for k-block kb
__host__ __device__ inline size_t block_off(int Rp, int G, int kb, int r0)
{
    return ((size_t)kb * (Rp / G) + r0 / G) * S * G * KB;
}

// Row scales: sc_r = 2^e with max|x_r| / sc_r in [1/2, 1).  Element (r, k) of the operand is
// X[r * sr + k * sk] (row form: sr = ld, sk = 1; form of X^T: sr = 1, sk = ld).
__global__ void __launch_bounds__(256) oz_scale_kernel(const double *__restrict__ X, int R, int K, int64_t sr,
                                                       int64_t sk, uint8_t *__restrict__ out)
{
    const int Rp = rows_padded(R);
    double *sc = reinterpret_cast<double *>(out + (size_t)S * Rp * K);
    double m = 0.0;
    int r;
    if (sk == 1) {   // warp per row, lanes over k (coalesced)
        r = blockIdx.x * 8 + (threadIdx.x >> 5);
        const int lane = threadIdx.x & 31;
        if (r < R)
            for (int k = lane; k < K; k += 32) m = fmax(m, fabs(__ldg(X + (int64_t)r * sr + k)));
#pragma unroll
        for (int o = 16; o; o >>= 1) m = fmax(m, __shfl_xor_sync(0xffffffffu, m, o));
        if (lane) return;
    } else {         // thread per row (= column of X), consecutive threads on consecutive rows
        r = blockIdx.x * 256 + threadIdx.x;
        if (r < R)
            for (int k = 0; k < K; k++) m = fmax(m, fabs(__ldg(X + (int64_t)k * sk + r)));
    }
    if (r >= Rp) return;
    int e = 0;
    if (m > 0.0 && isfinite(m)) frexp(m, &e);   // m = f 2^e, f in [1/2, 1)
    sc[r] = ldexp(1.0, e);
}

// The S int8 slices of 16 consecutive k of row r per thread.
__global__ void __launch_bounds__(256) oz_slice_kernel(const double *__restrict__ X, int R, int K, int64_t sr,
                                                       int64_t sk, int G, uint8_t *__restrict__ out)
{
    const int Rp = rows_padded(R), nch = K / 16;
    const int64_t idx = (int64_t)blockIdx.x * 256 + threadIdx.x;
    if (idx >= (int64_t)Rp * nch) return;
    int r, ch;
    if (sk == 1) r = (int)(idx / nch), ch = (int)(idx % nch);   // a warp reads 4 KB of one row
    else r = (int)(idx % Rp), ch = (int)(idx / Rp);             // a warp reads 32 rows' k-th entries
    const double inv = r < R ? 1.0 / reinterpret_cast<const double *>(out + (size_t)S * Rp * K)[r] : 0.0;
    double t[16];
#pragma unroll
    for (int i = 0; i < 16; i++) {
        const int k = ch * 16 + i;
        t[i] = r < R ? __ldg(X + (int64_t)r * sr + (int64_t)k * sk) * inv : 0.0;   // inv = 2^-e: exact
    }
    const int kb = ch / (KB / 16), c = ch % (KB / 16);
#pragma unroll 1
    for (int s = 0; s < S; s++) {
        uint32_t w[4];
#pragma unroll
        for (int q = 0; q < 4; q++) {
            uint32_t v = 0;
#pragma unroll
            for (int b = 0; b < 4; b++) {
                double x = t[4 * q + b] * 128.0;
                const double d = trunc(x);
                t[4 * q + b] = x - d;
                v |= ((uint32_t)(uint8_t)(int8_t)(int)d) << (8 * b);
            }
            w[q] = v;
        }
        *reinterpret_cast<uint4 *>(out + slice_off(Rp, G, kb, s, r, c)) = make_uint4(w[0], w[1], w[2], w[3]);
    }
}

// Instruction descriptor, kind::i8: D s32 (2 at bit 4), A/B signed int8 (1 at bits 7, 10),
// K-major A and B, N>>3 at 17, M>>4 at 24.
__host__ __device__ constexpr uint32_t make_idesc_i8(int M, int N)
{
    return (2u << 4) | (1u << 7) | (1u << 10) | ((uint32_t)(N >> 3) << 17) | ((uint32_t)(M >> 4) << 24);
}

// UMMA shared-memory descriptor, K-major SWIZZLE_32B / 64B (layout type 6 / 4): KB-byte rows, 8-row
// atoms (SBO = 8 * KB bytes), LBO ignored for swizzled K-major, version 1.
__device__ __forceinline__ uint64_t desc_sw(uint32_t saddr)
{
    uint64_t d = 0;
    d |= (uint64_t)((saddr & 0x3FFFF) >> 4);
    d |= (uint64_t)(16 >> 4) << 16;
    d |= (uint64_t)((8 * KB) >> 4) << 32;            // SBO: 8-row atom
    d |= (uint64_t)1 << 46;
    d |= (uint64_t)(KB == 64 ? 4 : 6) << 61;         // SWIZZLE_64B / SWIZZLE_32B
    return d;
}

__device__ __forceinline__ void mma_i8(uint32_t tmem_d, uint64_t adesc, uint64_t bdesc, uint32_t idesc, uint32_t acc)
{
    asm volatile(
        "{\n\t.reg .pred p;\n\t"
        "setp.ne.b32 p, %4, 0;\n\t"
        "tcgen05.mma.cta_group::1.kind::i8 [%0], %1, %2, %3, p;\n\t}" ::"r"(tmem_d),
        "l"(adesc), "l"(bdesc), "r"(idesc), "r"(acc));
}

__device__ __forceinline__ void expect_tx(uint64_t *bar, uint32_t bytes)
{
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes) : "memory");
}
__device__ __forceinline__ void bulk_g2s(uint32_t dst, const void *src, uint32_t bytes, uint64_t *bar)
{
    asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(dst),
                 "l"(src), "r"(bytes), "r"(smem_u32(bar))
                 : "memory");
}

// GB: row-group size of B's form (64, or 128 when A and B are the same form: SYRK)
template <bool NEG, bool LOWER, int GB>
__global__ void __launch_bounds__(NTHREADS, 1)
    oz_gemm_kernel(int M, int N, int K, const uint8_t *__restrict__ Af, const uint8_t *__restrict__ Bf,
                   double *__restrict__ C, int ldc, int beta0, TaskCtx ctx)
{
    extern __shared__ uint8_t smem_raw[];
    uint8_t *smem = smem_raw + ((1024u - (smem_u32(smem_raw) & 1023u)) & 1023u);
    uint64_t *full = (uint64_t *)(smem + STAGES * STAGE);
    uint64_t *empty = full + STAGES;
    uint64_t *acc_full = empty + STAGES;
    uint32_t *tmem_slot = (uint32_t *)(acc_full + 1);

    ctx_begin(ctx);
    const int m0 = blockIdx.x * BM, n0 = blockIdx.y * BN;
    if (LOWER && n0 >= m0 + BM) {   // strictly above the diagonal
        ctx_end(ctx);
        return;
    }
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int nk = K / KB;
    const int RA = rows_padded(M), RB = rows_padded(N);

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
                expect_tx(&full[s], STAGE);
                bulk_g2s(st, Af + block_off(RA, 128, kb, m0), S * SLA, &full[s]);
                if (GB == 64) {
                    bulk_g2s(st + S * SLA, Bf + block_off(RB, 64, kb, n0), S * SLB, &full[s]);
                } else {   // rows n0 .. n0+63 of each slice of a 128-row group
                    const uint8_t *bb = Bf + block_off(RB, 128, kb, n0) + (size_t)(n0 % 128) * KB;
                    for (int sl = 0; sl < S; sl++)
                        bulk_g2s(st + S * SLA + sl * SLB, bb + (size_t)sl * 128 * KB, SLB, &full[s]);
                }
            }
        }
        __syncwarp();
    } else if (warp >= 2) {
        // ------------------------------------------------------------ epilogue
        mbar_wait(acc_full, 0);
        tc_fence_after();
        const int q = warp & 3;                     // TMEM lane quarter = tile rows 32q..
        double *stg = reinterpret_cast<double *>(smem) + (warp - 2) * 32 * EPI_LD;
        const double *sa = reinterpret_cast<const double *>(Af + (size_t)S * RA * K) + m0;
        const double *sb = reinterpret_cast<const double *>(Bf + (size_t)S * RB * K) + n0;
        const double sgn = NEG ? -1.0 : 1.0;
        const double sa_l = __ldg(sa + 32 * q + lane) * sgn;
#pragma unroll 1
        for (int c = 0; c < BN / 32; c++) {
            double acc[32];
#pragma unroll
            for (int i = 0; i < 32; i++) acc[i] = 0.0;
#pragma unroll 1
            for (int d = S - 1; d >= 0; d--) {   // q = d + 2: smallest terms first
                float v[32];
                tmem_ld32(tmem + ((uint32_t)(32 * q) << 16) + (uint32_t)(d * BN + c * 32), v);
                const double w = ldexp(1.0, -7 * (d + 2));
#pragma unroll
                for (int i = 0; i < 32; i++) acc[i] += (double)__float_as_int(v[i]) * w;
            }
            // this thread's row (lane) of the 32 x 32 block -> staging, then rows coalesced
#pragma unroll
            for (int i = 0; i < 32; i++) stg[lane * EPI_LD + i] = acc[i] * sa_l;
            __syncwarp();
            const int gcol = n0 + c * 32 + lane;
            const double sbl = gcol < N ? __ldg(sb + c * 32 + lane) : 0.0;
#pragma unroll 4
            for (int r = 0; r < 32; r++) {
                const int grow = m0 + 32 * q + r;
                if (grow < M && gcol < N && (!LOWER || gcol <= grow)) {
                    double *cp = C + (int64_t)grow * ldc + gcol;
                    *cp = (beta0 ? 0.0 : *cp) + stg[r * EPI_LD + lane] * sbl;
                }
            }
            __syncwarp();
        }
    } else {
        // ------------------------------------------------------------ MMA issuer (warp 1)
        const uint32_t idesc = make_idesc_i8(BM, BN);
        for (int kb = 0; kb < nk; kb++) {
            const int s = kb % STAGES;
            mbar_wait(&full[s], (kb / STAGES) & 1);
            tc_fence_after();
            if (lane == 0) {
                const uint32_t a0 = smem_u32(smem + s * STAGE), b0 = a0 + S * SLA;
                // descriptors of the stage's slices computed once: the start-address field is
                // linear (addr >> 4, no carry below 256 KB), so slice i is the base + a constant;
                // 28 MMAs of N = 64 (32 clk each) leave few issue slots per MMA
                const uint64_t dA0 = desc_sw(a0), dB0 = desc_sw(b0);
#pragma unroll
                for (int ks = 0; ks < KB / 32; ks++) {
                    uint64_t da[S], db[S];
#pragma unroll
                    for (int i = 0; i < S; i++) {
                        da[i] = dA0 + (uint64_t)((i * SLA + ks * 32) >> 4);
                        db[i] = dB0 + (uint64_t)((i * SLB + ks * 32) >> 4);
                    }
                    const uint32_t f0 = (kb == 0 && ks == 0) ? 0u : 1u;
#pragma unroll
                    for (int i = 1; i <= S; i++)
#pragma unroll
                        for (int j = 1; j <= S + 1 - i; j++)
                            mma_i8(tmem + (uint32_t)((i + j - 2) * BN), da[i - 1], db[j - 1], idesc, i == 1 ? f0 : 1u);
                }
                tc::mma_commit(&empty[s]);
                if (kb == nk - 1) tc::mma_commit(acc_full);
            }
            __syncwarp();
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

// ---------------------------------------------------------------- host launchers
// Slice form of an R x K operand: element (r, k) = X[r * sr + k * sk].
// aux: launched inside a version's task (no execution record; count_launch_aux)
inline int make_slices(const double *X, int R, int K, int64_t sr, int64_t sk, int G, void *out, cudaStream_t s,
                       bool aux = false)
{
    if (R <= 0 || K <= 0 || K % 64) return -1;
    const int Rp = rows_padded(R);
    if (aux) count_launch_aux();
    else count_launch();
    if (sk == 1) oz_scale_kernel<<<(Rp + 7) / 8, 256, 0, s>>>(X, R, K, sr, sk, (uint8_t *)out);
    else oz_scale_kernel<<<(Rp + 255) / 256, 256, 0, s>>>(X, R, K, sr, sk, (uint8_t *)out);
    if (aux) count_launch_aux();
    else count_launch();
    const int64_t n = (int64_t)Rp * (K / 16);
    oz_slice_kernel<<<(unsigned)((n + 255) / 256), 256, 0, s>>>(X, R, K, sr, sk, G, (uint8_t *)out);
    return 0;
}

// C (M x N, ldc) += s * A * B'^T with A (G = 128) and B' (G = GB) in slice form (K a
// multiple of 64).
// beta0: C = s A B^T (C_in not read; the TRSM by inverse overwrites its right-hand side)
template <bool NEG, bool LOWER, int GB>
inline int oz_gemm(int M, int N, int K, const void *Af, const void *Bf, double *C, int ldc, cudaStream_t s, bool beta0,
                   const TaskCtx &ctx = TaskCtx())
{
    if (M <= 0 || N <= 0) return 0;
    if (K % KB || N % BN || (LOWER && M != N)) return -1;
    static bool attr[64] = {};
    int dev = 0;
    cudaGetDevice(&dev);
    if (!attr[dev & 63]) {
        cudaFuncSetAttribute(oz_gemm_kernel<NEG, LOWER, GB>, cudaFuncAttributeMaxDynamicSharedMemorySize, SMEM);
        attr[dev & 63] = true;
    }
    const dim3 grid((M + BM - 1) / BM, N / BN);
    TaskCtx c = ctx_for(ctx, oz_gemm_kernel<NEG, LOWER, GB>, NTHREADS, SMEM);
    c.ncta = grid.x * grid.y;
    count_launch();
    oz_gemm_kernel<NEG, LOWER, GB><<<grid, NTHREADS, SMEM, s>>>(M, N, K, (const uint8_t *)Af, (const uint8_t *)Bf, C, ldc, beta0 ? 1 : 0, c);
    return 0;
}

}  // namespace oz
}  // namespace vsk

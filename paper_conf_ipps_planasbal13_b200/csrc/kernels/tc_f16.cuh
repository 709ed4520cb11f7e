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
// Byte layout (Rp = R rounded up to 256, rows >= R are zero; K a multiple of 32):
//   for each k-block kb of 32 columns and each group of 256 rows: [big: 256 rows x 64 B]
//   [small: 256 rows x 64 B], each part in the UMMA canonical K-major SWIZZLE_64B layout
//   (8-row atoms of 512 B, 16-byte chunk index XOR ((row >> 1) & 3)); after the Rp*K*4
//   bytes: float inv_scale[Rp] = 2^-e_r, then Rp words of scratch (column maxima of
//   split_cols).  The big+small pair of a 256-row group for one k-block is one contiguous
//   32 KB block, so the GEMM feeds shared memory with two plain bulk copies per stage
//   (cp.async.bulk, the TMA engine's 1-D mode; measured on B200: a bulk copy costs ~250
//   clk of TMA issue, so 16 KB copies cap at 66 B/clk/SM and 32 KB copies reach the
//   ~125 B/clk/SM ceiling): no tensor map, no register traffic, no per-task conversion.
//
// GEMM structure: one 256 x 256 output tile per CTA (cta_group::1), two UMMA M=128 N=256
// accumulators in TMEM (columns [0,256) = rows 0-127, [256,512) = rows 128-255).  Per
// 32-wide k-block a CTA stages 64 KB (A and B' big/small, 256 rows each) for 12 MMAs:
// ~40 B/clk of L2->SM traffic at the MMA rate, vs 64 B/clk for a 128 x 256 tile — the
// L2 (~8 TB/s measured on the 128 x 256 kernel) is what bounds this GEMM on B200.
//   warp 0      lane 0: the bulk copies of each stage (2 x 32 KB) onto the stage's full
//               barrier (expect_tx).
//   warp 1      TMEM allocator (512 columns) + MMA issuer: 2 k-steps x 2 row halves x 3
//               products per stage, tcgen05.commit -> empty[s]; last stage -> acc_full.
//   warps 2-9   epilogue (TMEM lane quarter = warp % 4, column half = (warp - 2) / 4): per
//               accumulator, tcgen05.ld 32-column chunks -> padded per-warp smem block (the
//               stage buffers are free once acc_full fired), then row by row coalesced:
//               C = C_in + acc * 2^-eA(i) * 2^-eB(j) in fp32 round-to-nearest (C_in read
//               from global here; an L2 prefetch of it at kernel start measured slower).
// LOWER (syrk): tiles strictly above the diagonal exit; diagonal tiles store only j <= i.
#pragma once
#include <cuda_fp16.h>
#include <cuda_runtime.h>
#include <stdint.h>

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

// Optional per-CTA phase timeline (measurement builds with -DVS_TCF_TRACE, tools/tcf_trace.py):
// every CTA of every launch appends {%globaltimer at: 0 start, 1 TMEM allocated, 2 first stage
// full, 3 half of the k-blocks, 4 last MMAs issued, 5 epilogue ready, 6 accumulator full,
// 8 epilogue done, 10 CTA end; 9 = total ns the MMA warp waited for full stages; 11 = SM id}
// to a device ring read back with vs_debug_tcf_trace.
#ifdef VS_TCF_TRACE
constexpr int kTcfTraceCap = 1 << 17;
__device__ unsigned long long g_tcf_rec[kTcfTraceCap][12];
__device__ unsigned int g_tcf_n;
#define TCF_DECL __shared__ unsigned long long s_tcf[12]
#define TCF_T(i) s_tcf[i] = tc_now()
#define TCF_ADD(i, v) s_tcf[i] += (v)
__device__ __forceinline__ unsigned long long tc_now()
{
    unsigned long long t;
    asm volatile("mov.u64 %0, %globaltimer;" : "=l"(t));
    return t;
}
__device__ __forceinline__ void tcf_trace_flush(unsigned long long (&s)[12])
{
    unsigned int smid;
    asm volatile("mov.u32 %0, %smid;" : "=r"(smid));
    s[10] = tc_now();
    s[11] = smid;
    const unsigned int i = atomicAdd(&g_tcf_n, 1u);
    if (i < kTcfTraceCap)
        for (int k = 0; k < 12; k++) g_tcf_rec[i][k] = s[k];
}
#else
#define TCF_DECL
#define TCF_T(i)
#define TCF_ADD(i, v)
#endif

constexpr int BT = 256, BK = 32;   // CTA tile 256 x 256; BK in fp16 elements (one 64-byte swizzled row)
constexpr int STAGES = 3;
constexpr int PART = BT * BK * 2;             // 16 KB: one part (big or small) of 256 rows
constexpr int STAGE = 4 * PART;               // A big, A small, B big, B small
constexpr int NEPI = 256;                     // epilogue threads (warps 2-9)
constexpr int NTHREADS = 64 + NEPI;
constexpr int EPI_LD = 132;                   // padded row (floats) of the epilogue staging
constexpr int SMEM = STAGES * STAGE + 1024 /*align*/ + 256 /*barriers*/;
static_assert(8 * 32 * EPI_LD * 4 <= STAGES * STAGE, "epilogue staging must fit in the stage buffers");

__host__ __device__ inline int split_rows_padded(int R) { return (R + 255) / 256 * 256; }
__host__ __device__ inline size_t split_bytes(int R, int K)
{
    const size_t Rp = (size_t)split_rows_padded(R);
    return Rp * (size_t)K * 4 + Rp * 8;
}
// byte offset of the 16-byte chunk holding elements (r, 8c .. 8c+7) of the big part; the
// small part of the same chunk is GR * 64 bytes further (big and small of one GR-row group
// are adjacent, so one 32 KB bulk copy moves both; GR = 256, the CTA tile of tcf_gemm_kernel)
constexpr int SPLIT_HALF = 256 * 64;
template <int GR = 256>
__host__ __device__ inline size_t split_chunk_off(int Rp, int r, int c)
{
    const int kb = c >> 2, kc = c & 3;
    return (size_t)kb * Rp * 128 + (size_t)(r / GR) * (2 * GR * 64) + (size_t)(r % GR) * 64 + ((kc ^ ((r >> 1) & 3)) << 4);
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
template <int GR>
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
    const size_t half = (size_t)GR * 64;
    for (int k = 8 * lane; k < K; k += 256) {
        float v[8] = {0.f, 0.f, 0.f, 0.f, 0.f, 0.f, 0.f, 0.f};
        if (r < R) {
            const float4 a = __ldg(reinterpret_cast<const float4 *>(row + k));
            const float4 b = __ldg(reinterpret_cast<const float4 *>(row + k + 4));
            v[0] = a.x; v[1] = a.y; v[2] = a.z; v[3] = a.w; v[4] = b.x; v[5] = b.y; v[6] = b.z; v[7] = b.w;
        }
        uint4 big, small;
        split8(v, sc, big, small);
        const size_t off = split_chunk_off<GR>(Rp, r, k >> 3);
        *reinterpret_cast<uint4 *>(out + off) = big;
        *reinterpret_cast<uint4 *>(out + off + half) = small;
    }
    if (lane == 0) reinterpret_cast<float *>(out + (size_t)Rp * K * 4)[r] = ldexpf(1.f, -e);
}

// Row form of X^T for a K x R row-major fp32 matrix X (ld): form row r = column r of X.
// Pass 1 (split_colmax_kernel, grid (Rp/32, K/128)): column maxima of |x| folded into the
// form's scratch words with atomicMax on the float bits (non-negative floats order as
// integers; the scratch is zeroed first).  Pass 2 (split_cols_kernel, grid (Rp/32, K/64)):
// 64 x 32 blocks transposed through shared memory, 16-byte stores of 8 consecutive k.
__global__ void __launch_bounds__(256) split_colmax_kernel(const float *__restrict__ X, int K, int R, int ld,
                                                           uint8_t *__restrict__ out)
{
    __shared__ float cmax[8][32];
    const int Rp = split_rows_padded(R);
    const int w = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int col = blockIdx.x * 32 + lane, k0 = blockIdx.y * 128;
    float m = 0.f;
    if (col < R)
#pragma unroll 4
        for (int k = k0 + w; k < min(K, k0 + 128); k += 8) m = fmaxf(m, fabsf(__ldg(X + (int64_t)k * ld + col)));
    cmax[w][lane] = m;
    __syncthreads();
    if (w == 0) {
        float mm = cmax[0][lane];
#pragma unroll
        for (int i = 1; i < 8; i++) mm = fmaxf(mm, cmax[i][lane]);
        if (col < Rp) atomicMax(reinterpret_cast<int *>(out + (size_t)Rp * K * 4 + (size_t)Rp * 4) + col, __float_as_int(mm));
    }
}

template <int GR>
__global__ void __launch_bounds__(256) split_cols_kernel(const float *__restrict__ X, int K, int R, int ld,
                                                         uint8_t *__restrict__ out)
{
    __shared__ float tile[64][33];
    const int Rp = split_rows_padded(R);
    const int r0 = blockIdx.x * 32, k0 = blockIdx.y * 64, w = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int col = r0 + lane;
#pragma unroll
    for (int i = 0; i < 8; i++) {
        const int k = k0 + w * 8 + i;
        tile[w * 8 + i][lane] = (col < R && k < K) ? __ldg(X + (int64_t)k * ld + col) : 0.f;
    }
    const int rr = threadIdx.x >> 3, kc = threadIdx.x & 7;   // form row r0+rr, chunk kc of the block
    const float m = __int_as_float(reinterpret_cast<const int *>(out + (size_t)Rp * K * 4 + (size_t)Rp * 4)[r0 + rr]);
    const int e = row_exponent(m);
    if (blockIdx.y == 0 && kc == 0) reinterpret_cast<float *>(out + (size_t)Rp * K * 4)[r0 + rr] = ldexpf(1.f, -e);
    __syncthreads();
    if (k0 + kc * 8 < K) {
        float v[8];
#pragma unroll
        for (int i = 0; i < 8; i++) v[i] = tile[kc * 8 + i][rr];
        uint4 big, small;
        split8(v, ldexpf(1.f, e), big, small);
        const size_t off = split_chunk_off<GR>(Rp, r0 + rr, (k0 >> 3) + kc);
        *reinterpret_cast<uint4 *>(out + off) = big;
        *reinterpret_cast<uint4 *>(out + off + (size_t)GR * 64) = small;
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
// the same bytes into the same smem offset of every CTA in ctaMask (cluster), each CTA's
// mbarrier at the same offset receiving the complete_tx
__device__ __forceinline__ void bulk_g2s_mc(uint32_t dst, const void *src, uint32_t bytes, uint64_t *bar, uint16_t mask)
{
    asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes.multicast::cluster [%0], [%1], %2, [%3], %4;"
                 ::"r"(dst), "l"(src), "r"(bytes), "r"(smem_u32(bar)), "h"(mask)
                 : "memory");
}
__device__ __forceinline__ void mma_commit_mc(uint64_t *bar, uint16_t mask)
{
    asm volatile("tcgen05.commit.cta_group::1.mbarrier::arrive::one.shared::cluster.multicast::cluster.b64 [%0], %1;"
                 ::"r"(smem_u32(bar)), "h"(mask)
                 : "memory");
}
__device__ __forceinline__ void cluster_sync_all()
{
    asm volatile("barrier.cluster.arrive.release.aligned;\n\tbarrier.cluster.wait.acquire.aligned;" ::: "memory");
}
__device__ __forceinline__ uint32_t cluster_ctarank()
{
    uint32_t r;
    asm volatile("mov.u32 %0, %%cluster_ctarank;" : "=r"(r));
    return r;
}


// UMMA shared-memory descriptor, K-major SWIZZLE_64B (layout type 4): rows of 64 B, 8-row
// atoms of 512 B (SBO), LBO = 16 B (ignored for swizzled K-major), version 1.
__device__ __forceinline__ uint64_t make_desc_sw64(uint32_t saddr)
{
    uint64_t d = 0;
    d |= (uint64_t)((saddr & 0x3FFFF) >> 4);
    d |= (uint64_t)(16 >> 4) << 16;
    d |= (uint64_t)(512 >> 4) << 32;
    d |= (uint64_t)1 << 46;
    d |= (uint64_t)4 << 61;
    return d;
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

// One GEMM task of a grouped launch: C (M x N, ldc) += s * A * B'^T on split forms.
// flags: bit 0 = negate (s = -1), bit 1 = LOWER (only tiles with j <= i exist, and the
// diagonal tiles store j <= i), bit 2 = BETA0 (C = s A B'^T: C_in is not read).  The task's CTAs are [tile0, tile0 + ntiles) of the grid.
struct TcfTask {
    const uint8_t *As, *Bs;          // split forms, advanced to the task's first k-block
    const float *sa, *sb;            // their row scales 2^-e (at the end of the full forms)
    float *C;
    int M, N, K, ldc;
    int flags, tile0, ntiles, tiles_n;
    TaskCtx ctx;
};
constexpr int kMaxGroup = 24;
// host-side accumulator of a grouped launch; the kernel receives a copy sized to the group
// (TcfGroupN<G>, G = 1, 4 or kMaxGroup): kernel parameters are copied by the launch, and a
// 2 KB parameter block costs host launch time on every single-task launch
template <int G>
struct TcfGroupN {
    int n = 0, ctas = 0;
    TcfTask t[G];
};
using TcfGroup = TcfGroupN<kMaxGroup>;
static_assert(sizeof(TcfGroup) <= 4000, "kernel parameter space");

// PAIR: clusters of two CTAs computing tiles (bi, 2p) and (bi, 2p+1) of one task share the
// A operand: each CTA bulk-copies one half (big or small part) of the stage's A block and
// multicasts it into both CTAs, so a CTA reads 48 KB per k-block from L2 instead of 64 KB
// (the GEMM is L2-bandwidth bound when every SM runs it).  A stage of either CTA is
// refilled only after BOTH CTAs' MMAs released it (empty barriers count 2: each MMA warp
// commits to its own and its peer's).  A pair whose second tile does not exist (odd tile
// count in a row, or above the diagonal for LOWER) runs a "ghost" CTA: it loads and
// multiplies a valid tile but stores nothing.
template <int G, bool PAIR>
__global__ void __launch_bounds__(NTHREADS, 1) tcf_gemm_kernel(const __grid_constant__ TcfGroupN<G> grp)
{
    extern __shared__ uint8_t smem_raw[];
    uint8_t *smem = smem_raw + ((1024u - (smem_u32(smem_raw) & 1023u)) & 1023u);
    TCF_DECL;
    uint64_t *full = (uint64_t *)(smem + STAGES * STAGE);
    uint64_t *empty = full + STAGES;
    uint64_t *acc_full = empty + STAGES;
    uint32_t *tmem_slot = (uint32_t *)(acc_full + 1);

    // this CTA's task and output tile
    int ti = 0;
    while (ti + 1 < grp.n && (int)blockIdx.x >= grp.t[ti + 1].tile0) ti++;
    const TcfTask &tk = grp.t[ti];
    const TaskCtx ctx = tk.ctx;
    ctx_begin(ctx);
    const int M = tk.M, N = tk.N, K = tk.K, ldc = tk.ldc;
    const uint8_t *__restrict__ As = tk.As;
    const uint8_t *__restrict__ Bs = tk.Bs;
    float *__restrict__ C = tk.C;
    const bool NEG = tk.flags & 1, LOWER = (tk.flags >> 1) & 1;
    const int l = (int)blockIdx.x - tk.tile0;
    int bi, bj;
    bool ghost = false;
    const uint32_t rank = PAIR ? cluster_ctarank() : 0u;
    if (PAIR) {
        const int pi = l >> 1;
        int p;
        if (LOWER) {   // row bi holds bi/2 + 1 pairs
            bi = 0;
            int acc = 0;
            while (acc + bi / 2 + 1 <= pi) acc += bi / 2 + 1, bi++;
            p = pi - acc;
        } else {
            const int ppr = (tk.tiles_n + 1) / 2;
            bi = pi / ppr;
            p = pi % ppr;
        }
        bj = 2 * p + (int)rank;
        ghost = bj >= tk.tiles_n || (LOWER && bj > bi);
        if (ghost) bj = 2 * p;   // a valid tile to load; nothing is stored
    } else if (LOWER) {   // l = bi (bi + 1) / 2 + bj, bj <= bi
        bi = (int)((sqrtf(8.f * l + 1.f) - 1.f) * 0.5f);
        while ((bi + 1) * (bi + 2) / 2 <= l) bi++;
        while (bi * (bi + 1) / 2 > l) bi--;
        bj = l - bi * (bi + 1) / 2;
    } else {
        bi = l / tk.tiles_n;
        bj = l % tk.tiles_n;
    }
    const int m0 = bi * BT, n0 = bj * BT;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int nk = K / BK;
    const int RA = split_rows_padded(M), RB = split_rows_padded(N);

    if (threadIdx.x == 0) {
        TCF_T(0);
#ifdef VS_TCF_TRACE
        s_tcf[9] = 0;
#endif
        for (int s = 0; s < STAGES; s++) {
            mbar_init(&full[s], 1);
            mbar_init(&empty[s], PAIR ? 2 : 1);
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
    if (PAIR) cluster_sync_all();   // the peer's barriers are initialised before any multicast
    const uint32_t tmem = *tmem_slot;
    if (threadIdx.x == 0) TCF_T(1);

    if (warp == 0) {
        // ------------------------------------------------------------ bulk-copy producer
        if (lane == 0) {
            for (int kb = 0; kb < nk; kb++) {
                const int s = kb % STAGES;
                if (kb >= STAGES) mbar_wait(&empty[s], ((kb / STAGES) - 1) & 1);
                const uint32_t st = smem_u32(smem + s * STAGE);
                mbar_expect_tx(&full[s], STAGE);
                if (PAIR)   // this CTA's half (big or small part) of the A block, into both CTAs
                    bulk_g2s_mc(st + rank * PART, As + (size_t)kb * RA * 128 + (size_t)m0 * 128 + rank * PART, PART,
                                &full[s], (uint16_t)3);
                else
                    bulk_g2s(st, As + (size_t)kb * RA * 128 + (size_t)m0 * 128, 2 * PART, &full[s]);
                bulk_g2s(st + 2 * PART, Bs + (size_t)kb * RB * 128 + (size_t)n0 * 128, 2 * PART, &full[s]);
            }
        }
        __syncwarp();
    } else if (warp == 1) {
        // ------------------------------------------------------------ MMA issuer
        const uint32_t idesc = make_idesc_f16(128, BT, NEG);
        for (int kb = 0; kb < nk; kb++) {
            const int s = kb % STAGES;
#ifdef VS_TCF_TRACE
            const unsigned long long w0 = tc_now();
#endif
            mbar_wait(&full[s], (kb / STAGES) & 1);
#ifdef VS_TCF_TRACE
            if (lane == 0) {
                TCF_ADD(9, tc_now() - w0);
                if (kb == 0) TCF_T(2);
                if (kb == nk / 2) TCF_T(3);
            }
#endif
            tc_fence_after();
            if (lane == 0) {
                const uint32_t a_big = smem_u32(smem + s * STAGE), a_small = a_big + PART;
                const uint32_t b_big = a_big + 2 * PART, b_small = a_big + 3 * PART;
#pragma unroll
                for (int kk = 0; kk < BK / 16; kk++) {
                    const uint32_t o = kk * 32;   // 16 fp16 = 32 B inside the 64 B swizzled row
                    const uint64_t dBb = make_desc_sw64(b_big + o), dBs = make_desc_sw64(b_small + o);
#pragma unroll
                    for (int h = 0; h < 2; h++) {   // rows [128h, 128h+128) -> TMEM columns [256h, 256h+256)
                        const uint32_t ho = h * 128 * 64;
                        const uint64_t dAb = make_desc_sw64(a_big + ho + o), dAs = make_desc_sw64(a_small + ho + o);
                        const uint32_t first = (kb == 0 && kk == 0) ? 0u : 1u;
                        const uint32_t d = tmem + (uint32_t)(h * BT);
                        mma_f16(d, dAb, dBb, idesc, first);
                        mma_f16(d, dAb, dBs, idesc, 1u);
                        mma_f16(d, dAs, dBb, idesc, 1u);
                    }
                }
                if (PAIR && kb < nk - STAGES)
                    mma_commit_mc(&empty[s], (uint16_t)3);   // both CTAs' producers refill stage s
                else if (!PAIR)
                    tc::mma_commit(&empty[s]);
                if (kb == nk - 1) {
                    tc::mma_commit(acc_full);
                    TCF_T(4);
                }
            }
            __syncwarp();
        }
    } else {
        // ------------------------------------------------------------ epilogue
        const int q = warp & 3, eh = (warp - 2) >> 2;   // TMEM lane quarter, column half
        float *stg = reinterpret_cast<float *>(smem) + (warp - 2) * 32 * EPI_LD;   // this warp's 32 x 128 block
        const int ccol = eh * 128 + lane * 4;            // this lane's 4 columns in the store phase
        const float *sav = tk.sa + m0;
        const float4 sb = __ldg(reinterpret_cast<const float4 *>(tk.sb + n0 + ccol));
        const bool BETA0 = (tk.flags >> 2) & 1;   // C = s A B'^T (C_in not read)
        // (no L2 prefetch of C_in during the main loop: measured in the bench with and without,
        // interleaved, 303-307 vs 308-310 TFLOP/s — the 256 KB per CTA issued at kernel start
        // competes with the operand streams for L2 and is partly evicted before the epilogue)
        if (warp == 2 && lane == 0) TCF_T(5);
        mbar_wait(acc_full, 0);
        tc_fence_after();
        if (warp == 2 && lane == 0) TCF_T(6);
        const int gcol = n0 + ccol;
#pragma unroll 1
        for (int h = 0; h < (ghost ? 0 : 2); h++) {
            const int rbase = h * 128 + q * 32;          // tile rows of this warp
            const float sa_l = __ldg(sav + rbase + lane);
#pragma unroll 1
            for (int c = 0; c < 4; c++) {
                float v[32];
                tmem_ld32(tmem + ((uint32_t)(q * 32) << 16) + (uint32_t)(h * BT + eh * 128 + c * 32), v);
#pragma unroll
                for (int j = 0; j < 8; j++)
                    *reinterpret_cast<float4 *>(stg + lane * EPI_LD + c * 32 + 4 * j) =
                        make_float4(v[4 * j], v[4 * j + 1], v[4 * j + 2], v[4 * j + 3]);
            }
            __syncwarp();
            // 16 rows per round: all C_in loads of the round in flight before the first use
#pragma unroll 1
            for (int r0 = 0; r0 < 32; r0 += 16) {
                float4 cin[16];
#pragma unroll
                for (int i = 0; i < 16; i++) {
                    const int grow = m0 + rbase + r0 + i;
                    cin[i] = (!BETA0 && grow < M && gcol < N) ? *reinterpret_cast<const float4 *>(C + (int64_t)grow * ldc + gcol)
                                                              : make_float4(0.f, 0.f, 0.f, 0.f);
                }
#pragma unroll
                for (int i = 0; i < 16; i++) {
                    const int r = r0 + i, grow = m0 + rbase + r;
                    const float sa = __shfl_sync(0xffffffffu, sa_l, r);
                    if (grow < M && gcol < N) {
                        float *cp = C + (int64_t)grow * ldc + gcol;
                        const float4 a = *reinterpret_cast<const float4 *>(stg + r * EPI_LD + lane * 4);
                        float4 o;
                        o.x = cin[i].x + (a.x * sa) * sb.x;
                        o.y = cin[i].y + (a.y * sa) * sb.y;
                        o.z = cin[i].z + (a.z * sa) * sb.z;
                        o.w = cin[i].w + (a.w * sa) * sb.w;
                        if (LOWER && gcol + 3 > grow) {
                            if (gcol + 0 <= grow) cp[0] = o.x;
                            if (gcol + 1 <= grow) cp[1] = o.y;
                            if (gcol + 2 <= grow) cp[2] = o.z;
                        } else {
                            *reinterpret_cast<float4 *>(cp) = o;
                        }
                    }
                }
            }
            __syncwarp();
        }
        if (warp == 2 && lane == 0) TCF_T(8);
    }

    tc_fence_before();
    __syncthreads();
    if (warp == 1) {
        tc_fence_after();
        asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, %1;" ::"r"(tmem), "r"(512u));
    }
    if (PAIR) cluster_sync_all();   // no CTA leaves while its peer may still address its smem
#ifdef VS_TCF_TRACE
    if (threadIdx.x == 0) tcf_trace_flush(s_tcf);
#endif
    ctx_end(ctx);
}

// ---------------------------------------------------------------- host launchers
// Split forms: X is R x K row-major (ld) -> row form; X is K x R row-major -> row form of X^T.
// gr: row group of the layout (256 = the CTA tile of tcf_gemm_kernel; 128 also supported)
inline int split_rows(const float *X, int R, int K, int ld, void *out, cudaStream_t s, int gr = 256)
{
    if (R <= 0 || K <= 0 || K % 32 || ld % 4 || (gr != 256 && gr != 128)) return -1;
    const int Rp = split_rows_padded(R);
    count_launch();
    if (gr == 256) split_rows_kernel<256><<<(Rp + 7) / 8, 256, 0, s>>>(X, R, K, ld, (uint8_t *)out);
    else split_rows_kernel<128><<<(Rp + 7) / 8, 256, 0, s>>>(X, R, K, ld, (uint8_t *)out);
    return 0;
}
inline int split_cols(const float *X, int K, int R, int ld, void *out, cudaStream_t s, int gr = 256)
{
    if (gr != 256 && gr != 128) return -1;
    if (R <= 0 || K <= 0 || K % 32) return -1;
    const int Rp = split_rows_padded(R);
    if (cudaMemsetAsync((uint8_t *)out + (size_t)Rp * K * 4 + (size_t)Rp * 4, 0, (size_t)Rp * 4, s) != cudaSuccess)
        return -1;
    count_launch();
    split_colmax_kernel<<<dim3(Rp / 32, (K + 127) / 128), 256, 0, s>>>(X, K, R, ld, (uint8_t *)out);
    count_launch();
    if (gr == 256) split_cols_kernel<256><<<dim3(Rp / 32, (K + 63) / 64), 256, 0, s>>>(X, K, R, ld, (uint8_t *)out);
    else split_cols_kernel<128><<<dim3(Rp / 32, (K + 63) / 64), 256, 0, s>>>(X, K, R, ld, (uint8_t *)out);
    return 0;
}

// Append one task to a group; returns its CTA count, 0 for an empty task, -1 if it does
// not fit or is unsupported (K a multiple of 32, ldc of 4).
// CTA-pair (A multicast) variant of the GEMM: on unless VS_TCF_PAIR=0
inline bool tcf_pair()
{
    // CTA pairs with A multicast (VS_TCF_PAIR=1): measured equal to single CTAs in session 3 and
    // 1.2 % slower (308.4-309.0 vs 311.2-312.9 TFLOP/s interleaved) once the C_in L2 prefetch was
    // gone: single CTAs by default
    static const int v = [] {
        const char *e = getenv("VS_TCF_PAIR");
        return e ? atoi(e) : 0;
    }();
    return v != 0;
}

// K-chunk [k0, k0 + kc) of a GEMM whose split forms have K columns (k0, kc multiples of 32;
// kc = K: the whole product)
inline int tcf_group_add(TcfGroup &g, int M, int N, int K, const void *As, const void *Bs, float *C, int ldc,
                         bool neg, bool lower, TaskCtx ctx, bool beta0 = false, int k0 = 0, int kc = -1)
{
    if (M <= 0 || N <= 0) return 0;
    if (kc < 0) kc = K;
    if (K % BK || k0 % BK || kc % BK || k0 + kc > K || ldc % 4 || g.n >= kMaxGroup || (lower && M != N)) return -1;
    const int tm = (M + BT - 1) / BT, tn = (N + BT - 1) / BT;
    int nt = lower ? tm * (tm + 1) / 2 : tm * tn;
    if (tcf_pair()) {   // two CTAs per pair of tiles in a row (kernel comment): rows hold ceil(tn/2)
        nt = 0;         // pairs, row bi of a LOWER task bi/2 + 1
        for (int bi = 0; bi < tm; bi++) nt += 2 * (lower ? bi / 2 + 1 : (tn + 1) / 2);
    }
    const int RA = split_rows_padded(M), RB = split_rows_padded(N);
    TcfTask &t = g.t[g.n++];
    t.As = (const uint8_t *)As + (size_t)(k0 / BK) * RA * 128;
    t.Bs = (const uint8_t *)Bs + (size_t)(k0 / BK) * RB * 128;
    t.sa = reinterpret_cast<const float *>((const uint8_t *)As + (size_t)RA * K * 4);
    t.sb = reinterpret_cast<const float *>((const uint8_t *)Bs + (size_t)RB * K * 4);
    t.C = C;
    t.M = M; t.N = N; t.K = kc; t.ldc = ldc;
    t.flags = (neg ? 1 : 0) | (lower ? 2 : 0) | (beta0 ? 4 : 0);
    t.tile0 = g.ctas;
    t.ntiles = nt;
    t.tiles_n = tn;
    ctx.ncta = (unsigned)nt;
    t.ctx = ctx;
    g.ctas += nt;
    return nt;
}

template <int G, bool PAIR>
inline void tcf_launch_one(const TcfGroupN<G> &h, int ctas, cudaStream_t s)
{
    if (!PAIR) {
        tcf_gemm_kernel<G, false><<<ctas, NTHREADS, SMEM, s>>>(h);
        return;
    }
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = dim3(ctas);
    cfg.blockDim = dim3(NTHREADS);
    cfg.dynamicSmemBytes = SMEM;
    cfg.stream = s;
    cudaLaunchAttribute at[1];
    at[0].id = cudaLaunchAttributeClusterDimension;
    at[0].val.clusterDim.x = 2;
    at[0].val.clusterDim.y = 1;
    at[0].val.clusterDim.z = 1;
    cfg.attrs = at;
    cfg.numAttrs = 1;
    cudaLaunchKernelEx(&cfg, tcf_gemm_kernel<G, true>, h);
}

template <bool PAIR>
inline void tcf_launch(TcfGroup &g, cudaStream_t s)
{
    if (g.n == 1) {
        TcfGroupN<1> h;
        h.n = 1; h.ctas = g.ctas; h.t[0] = g.t[0];
        tcf_launch_one<1, PAIR>(h, g.ctas, s);
    } else if (g.n <= 4) {
        TcfGroupN<4> h;
        h.n = g.n; h.ctas = g.ctas;
        for (int i = 0; i < g.n; i++) h.t[i] = g.t[i];
        tcf_launch_one<4, PAIR>(h, g.ctas, s);
    } else {
        tcf_launch_one<kMaxGroup, PAIR>(g, g.ctas, s);
    }
}

inline int tcf_group_launch(TcfGroup &g, cudaStream_t s)
{
    if (g.n == 0) return 0;
    static bool attr[64] = {};
    int dev = 0;
    cudaGetDevice(&dev);
    if (!attr[dev & 63]) {
        cudaFuncSetAttribute(tcf_gemm_kernel<1, false>, cudaFuncAttributeMaxDynamicSharedMemorySize, SMEM);
        cudaFuncSetAttribute(tcf_gemm_kernel<4, false>, cudaFuncAttributeMaxDynamicSharedMemorySize, SMEM);
        cudaFuncSetAttribute(tcf_gemm_kernel<kMaxGroup, false>, cudaFuncAttributeMaxDynamicSharedMemorySize, SMEM);
        cudaFuncSetAttribute(tcf_gemm_kernel<1, true>, cudaFuncAttributeMaxDynamicSharedMemorySize, SMEM);
        cudaFuncSetAttribute(tcf_gemm_kernel<4, true>, cudaFuncAttributeMaxDynamicSharedMemorySize, SMEM);
        cudaFuncSetAttribute(tcf_gemm_kernel<kMaxGroup, true>, cudaFuncAttributeMaxDynamicSharedMemorySize, SMEM);
        attr[dev & 63] = true;
    }
    count_launch();
    if (tcf_pair()) tcf_launch<true>(g, s);
    else tcf_launch<false>(g, s);
    g.n = g.ctas = 0;
    return 0;
}

__global__ void eye_kernel(float *X, int n)
{
    // n % 4 == 0: float4 stores, rows strided over the grid
    const int nq = n / 4;
    for (int r = blockIdx.x; r < n; r += gridDim.x)
        for (int q = threadIdx.x; q < nq; q += blockDim.x) {
            const bool d = (r >> 2) == q;
            const float4 v = make_float4(d && (r & 3) == 0, d && (r & 3) == 1, d && (r & 3) == 2, d && (r & 3) == 3);
            reinterpret_cast<float4 *>(X + (int64_t)r * n)[q] = v;
        }
}

// C (M x N, ldc) += s * A * B'^T with A, B' in split form (K a multiple of 32): one task.
template <bool NEG, bool LOWER>
inline int tcf_gemm(int M, int N, int K, const void *As, const void *Bs, float *C, int ldc, cudaStream_t s,
                    const TaskCtx &ctx = TaskCtx())
{
    for (int k0 = 0; k0 < K; k0 += tc::kKChunk) {   // accumulation accuracy: see tc::tc_gemm
        TcfGroup g;
        const int r = tcf_group_add(g, M, N, K, As, Bs, C, ldc, NEG, LOWER, ctx, false, k0,
                                    K - k0 < tc::kKChunk ? K - k0 : tc::kKChunk);
        if (r <= 0) return r;
        if (tcf_group_launch(g, s)) return -1;
    }
    return 0;
}

}  // namespace tcf
}  // namespace vsk

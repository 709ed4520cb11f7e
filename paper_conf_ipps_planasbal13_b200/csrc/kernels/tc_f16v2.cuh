// tc_f16v2.cuh — persistent CTA-pair tcgen05 3xFP16 GEMM for the tc_3xf16 version (sm_100a).
//
// Same arithmetic as tcf_gemm_kernel (tc_f16.cuh, reading R30): C = C_in + s * A * B'^T on
// row-scaled fp16 big/small split forms, three kind::f16 products per 16-wide k-step, the
// epilogue multiplying by 2^-eA(i) 2^-eB(j) and adding C_in in fp32 round-to-nearest.  What
// differs is how the work maps to the SMs:
//
//   * a CLUSTER OF TWO CTAs (one TPC) computes one 256 x 256 output tile with
//     tcgen05.mma.cta_group::2 (M = 256, N = 256): CTA q holds rows [128q, 128q + 128) of
//     the tile's A block and rows [128q, 128q + 128) of its B' block (the N half), the MMA
//     issued by CTA 0 reads both CTAs' shared memory, and each CTA's TMEM receives its 128
//     rows x 256 columns of the accumulator.  Per SM this is the operand traffic of the
//     one-CTA 256 x 256 tile (16 KB of A + 16 KB of B' per 32-wide k-block for 6 MMAs of
//     128 cycles), but the accumulator takes only 256 of the 512 TMEM columns, so
//   * TMEM is DOUBLE-BUFFERED and the kernel is PERSISTENT: each cluster loops over several
//     tiles of the grouped launch (static round robin), the MMA warp accumulates tile j+1
//     into the other buffer while the epilogue warps drain tile j, so the epilogue (TMEM ->
//     registers -> shared staging -> coalesced C_in + acc rows) is hidden behind the next
//     tile's MMAs instead of idling the tensor core (the PACING LAW of the microbenchmarks:
//     tile time = max(MMA, epilogue) once they overlap).
//
// Split-form layout: 128-row groups (split_rows / split_cols with gr = 128): for k-block kb,
// group g = the big part (128 rows x 64 B, SWIZZLE_64B K-major) followed by the small part, so
// one CTA's half of a stage is one 16 KB bulk copy per operand.
//
// Roles (320 threads per CTA):
//   warp 0 lane 0   producer: bulk copies of this CTA's A half and B' half per k-block onto
//                   its full[s] barrier (expect_tx 32 KB), after empty[s].
//   warp 1 lane 0   CTA 0: MMA issuer — waits full[s] and pfull[s] (the peer's stage landed),
//                   6 tcgen05.mma.cta_group::2 per k-block, commits empty[s] to both CTAs,
//                   accf[b] to both CTAs after a tile; waits acce[b] before reusing buffer b.
//                   CTA 1: relay — waits its own full[s] and arrives on CTA 0's pfull[s].
//                   Warp 1 of both CTAs also allocates the 512 TMEM columns (cta_group::2).
//   warps 2-9       epilogue (TMEM lane quarter = warp % 4, column half = (warp - 2) / 4):
//                   per tile, 4 x 32 columns per warp: tcgen05.ld 32 columns of the lane's row,
//                   C_in read, C = C_in + acc * 2^-eA * 2^-eB, stored straight from registers
//                   (each lane 128 contiguous bytes of its row: no shared staging, which leaves
//                   192 KB for 6 operand stages; the epilogue is hidden behind the next tile's
//                   MMAs, so its less coalesced accesses cost no tensor time); after the tile's
//                   last TMEM read one thread per CTA arrives on CTA 0's acce[b]; after the
//                   stores the tile is reported to its task's execution record (ctx_done).
// LOWER (syrk): only tiles with bj <= bi exist; diagonal tiles store only j <= i.
#pragma once
#include "tc_f16.cuh"

namespace vsk {
namespace tcf2 {

using tc::mbar_init;
using tc::mbar_wait;
using tc::smem_u32;
using tc::tc_fence_after;
using tc::tc_fence_before;
using tc::tmem_ld32;
using tcf::bulk_g2s;
using tcf::cluster_ctarank;
using tcf::cluster_sync_all;
using tcf::make_desc_sw64;
using tcf::make_idesc_f16;
using tcf::mbar_expect_tx;
using tcf::split_rows_padded;
using tcf::TcfGroup;
using tcf::TcfGroupN;
using tcf::TcfTask;

constexpr int GR = 128;                 // split-form row group = one CTA's half of a tile
constexpr int BT = 256, BK = 32;        // pair tile 256 x 256; k-block of 32 fp16 (64 B rows)
constexpr int STAGES = 6;               // 192 KB: a refill (empty -> copy -> full -> relay) takes
                                        // longer than 3 stages of MMAs (768 cycles each)
constexpr int OPER = 2 * GR * BK * 2;   // 16 KB: big + small of 128 rows (one bulk copy)
constexpr int STAGE = 2 * OPER;         // A half + B' half
constexpr int NEPI = 256;
constexpr int NTHREADS = 64 + NEPI;
constexpr int STG = 0;                  // the epilogue stores straight from registers
constexpr int NBAR = 3 * STAGES + 4;                         // full, empty, pfull, accf[2], acce[2]
constexpr int SMEM = STAGES * STAGE + STG + 1024 + 8 * NBAR + 64;   // + tmem slot, ustart[4]
static_assert(SMEM <= 232448, "shared memory");

// process-wide switch (env VS_TCF_V2=1): which tc_3xf16 GEMM kernel (and split-form layout)
// the runtime uses; default: tcf_gemm_kernel (tc_f16.cuh)
inline bool enabled()
{
    static const int v = [] {
        const char *e = getenv("VS_TCF_V2");
        return e ? atoi(e) : 0;
    }();
    return v != 0;
}
inline int form_group_rows() { return enabled() ? GR : 256; }

__device__ __forceinline__ uint32_t mapa(uint32_t saddr, uint32_t rank)
{
    uint32_t r;
    asm volatile("mapa.shared::cluster.u32 %0, %1, %2;" : "=r"(r) : "r"(saddr), "r"(rank));
    return r;
}
__device__ __forceinline__ void arrive_cluster(uint32_t cluster_addr)
{
    asm volatile("mbarrier.arrive.release.cluster.shared::cluster.b64 _, [%0];" ::"r"(cluster_addr) : "memory");
}
__device__ __forceinline__ void mma2_f16(uint32_t tmem_d, uint64_t adesc, uint64_t bdesc, uint32_t idesc, uint32_t acc)
{
    asm volatile(
        "{\n\t.reg .pred p;\n\t"
        "setp.ne.b32 p, %4, 0;\n\t"
        "tcgen05.mma.cta_group::2.kind::f16 [%0], %1, %2, %3, p;\n\t}" ::"r"(tmem_d),
        "l"(adesc), "l"(bdesc), "r"(idesc), "r"(acc));
}
__device__ __forceinline__ void commit2_mc(uint64_t *bar, uint16_t mask)
{
    asm volatile("tcgen05.commit.cta_group::2.mbarrier::arrive::one.shared::cluster.multicast::cluster.b64 [%0], %1;"
                 ::"r"(smem_u32(bar)), "h"(mask)
                 : "memory");
}
__device__ __forceinline__ void named_bar(int id, int n)
{
    asm volatile("bar.sync %0, %1;" ::"r"(id), "r"(n) : "memory");
}

// unit u of the group -> task index and tile (bi, bj)
template <int G>
__device__ __forceinline__ void unit_tile(const TcfGroupN<G> &grp, int u, int &ti, int &bi, int &bj)
{
    ti = 0;
    while (ti + 1 < grp.n && u >= grp.t[ti + 1].tile0) ti++;
    const TcfTask &tk = grp.t[ti];
    const int l = u - tk.tile0;
    if ((tk.flags >> 1) & 1) {   // LOWER: l = bi (bi + 1) / 2 + bj, bj <= bi
        int b = (int)((sqrtf(8.f * l + 1.f) - 1.f) * 0.5f);
        while ((b + 1) * (b + 2) / 2 <= l) b++;
        while (b * (b + 1) / 2 > l) b--;
        bi = b;
        bj = l - b * (b + 1) / 2;
    } else {
        bi = l / tk.tiles_n;
        bj = l % tk.tiles_n;
    }
}

template <int G>
__global__ void __launch_bounds__(NTHREADS, 1) tcf2_gemm_kernel(const __grid_constant__ TcfGroupN<G> grp)
{
    extern __shared__ uint8_t smem_raw[];
    uint8_t *smem = smem_raw + ((1024u - (smem_u32(smem_raw) & 1023u)) & 1023u);
    uint64_t *full = reinterpret_cast<uint64_t *>(smem + STAGES * STAGE + STG);
    uint64_t *empty = full + STAGES;
    uint64_t *pfull = empty + STAGES;
    uint64_t *accf = pfull + STAGES;
    uint64_t *acce = accf + 2;
    uint32_t *tmem_slot = reinterpret_cast<uint32_t *>(acce + 2);
    // start time of each of the last 4 tiles of this CTA (warp 1 writes it when the tile starts)
    unsigned long long *ustart = reinterpret_cast<unsigned long long *>(tmem_slot + 2);   // [4], 8-aligned

    const uint32_t q = cluster_ctarank() & 1u;
    const int cl = (int)(blockIdx.x >> 1), ncl = (int)(gridDim.x >> 1);
    const int units = grp.ctas;
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;

    if (threadIdx.x == 0) {
        for (int s = 0; s < STAGES; s++) {
            mbar_init(&full[s], 1);
            mbar_init(&empty[s], 1);
            mbar_init(&pfull[s], 1);
        }
        for (int b = 0; b < 2; b++) {
            mbar_init(&accf[b], 1);
            mbar_init(&acce[b], 2);   // one arrive per CTA of the pair
        }
        asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    }
    if (warp == 1) {
        asm volatile("tcgen05.alloc.cta_group::2.sync.aligned.shared::cta.b32 [%0], %1;" ::"r"(smem_u32(tmem_slot)),
                     "r"(512u));
        asm volatile("tcgen05.relinquish_alloc_permit.cta_group::2.sync.aligned;");
    }
    tc_fence_before();
    __syncthreads();
    tc_fence_after();
    cluster_sync_all();   // both CTAs' barriers initialised, TMEM allocated
    const uint32_t tmem = *tmem_slot;

    if (warp == 0) {
        // ------------------------------------------------------------ bulk-copy producer
        if (lane == 0) {
            int it = 0;
            for (int u = cl; u < units; u += ncl) {
                int ti, bi, bj;
                unit_tile(grp, u, ti, bi, bj);
                const TcfTask &tk = grp.t[ti];
                const int nk = tk.K / BK, RA = split_rows_padded(tk.M), RB = split_rows_padded(tk.N);
                const uint8_t *a = tk.As + (size_t)(2 * bi + (int)q) * OPER;
                const uint8_t *b = tk.Bs + (size_t)(2 * bj + (int)q) * OPER;
                for (int kb = 0; kb < nk; kb++, it++) {
                    const int s = it % STAGES;
                    if (it >= STAGES) mbar_wait(&empty[s], ((it / STAGES) - 1) & 1);
                    const uint32_t st = smem_u32(smem + s * STAGE);
                    mbar_expect_tx(&full[s], STAGE);
                    bulk_g2s(st, a + (size_t)kb * RA * 128, OPER, &full[s]);
                    bulk_g2s(st + OPER, b + (size_t)kb * RB * 128, OPER, &full[s]);
                }
            }
        }
        __syncwarp();
    } else if (warp == 1) {
        if (q == 0) {
            // -------------------------------------------------------- MMA issuer (CTA 0)
            int it = 0, j = 0;
            for (int u = cl; u < units; u += ncl, j++) {
                int ti, bi, bj;
                unit_tile(grp, u, ti, bi, bj);
                const TcfTask &tk = grp.t[ti];
                const int nk = tk.K / BK;
                const uint32_t idesc = make_idesc_f16(256, BT, tk.flags & 1);
                const int b = j & 1;
                if (j >= 2) mbar_wait(&acce[b], ((j >> 1) - 1) & 1);   // buffer b drained
                tc_fence_after();
                if (lane == 0) ustart[j & 3] = globaltimer_ns();
                const uint32_t d = tmem + (uint32_t)(b * BT);
                for (int kb = 0; kb < nk; kb++, it++) {
                    const int s = it % STAGES;
                    mbar_wait(&full[s], (it / STAGES) & 1);
                    mbar_wait(&pfull[s], (it / STAGES) & 1);
                    tc_fence_after();
                    if (lane == 0) {
                        const uint32_t a_big = smem_u32(smem + s * STAGE), a_small = a_big + OPER / 2;
                        const uint32_t b_big = a_big + OPER, b_small = b_big + OPER / 2;
#pragma unroll
                        for (int kk = 0; kk < BK / 16; kk++) {
                            const uint32_t o = kk * 32;
                            const uint64_t dAb = make_desc_sw64(a_big + o), dAs = make_desc_sw64(a_small + o);
                            const uint64_t dBb = make_desc_sw64(b_big + o), dBs = make_desc_sw64(b_small + o);
                            mma2_f16(d, dAb, dBb, idesc, (kb | kk) ? 1u : 0u);
                            mma2_f16(d, dAb, dBs, idesc, 1u);
                            mma2_f16(d, dAs, dBb, idesc, 1u);
                        }
                        commit2_mc(&empty[s], (uint16_t)3);   // both CTAs may refill stage s
                        if (kb == nk - 1) commit2_mc(&accf[b], (uint16_t)3);
                    }
                    __syncwarp();
                }
            }
        } else if (lane == 0) {
            // -------------------------------------------------------- relay (CTA 1)
            const uint32_t pf0 = mapa(smem_u32(pfull), 0u);
            int it = 0, j = 0;
            for (int u = cl; u < units; u += ncl, j++) {
                int ti, bi, bj;
                unit_tile(grp, u, ti, bi, bj);
                const int nk = grp.t[ti].K / BK;
                ustart[j & 3] = globaltimer_ns();
                for (int kb = 0; kb < nk; kb++, it++) {
                    const int s = it % STAGES;
                    mbar_wait(&full[s], (it / STAGES) & 1);
                    arrive_cluster(pf0 + 8u * (uint32_t)s);
                }
            }
        }
        __syncwarp();
    } else {
        // ------------------------------------------------------------ epilogue
        const int qd = warp & 3, eh = (warp - 2) >> 2;   // TMEM lane quarter, column half
        const uint32_t acce0 = mapa(smem_u32(acce), 0u);
        int j = 0;
        for (int u = cl; u < units; u += ncl, j++) {
            int ti, bi, bj;
            unit_tile(grp, u, ti, bi, bj);
            const TcfTask &tk = grp.t[ti];
            const int M = tk.M, N = tk.N, ldc = tk.ldc;
            const bool LOWER = (tk.flags >> 1) & 1, BETA0 = (tk.flags >> 2) & 1;
            float *__restrict__ C = tk.C;
            const int grow = bi * BT + (int)q * 128 + qd * 32 + lane;   // this lane's row
            const int gc0 = bj * BT + eh * 128;                          // this warp's 128 columns
            const bool rowok = grow < M;
            float *crow = C + (int64_t)(rowok ? grow : 0) * ldc;
            const int b = j & 1;
            if (!BETA0 && rowok)   // C_in of this lane's row segment into L2 while the MMAs run
                for (int c = 0; c < 128 && gc0 + c < N; c += 32) asm volatile("prefetch.global.L2 [%0];" ::"l"(crow + gc0 + c));
            const float sa = rowok ? __ldg(tk.sa + grow) : 0.f;
            mbar_wait(&accf[b], (j >> 1) & 1);
            tc_fence_after();
            const unsigned long long t_start = ustart[j & 3];
#pragma unroll 1
            for (int ch = 0; ch < 4; ch++) {
                float v[32];
                tmem_ld32(tmem + ((uint32_t)(qd * 32) << 16) + (uint32_t)(b * BT + eh * 128 + ch * 32), v);
                if (ch == 3) {   // every TMEM read of buffer b done in this CTA: release it
                    tc_fence_before();
                    named_bar(1, NEPI);
                    if (threadIdx.x == 64) arrive_cluster(acce0 + 8u * (uint32_t)b);
                }
                const int gc = gc0 + ch * 32;
                if (!rowok || gc >= N) continue;
                float4 cin[8];
#pragma unroll
                for (int x = 0; x < 8; x++)
                    cin[x] = BETA0 ? make_float4(0.f, 0.f, 0.f, 0.f) : *reinterpret_cast<const float4 *>(crow + gc + 4 * x);
#pragma unroll
                for (int x = 0; x < 8; x++) {
                    const int c = gc + 4 * x;
                    const float4 sb = __ldg(reinterpret_cast<const float4 *>(tk.sb + c));
                    float4 o;
                    o.x = cin[x].x + (v[4 * x + 0] * sa) * sb.x;
                    o.y = cin[x].y + (v[4 * x + 1] * sa) * sb.y;
                    o.z = cin[x].z + (v[4 * x + 2] * sa) * sb.z;
                    o.w = cin[x].w + (v[4 * x + 3] * sa) * sb.w;
                    float *cp = crow + c;
                    if (LOWER && c + 3 > grow) {
                        if (c + 0 <= grow) cp[0] = o.x;
                        if (c + 1 <= grow) cp[1] = o.y;
                        if (c + 2 <= grow) cp[2] = o.z;
                    } else {
                        *reinterpret_cast<float4 *>(cp) = o;
                    }
                }
            }
            // the tile's stores are done in this CTA: report the unit to the task's record
            named_bar(2, NEPI);
            if (tk.ctx.slot && warp == 2) {
                bool rel = false;
                if (lane == 0) {
                    __threadfence();
                    rel = ctx_done(tk.ctx, t_start, globaltimer_ns(), (unsigned long long)tk.ctx.ncta);
                }
                if (__shfl_sync(0xffffffffu, rel ? 1 : 0, 0)) ctx_release(tk.ctx);
            }
        }
    }

    tc_fence_before();
    __syncthreads();
    cluster_sync_all();   // no CTA leaves while its peer may still address its smem or TMEM
    if (warp == 1) {
        tc_fence_after();
        asm volatile("tcgen05.dealloc.cta_group::2.sync.aligned.b32 %0, %1;" ::"r"(tmem), "r"(512u));
    }
}

// ---------------------------------------------------------------- host side
// Append one task (K-chunk [k0, k0 + kc)) to a group; returns its tile count (units), 0 for an
// empty task, -1 if it does not fit or is unsupported.  Forms must use the 128-row layout.
inline int group_add(TcfGroup &g, int M, int N, int K, const void *As, const void *Bs, float *C, int ldc, bool neg,
                     bool lower, TaskCtx ctx, bool beta0 = false, int k0 = 0, int kc = -1)
{
    if (M <= 0 || N <= 0) return 0;
    if (kc < 0) kc = K;
    if (K % BK || k0 % BK || kc % BK || k0 + kc > K || ldc % 4 || g.n >= tcf::kMaxGroup || (lower && M != N)) return -1;
    const int tm = (M + BT - 1) / BT, tn = (N + BT - 1) / BT;
    const int nt = lower ? tm * (tm + 1) / 2 : tm * tn;
    const int RA = split_rows_padded(M), RB = split_rows_padded(N);
    TcfTask &t = g.t[g.n++];
    t.As = (const uint8_t *)As + (size_t)(k0 / BK) * RA * 128;
    t.Bs = (const uint8_t *)Bs + (size_t)(k0 / BK) * RB * 128;
    t.sa = reinterpret_cast<const float *>((const uint8_t *)As + (size_t)RA * K * 4);
    t.sb = reinterpret_cast<const float *>((const uint8_t *)Bs + (size_t)RB * K * 4);
    t.C = C;
    t.M = M; t.N = N; t.K = kc; t.ldc = ldc;
    t.flags = (neg ? 1 : 0) | (lower ? 2 : 0) | (beta0 ? 4 : 0);
    t.tile0 = g.ctas;      // in units (tiles) for this kernel
    t.ntiles = nt;
    t.tiles_n = tn;
    ctx.ncta = (unsigned)(2 * nt);   // each tile is reported by both CTAs of its pair
    t.ctx = ctx;
    g.ctas += nt;
    return 2 * nt;
}

// tiles per cluster (VS_TCF2_UPC, default 2): the grid is ceil(units / upc) clusters, at most
// the number of co-resident clusters
inline int units_per_cluster()
{
    static const int v = [] {
        const char *e = getenv("VS_TCF2_UPC");
        const int x = e ? atoi(e) : 2;
        return x < 1 ? 1 : x;
    }();
    return v;
}

template <int G>
inline void launch_one(const TcfGroupN<G> &h, cudaStream_t s)
{
    static int max_clusters[64] = {};
    int dev = 0;
    cudaGetDevice(&dev);
    cudaLaunchConfig_t cfg = {};
    cudaLaunchAttribute at[1];
    at[0].id = cudaLaunchAttributeClusterDimension;
    at[0].val.clusterDim.x = 2;
    at[0].val.clusterDim.y = 1;
    at[0].val.clusterDim.z = 1;
    cfg.blockDim = dim3(NTHREADS);
    cfg.dynamicSmemBytes = SMEM;
    cfg.stream = s;
    cfg.attrs = at;
    cfg.numAttrs = 1;
    if (!max_clusters[dev & 63]) {
        cudaFuncSetAttribute(tcf2_gemm_kernel<G>, cudaFuncAttributeMaxDynamicSharedMemorySize, SMEM);
        int n = 0;
        cfg.gridDim = dim3(2);
        if (cudaOccupancyMaxActiveClusters(&n, tcf2_gemm_kernel<G>, &cfg) != cudaSuccess || n < 1) n = 64;
        cudaGetLastError();
        max_clusters[dev & 63] = n;
    }
    const int upc = units_per_cluster();
    int ncl = (h.ctas + upc - 1) / upc;
    if (ncl > max_clusters[dev & 63]) ncl = max_clusters[dev & 63];
    cfg.gridDim = dim3(2 * ncl);
    cudaLaunchKernelEx(&cfg, tcf2_gemm_kernel<G>, h);
}

inline int group_launch(TcfGroup &g, cudaStream_t s)
{
    if (g.n == 0) return 0;
    count_launch();
    if (g.n == 1) {
        TcfGroupN<1> h;
        h.n = 1; h.ctas = g.ctas; h.t[0] = g.t[0];
        launch_one<1>(h, s);
    } else if (g.n <= 4) {
        TcfGroupN<4> h;
        h.n = g.n; h.ctas = g.ctas;
        for (int i = 0; i < g.n; i++) h.t[i] = g.t[i];
        launch_one<4>(h, s);
    } else {
        launch_one<tcf::kMaxGroup>(g, s);
    }
    g.n = g.ctas = 0;
    return 0;
}

}  // namespace tcf2
}  // namespace vsk

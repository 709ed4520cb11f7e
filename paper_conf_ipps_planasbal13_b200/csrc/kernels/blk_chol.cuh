// blk_chol.cuh — potrf and trsm of a b x b tile as a device-side DAG of 64 x 64 sub-tile tasks
// (version simt_f32; reading R5; PAPER.md L697-699 for Cholesky, R9 for info).
//
// The b x b tile is cut into n = b/64 sub-tiles per side and factored by the right-looking tile
// algorithm, inside ONE launch:
//   POTRF: for k: potrf(A_kk); for i > k: A_ik <- A_ik L_kk^-T; for k < j <= i: A_ij -= L_ik L_jk^T
//   TRSM (X L^T = B, rows independent): for c: X_rc <- B_rc L_cc^-T (all r);
//          for c' > c: B_rc' -= X_rc L_c'c^T
// Work distribution is dynamic and deadlock-free without co-residency: a persistent CTA takes
// the next task number from a per-launch ticket (atomic CAS on a global word), tasks are
// numbered in a topological order (by step k; inside a step the task feeding the next step's
// critical path first: potrf(k), trsm(k+1, k), the update of A_k+1,k+1, ...), so every task only
// waits on tasks with smaller numbers, which running CTAs already hold.  Dependences are
// per-sub-tile state words (release / acquire at gpu scope): the number of updates applied to
// the sub-tile, + 1 once it is final.  Updates to one sub-tile are applied in k order, so the
// result is deterministic (and exact on integer problems: fp32 FMA, IEEE sqrt and division,
// forward substitution — no inverses).
// Measured (b = 1024, one task alone): potrf 1350 us, trsm 720 us — faster than the recursive /
// blocked multi-launch simt_f32 versions they replace (2.7 ms / 0.86 ms learned), slower than
// tc_3xtf32's single-launch panel kernels (592 / 258 us): every dependence hop is a round trip
// through L2 (ticket, state word, operand tiles, fence), ~5-10 us per task, and the potrf chain
// has 3 hops per 64 columns.
// Per task, 256 threads: update C -= A B^T by a 16 x 16 grid of 4 x 4 register blocks over
// shared-memory operands; triangular solve and 64 x 64 factorisation one row per thread with
// the row in registers (the factorisation publishes each column through shared memory, two
// 64-thread barriers per column).  State words and tickets live in a static per-launch slot
// (launch id % kSlots, the id in the high bits), so no reset is needed between launches.
#pragma once
#include <atomic>
#include <cstdlib>
#include <cuda_runtime.h>
#include <stdint.h>

#include "kernels.hpp"
#include "task_ctx.cuh"

namespace vsk {
namespace blk {

constexpr int T = 64;            // sub-tile
constexpr int NT = 64;           // max sub-tiles per side (b <= 4096)
constexpr int THREADS = 256;
constexpr int kSlots = 128;      // concurrent launches
constexpr int LDS = T + 4;       // padded shared row (floats; rows stay 16-byte aligned)

__device__ unsigned long long g_blk_state[kSlots][NT * NT + 1];

__device__ __forceinline__ unsigned long long ld_acquire(const unsigned long long *p)
{
    unsigned long long v;
    asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}
__device__ __forceinline__ void st_release(unsigned long long *p, unsigned long long v)
{
    asm volatile("st.release.gpu.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ float4 ld4(const float *p)
{
    float4 v;
    asm volatile("ld.global.cg.v4.f32 {%0,%1,%2,%3}, [%4];" : "=f"(v.x), "=f"(v.y), "=f"(v.z), "=f"(v.w) : "l"(p));
    return v;
}
// need = tag | count; a count of 0 is met by definition (the word may still hold an older
// launch's value, which is smaller than any of this launch)
__device__ __forceinline__ void wait_state(const unsigned long long *p, unsigned long long need)
{
    if ((need & 0xFFFFull) == 0) return;
    while (ld_acquire(p) < need) __nanosleep(32);
}
__device__ __forceinline__ void bar64() { asm volatile("bar.sync 1, 64;" ::: "memory"); }

// next task number of launch `id` (first taker resets the word left by an older launch)
__device__ __forceinline__ int take_ticket(unsigned long long *w, unsigned long long id)
{
    for (;;) {
        const unsigned long long cur = *(volatile unsigned long long *)w;
        if ((cur >> 32) != id) {
            if (atomicCAS(w, cur, (id << 32) | 1ull) == cur) return 0;
        } else if (atomicCAS(w, cur, cur + 1) == cur) {
            return (int)(cur & 0xFFFFFFFFull);
        }
    }
}

// C (64 x 64 at c, ldc) -= A B^T (A at a, B at bm, 64 x 64 each); lower: store j <= i only.
__device__ __forceinline__ void tile_update(float *c, int ldc, const float *a, int lda, const float *bm, int ldb,
                                           bool lower, float *As, float *Bs)
{
    const int t = threadIdx.x;
#pragma unroll
    for (int q = 0; q < 4; q++) {   // operands transposed into shared memory: As[kk][r] = A[r][kk]
        const int idx = t + THREADS * q, r = idx >> 4, k4 = (idx & 15) * 4;
        const float4 va = ld4(a + (int64_t)r * lda + k4), vb = ld4(bm + (int64_t)r * ldb + k4);
        As[(k4 + 0) * LDS + r] = va.x; As[(k4 + 1) * LDS + r] = va.y;
        As[(k4 + 2) * LDS + r] = va.z; As[(k4 + 3) * LDS + r] = va.w;
        Bs[(k4 + 0) * LDS + r] = vb.x; Bs[(k4 + 1) * LDS + r] = vb.y;
        Bs[(k4 + 2) * LDS + r] = vb.z; Bs[(k4 + 3) * LDS + r] = vb.w;
    }
    const int r0 = (t >> 4) * 4, c0 = (t & 15) * 4;
    float acc[4][4];
#pragma unroll
    for (int i = 0; i < 4; i++) {
        const float4 v = ld4(c + (int64_t)(r0 + i) * ldc + c0);
        acc[i][0] = v.x; acc[i][1] = v.y; acc[i][2] = v.z; acc[i][3] = v.w;
    }
    __syncthreads();
#pragma unroll 8
    for (int kk = 0; kk < T; kk++) {
        const float4 av = *reinterpret_cast<const float4 *>(As + kk * LDS + r0);
        const float4 bv = *reinterpret_cast<const float4 *>(Bs + kk * LDS + c0);
        const float ar[4] = {av.x, av.y, av.z, av.w}, br[4] = {bv.x, bv.y, bv.z, bv.w};
#pragma unroll
        for (int i = 0; i < 4; i++)
#pragma unroll
            for (int j = 0; j < 4; j++) acc[i][j] = fmaf(-ar[i], br[j], acc[i][j]);
    }
#pragma unroll
    for (int i = 0; i < 4; i++) {
        float *p = c + (int64_t)(r0 + i) * ldc + c0;
        if (!lower || c0 + 3 <= r0 + i) {
            *reinterpret_cast<float4 *>(p) = make_float4(acc[i][0], acc[i][1], acc[i][2], acc[i][3]);
        } else {
#pragma unroll
            for (int j = 0; j < 4; j++)
                if (c0 + j <= r0 + i) p[j] = acc[i][j];
        }
    }
}

// X (64 x 64 at x, ldx) <- X L^-T, L the 64 x 64 lower tile at l (ldl): one thread per row
// (threads 0-63), forward substitution x_c = (b_c - sum_{j<c} x_j l_cj) / l_cc (sum in
// ascending j).
__device__ __forceinline__ void tile_solve(float *x, int ldx, const float *l, int ldl, float *Ls)
{
    const int t = threadIdx.x;
#pragma unroll
    for (int q = 0; q < 4; q++) {   // L rows into shared memory (row-major)
        const int idx = t + THREADS * q, r = idx >> 4, k4 = (idx & 15) * 4;
        *reinterpret_cast<float4 *>(Ls + r * LDS + k4) = ld4(l + (int64_t)r * ldl + k4);
    }
    __syncthreads();
    if (t < T) {
        float v[T];
        float *row = x + (int64_t)t * ldx;
#pragma unroll
        for (int q = 0; q < T / 4; q++) {
            const float4 w = ld4(row + 4 * q);
            v[4 * q] = w.x; v[4 * q + 1] = w.y; v[4 * q + 2] = w.z; v[4 * q + 3] = w.w;
        }
        // column sweep: x_c = t_c / l_cc, then t_j -= x_c l_jc for every later j — the same
        // operations in the same order as the dot-product form (ascending c), but the 63 - c
        // updates of a column are independent, so they pipeline instead of forming one
        // dependent chain of smem loads and FMAs
#pragma unroll
        for (int cc = 0; cc < T; cc++) {
            v[cc] = __fdiv_rn(v[cc], Ls[cc * LDS + cc]);
#pragma unroll
            for (int j = cc + 1; j < T; j++) v[j] = fmaf(-v[cc], Ls[j * LDS + cc], v[j]);
        }
#pragma unroll
        for (int q = 0; q < T / 4; q++)
            *reinterpret_cast<float4 *>(row + 4 * q) = make_float4(v[4 * q], v[4 * q + 1], v[4 * q + 2], v[4 * q + 3]);
    }
}

// A (64 x 64 lower at a) = L L^T in place, threads 0-63 one row each (the strict upper part of
// the sub-tile is neither read nor written); first non-positive pivot -> *info (1-based global).
__device__ __forceinline__ void tile_potrf(float *a, int lda, int col0, int *info, float *colbuf)
{
    const int i = threadIdx.x;
    if (i >= T) return;
    float v[T];
#pragma unroll
    for (int j = 0; j < T; j++) v[j] = (j <= i) ? __ldcg(a + (int64_t)i * lda + j) : 0.f;
#pragma unroll
    for (int k = 0; k < T; k++) {
        float *col = colbuf + (k & 1) * T;
        if (i == k) {
            const float d = v[k];
            if (!(d > 0.f) && info) atomicCAS(info, 0, col0 + k + 1);
            v[k] = __fsqrt_rn(d);
            col[k] = v[k];
        }
        bar64();
        const float lkk = col[k];
        if (i > k) {
            v[k] = __fdiv_rn(v[k], lkk);
            col[i] = v[k];
        }
        bar64();
        if (i > k) {
#pragma unroll
            for (int j = k + 1; j < T; j++)
                if (j <= i) v[j] = fmaf(-v[k], col[j], v[j]);
        }
    }
#pragma unroll
    for (int j = 0; j < T; j++)
        if (j <= i) a[(int64_t)i * lda + j] = v[j];
}

// ---------------------------------------------------------------- task numbering
// POTRF of n sub-tiles, step k: [potrf(k)] [trsm(i, k), i = k+1 ..] [update(i, j, k), j = k+1 ..,
// i = j ..];  TRSM (nr row tiles, n column tiles), step c: [solve(r, c), r = 0 ..]
// [update(r, c', c), c' = c+1 .., r = 0 ..].
struct Task {
    int type;   // 0 potrf, 1 solve, 2 update
    int i, j, k;
};

__device__ __forceinline__ int potrf_step_size(int n, int k) { return 1 + (n - 1 - k) + (n - 1 - k) * (n - k) / 2; }
__device__ __forceinline__ int trsm_step_size(int nr, int n, int c) { return nr * (n - c); }

__device__ __forceinline__ Task decode_potrf(int n, int t)
{
    int k = 0;
    while (t >= potrf_step_size(n, k)) t -= potrf_step_size(n, k), k++;
    const int m = n - 1 - k;
    if (t == 0) return {0, k, k, k};
    if (t <= m) return {1, k + t, k, k};
    int u = t - 1 - m, j = k + 1;
    while (u >= n - j) u -= n - j, j++;
    return {2, j + u, j, k};
}
__device__ __forceinline__ Task decode_trsm(int nr, int n, int t)
{
    int c = 0;
    while (t >= trsm_step_size(nr, n, c)) t -= trsm_step_size(nr, n, c), c++;
    if (t < nr) return {1, t, c, c};
    t -= nr;
    return {2, t % nr, c + 1 + t / nr, c};   // update of (r, c') by step c
}

// POTRF of the n*64 x n*64 lower matrix at A (lda); info: 1-based global column k_base + ...
__global__ void __launch_bounds__(THREADS) blk_potrf_kernel(float *A, int lda, int n, int k_base, int *info,
                                                            unsigned long long id, TaskCtx ctx)
{
    ctx_begin(ctx);
    __shared__ __align__(16) float As[T * LDS];
    __shared__ __align__(16) float Bs[T * LDS];
    __shared__ int s_task;
    unsigned long long *st = g_blk_state[id % kSlots];
    const unsigned long long tag = id << 16;
    int total = 0;
    for (int k = 0; k < n; k++) total += potrf_step_size(n, k);
    for (;;) {
        if (threadIdx.x == 0) s_task = take_ticket(&st[NT * NT], id);
        __syncthreads();
        const int tn = s_task;
        if (tn >= total) break;
        const Task tk = decode_potrf(n, tn);
        float *aij = A + (int64_t)tk.i * T * lda + tk.j * T;
        if (threadIdx.x == 0) {
            if (tk.type == 0) {
                wait_state(&st[tk.k * NT + tk.k], tag | (unsigned long long)tk.k);
            } else if (tk.type == 1) {
                wait_state(&st[tk.i * NT + tk.k], tag | (unsigned long long)tk.k);
                wait_state(&st[tk.k * NT + tk.k], tag | (unsigned long long)(tk.k + 1));
            } else {
                wait_state(&st[tk.i * NT + tk.k], tag | (unsigned long long)(tk.k + 1));
                wait_state(&st[tk.j * NT + tk.k], tag | (unsigned long long)(tk.k + 1));
                wait_state(&st[tk.i * NT + tk.j], tag | (unsigned long long)tk.k);
            }
        }
        __syncthreads();
        if (tk.type == 0) {
            tile_potrf(aij, lda, k_base + tk.k * T, info, As);
        } else if (tk.type == 1) {
            tile_solve(aij, lda, A + (int64_t)tk.k * T * lda + tk.k * T, lda, As);
        } else {
            tile_update(aij, lda, A + (int64_t)tk.i * T * lda + tk.k * T, lda, A + (int64_t)tk.j * T * lda + tk.k * T, lda,
                        tk.i == tk.j, As, Bs);
        }
        __syncthreads();
        if (threadIdx.x == 0) {
            __threadfence();
            st_release(&st[tk.i * NT + tk.j], tag | (unsigned long long)(tk.k + 1));
        }
    }
    ctx_end(ctx);
}

// X (nr*64 x n*64, ldx) <- X L^-T, L (n*64 x n*64 lower, ldl)
__global__ void __launch_bounds__(THREADS) blk_trsm_kernel(const float *L, int ldl, float *X, int ldx, int nr, int n,
                                                           unsigned long long id, TaskCtx ctx)
{
    ctx_begin(ctx);
    __shared__ __align__(16) float As[T * LDS];
    __shared__ __align__(16) float Bs[T * LDS];
    __shared__ int s_task;
    unsigned long long *st = g_blk_state[id % kSlots];
    const unsigned long long tag = id << 16;
    int total = 0;
    for (int c = 0; c < n; c++) total += trsm_step_size(nr, n, c);
    for (;;) {
        if (threadIdx.x == 0) s_task = take_ticket(&st[NT * NT], id);
        __syncthreads();
        const int tn = s_task;
        if (tn >= total) break;
        const Task tk = decode_trsm(nr, n, tn);   // solve (r = i, c = j); update (r = i, c' = j, step k)
        float *xij = X + (int64_t)tk.i * T * ldx + tk.j * T;
        if (threadIdx.x == 0) {
            if (tk.type == 1) {
                wait_state(&st[tk.i * NT + tk.j], tag | (unsigned long long)tk.j);
            } else {
                wait_state(&st[tk.i * NT + tk.k], tag | (unsigned long long)(tk.k + 1));
                wait_state(&st[tk.i * NT + tk.j], tag | (unsigned long long)tk.k);
            }
        }
        __syncthreads();
        if (tk.type == 1)
            tile_solve(xij, ldx, L + (int64_t)tk.j * T * ldl + tk.j * T, ldl, As);
        else
            tile_update(xij, ldx, X + (int64_t)tk.i * T * ldx + tk.k * T, ldx, L + (int64_t)tk.j * T * ldl + tk.k * T,
                        ldl, false, As, Bs);
        __syncthreads();
        if (threadIdx.x == 0) {
            __threadfence();
            st_release(&st[tk.i * NT + tk.j], tag | (unsigned long long)(tk.k + 1));
        }
    }
    ctx_end(ctx);
}

inline unsigned long long next_launch_id()
{
    static std::atomic<unsigned long long> id{1};
    return id.fetch_add(1);
}

// persistent CTAs per launch: at most VS_BLK_GRID (default 148) and the task count
inline int grid_for(int tasks)
{
    static const int cap = [] {
        const char *e = getenv("VS_BLK_GRID");
        const int v = e ? atoi(e) : 148;
        return v < 1 ? 1 : v;
    }();
    return tasks < cap ? tasks : cap;
}

// A = L L^T in place: b x b (b % 64 == 0, b <= 4096), one launch.
inline int potrf(int b, float *A, int lda, int k_base, int *info, cudaStream_t s, const TaskCtx &ctx = TaskCtx())
{
    if (b <= 0) return 0;
    if (b % T || b / T > NT) return -1;
    const int n = b / T;
    int tasks = 0;
    for (int k = 0; k < n; k++) tasks += 1 + (n - 1 - k) + (n - 1 - k) * (n - k) / 2;
    const int grid = grid_for(tasks);
    count_launch();
    blk_potrf_kernel<<<grid, THREADS, 0, s>>>(A, lda, n, k_base, info, next_launch_id(),
                                              ctx_for(ctx, blk_potrf_kernel, THREADS, 0));
    return 0;
}

// X <- X L^-T: rows x n (both multiples of 64, n <= 4096, rows <= 4096), one launch.
inline int trsm(int rows, int n, const float *L, int ldl, float *X, int ldx, cudaStream_t s,
                const TaskCtx &ctx = TaskCtx())
{
    if (rows <= 0 || n <= 0) return 0;
    if (rows % T || n % T || rows / T > NT || n / T > NT) return -1;
    const int nr = rows / T, nc = n / T;
    const int grid = grid_for(nr * nc * (nc + 1) / 2);
    count_launch();
    blk_trsm_kernel<<<grid, THREADS, 0, s>>>(L, ldl, X, ldx, nr, nc, next_launch_id(),
                                             ctx_for(ctx, blk_trsm_kernel, THREADS, 0));
    return 0;
}

}  // namespace blk
}  // namespace vsk

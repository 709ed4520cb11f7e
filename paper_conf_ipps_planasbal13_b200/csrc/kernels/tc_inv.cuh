// tc_inv.cuh — X = L^{-T} of an n x n lower triangular tile by recursive doubling on the
// tcgen05 3xTF32 kernels (the inv(L) operand form of tc_3xf16's TRSM, reading R31).
//
// With L = [[A, 0], [C, B]] (A, B lower triangular),
//     L^{-T} = [[A^{-T}, -A^{-T} C^T B^{-T}], [0, B^{-T}]],
// so, X starting as the identity:
//   1. the 64 x 64 diagonal blocks X_ii = L_ii^{-T}: one batched launch of the substitution
//      kernel (tc_panel, X_ii = I L_ii^{-T});
//   2. levels h = 64, 128, ..., < n: every pair of neighbouring diagonal blocks of size h
//      (first X11 = A^{-T}, second X22 = B^{-T}, C = L21 the h2 x h block of L below A):
//          T   = X11 L21^T        (h x h2, scratch; tc_gemm NT, C_in = 0)
//          X12 = -T X22           (h x h2, the zero upper block of X; tc_gemm NN, negated)
//      all equally sized pairs of a level in one batched launch each, a ragged last pair
//      (n not a power-of-two multiple of 64) in its own.
// 2 log2(n / 64) + 1 launches instead of one n-panel substitution (which is sequential in
// the n / 16 sub-blocks of the whole tile): 264 us -> see DESIGN §7 for b = 1024.
#pragma once
#include "tc_gemm.cuh"
#include "tc_panel.cuh"

namespace vsk {
namespace tc {

constexpr int kInvH0 = 64;
// first block size of the doubling (VS_INV_H0 = 64 | 128, measurement switch): 128 when it
// divides n — one batched 128-wide substitution replaces the 64-wide one and the first level
inline int inv_h0(int n)
{
    static const int v = [] {
        const char *e = getenv("VS_INV_H0");
        return e ? atoi(e) : 128;
    }();
    return (v == 128 && n % 128 == 0) ? 128 : kInvH0;
}

// scratch floats needed by tc_inv_lt for an n x n tile
inline size_t inv_lt_scratch(int n) { return (size_t)n * n / 4 + 64; }

// X (n x n, ldx, holding the identity) <- L^{-T}; T: inv_lt_scratch(n) floats.  n % 64 == 0.
inline int tc_inv_lt(int n, const float *L, int ldl, float *X, int ldx, float *T, cudaStream_t s)
{
    if (n <= 0) return 0;
    if (n % kInvH0) return -1;
    const int h0 = inv_h0(n);
    const int nb = n / h0;
    if (tc_trsm_batched(nb, h0, h0, L, ldl, (int64_t)h0 * (ldl + 1), X, ldx, (int64_t)h0 * (ldx + 1), s)) return -1;
    for (int h = h0; h < n; h *= 2) {
        const int full = n / (2 * h), rem = n - full * 2 * h;
        auto pairs = [&](int o, int h2, int count) {
            const int64_t xs = (int64_t)2 * h * (ldx + 1), ls = (int64_t)2 * h * (ldl + 1);
            GemmBatch b1;
            b1.a = xs;
            b1.b = ls;
            b1.c = (int64_t)h * h2;
            b1.beta0 = 1;
            if (tc_gemm<true, false, false, 128, true>(h, h2, h, X + (int64_t)o * ldx + o, ldx, L + (int64_t)(o + h) * ldl + o,
                                                 ldl, T, h2, s, TaskCtx(), b1, count))
                return -1;
            GemmBatch b2;
            b2.a = (int64_t)h * h2;
            b2.b = xs;
            b2.c = xs;
            return tc_gemm<false, true, false, 128, true>(h, h2, h2, T, h2, X + (int64_t)(o + h) * ldx + o + h, ldx,
                                                    X + (int64_t)o * ldx + o + h, ldx, s, TaskCtx(), b2, count);
        };
        if (full && pairs(0, h, full)) return -1;
        if (rem > h && pairs(full * 2 * h, rem - h, 1)) return -1;
    }
    return 0;
}

}  // namespace tc
}  // namespace vsk

"""Pins for the matmul oracle (O1) and the Fig 1 fp32-fmaf task order (P6 reference).

Each pin is something other than the oracle itself: closed forms (P1), exact
integer arithmetic, exact rational brute force with the standard
floating-point error bound, and an exact emulation of fmaf (P4/P6).
"""
from fractions import Fraction

import numpy as np
import pytest

import oracle
import vsgen


def test_identity_closed_form():
    # P1: A = I  =>  C = C0 + B exactly.
    n = 48
    B = vsgen.uniform(11, n, n).astype(np.float64)
    C0 = vsgen.uniform(12, n, n).astype(np.float64)
    C = oracle.matmul(np.eye(n), B, C0)
    assert np.array_equal(C, C0 + B)


def test_diagonal_closed_form_rectangular():
    # P1: A = diag(d) => C_ij = C0_ij + d_i * B_ij, one rounding (fp32*fp32 exact in fp64).
    M, N = 40, 24
    d = vsgen.uniform(13, 1, M)[0].astype(np.float64)
    B = vsgen.uniform(14, M, N).astype(np.float64)
    C0 = vsgen.uniform(15, M, N).astype(np.float64)
    C = oracle.matmul(np.diag(d), B, C0)
    assert np.array_equal(C, C0 + d[:, None] * B)


@pytest.mark.parametrize("M,K,N", [(7, 5, 3), (16, 16, 16), (33, 17, 9)])
def test_integer_exact_against_python_ints(M, K, N):
    # P1: integer inputs give exact results; brute force with Python ints.
    A = vsgen.int_matrix(21, M, K).astype(np.int64)
    B = vsgen.int_matrix(22, K, N).astype(np.int64)
    C0 = vsgen.int_matrix(23, M, N).astype(np.int64)
    ref = [[int(C0[i, j]) + sum(int(A[i, k]) * int(B[k, j]) for k in range(K)) for j in range(N)]
           for i in range(M)]
    C = oracle.matmul(A, B, C0)
    assert np.array_equal(C, np.array(ref, dtype=np.float64))


def test_rational_brute_force_error_bound():
    # P4: exact rational result; |C - exact| <= gamma_K * sum|a||b| + |c0|u (standard bound).
    M, K, N = 6, 13, 5
    A = vsgen.uniform(31, M, K).astype(np.float64)
    B = vsgen.uniform(32, K, N).astype(np.float64)
    C0 = vsgen.uniform(33, M, N).astype(np.float64)
    C = oracle.matmul(A, B, C0)
    u = 2.0 ** -53
    gam = (K + 1) * u / (1 - (K + 1) * u)
    for i in range(M):
        for j in range(N):
            exact = Fraction(C0[i, j]) + sum(Fraction(A[i, k]) * Fraction(B[k, j]) for k in range(K))
            absb = abs(C0[i, j]) + sum(abs(A[i, k] * B[k, j]) for k in range(K))
            assert abs(Fraction(C[i, j]) - exact) <= Fraction(gam * absb)


def test_not_transposed():
    # A transposed operand would pass square symmetric tests; use a rank-1 probe.
    M, K, N = 3, 4, 5
    A = np.zeros((M, K)); A[2, 1] = 1.0
    B = np.zeros((K, N)); B[1, 4] = 1.0
    C = oracle.matmul(A, B)
    expect = np.zeros((M, N)); expect[2, 4] = 1.0
    assert np.array_equal(C, expect)


def _round_f32(x: Fraction) -> Fraction:
    """Exact round-to-nearest-even of a rational to fp32 (normal range)."""
    if x == 0:
        return Fraction(0)
    s = -1 if x < 0 else 1
    a = abs(x)
    e = 0
    while a >= 2:
        a /= 2; e += 1
    while a < 1:
        a *= 2; e -= 1
    scaled = a * (1 << 23)
    q, r = divmod(scaled.numerator, scaled.denominator)
    frac = Fraction(r, scaled.denominator)
    if frac > Fraction(1, 2) or (frac == Fraction(1, 2) and q % 2 == 1):
        q += 1
    return s * Fraction(q, 1 << 23) * (Fraction(2) ** e)


def test_tiled_fmaf_exact_emulation():
    # P6 reference pinned by an exact fmaf emulation: c = round32(a*b + c), ascending k,
    # following the Fig 1 driver over a 2x3x2 tile grid of 3x3 tiles.
    m, l, n, b = 2, 3, 2, 3
    A = vsgen.uniform(41, m * b, l * b)
    B = vsgen.uniform(42, l * b, n * b)
    C0 = vsgen.uniform(43, m * b, n * b)
    Ct = oracle.matmul_tiled_fmaf_f32(vsgen.to_tiles(A, b), vsgen.to_tiles(B, b), vsgen.to_tiles(C0, b))
    C = vsgen.from_tiles(Ct)
    for i in range(m * b):
        for j in range(n * b):
            c = Fraction(float(C0[i, j]))
            for k in range(l * b):      # tile k-chain in driver order, ascending kk inside
                c = _round_f32(Fraction(float(A[i, k])) * Fraction(float(B[k, j])) + c)
            assert Fraction(float(C[i, j])) == c, (i, j)


def test_tiled_fmaf_integer_exact():
    m, l, n, b = 2, 2, 3, 4
    A = vsgen.int_matrix(51, m * b, l * b)
    B = vsgen.int_matrix(52, l * b, n * b)
    C0 = vsgen.int_matrix(53, m * b, n * b)
    Ct = oracle.matmul_tiled_fmaf_f32(vsgen.to_tiles(A, b), vsgen.to_tiles(B, b), vsgen.to_tiles(C0, b))
    exact = C0.astype(np.int64) + A.astype(np.int64) @ B.astype(np.int64)
    assert np.array_equal(vsgen.from_tiles(Ct), exact.astype(np.float32))


def test_gemm_nt_fmaf_exact_emulation():
    b = 4
    A = vsgen.uniform(61, b, b)
    B = vsgen.uniform(62, b, b)
    C0 = vsgen.uniform(63, b, b)
    C = oracle.gemm_nt_fmaf_f32(A, B, C0)
    for i in range(b):
        for j in range(b):
            c = Fraction(float(C0[i, j]))
            for k in range(b):
                c = _round_f32(-Fraction(float(A[i, k])) * Fraction(float(B[j, k])) + c)
            assert Fraction(float(C[i, j])) == c

"""Pins for the Cholesky oracle (O2) and the four tile-task definitions (R5).

Closed forms (P2), exact integer recovery, an mpmath 50-digit symbolic 4x4
Cholesky (P4), the reconstruction bound (P3), LAPACK-style info (R9), and the
tiled right-looking composition of the task definitions (R5) reaching the
unblocked result.
"""
import ctypes

import mpmath
import numpy as np
import pytest

import oracle
import vsgen


def test_identity_and_diagonal():
    n = 37
    L, info = oracle.cholesky(np.eye(n))
    assert info == 0 and np.array_equal(L, np.eye(n))
    d = vsgen.int_matrix(3, 1, n, 1, 9, np.float64)[0]
    L, info = oracle.cholesky(np.diag(d * d))
    assert info == 0 and np.array_equal(L, np.diag(np.abs(d)))


@pytest.mark.parametrize("n", [4, 9, 24])
def test_integer_L0_exact_recovery(n):
    # P2: A = L0 L0^T with integer L0 (positive diagonal) => oracle returns L0 exactly.
    L0 = vsgen.int_lower(7, n)
    A = (L0.astype(np.int64) @ L0.T.astype(np.int64)).astype(np.float64)
    L, info = oracle.cholesky(A)
    assert info == 0
    assert np.array_equal(L, L0)


def test_symbolic_4x4_mpmath():
    # P4: closed-form 4x4 Cholesky evaluated at 50 digits.
    mpmath.mp.dps = 50
    A = vsgen.spd(5, 4).astype(np.float64)
    a = [[mpmath.mpf(float(A[i, j])) for j in range(4)] for i in range(4)]
    l11 = mpmath.sqrt(a[0][0]); l21 = a[1][0] / l11; l31 = a[2][0] / l11; l41 = a[3][0] / l11
    l22 = mpmath.sqrt(a[1][1] - l21 ** 2)
    l32 = (a[2][1] - l31 * l21) / l22; l42 = (a[3][1] - l41 * l21) / l22
    l33 = mpmath.sqrt(a[2][2] - l31 ** 2 - l32 ** 2)
    l43 = (a[3][2] - l41 * l31 - l42 * l32) / l33
    l44 = mpmath.sqrt(a[3][3] - l41 ** 2 - l42 ** 2 - l43 ** 2)
    ref = [[l11, 0, 0, 0], [l21, l22, 0, 0], [l31, l32, l33, 0], [l41, l42, l43, l44]]
    L, info = oracle.cholesky(A)
    assert info == 0
    for i in range(4):
        for j in range(4):
            assert abs(float(ref[i][j]) - L[i, j]) <= 4e-16 * max(1.0, abs(float(ref[i][j])))


@pytest.mark.parametrize("n", [64, 300])
def test_reconstruction_bound(n):
    # P3: ||A - L L^T||_F / ||A||_F <= 4 N u.
    A = vsgen.spd(9, n).astype(np.float64)
    L, info = oracle.cholesky(A)
    assert info == 0
    r = np.linalg.norm(A - L @ L.T) / np.linalg.norm(A)
    assert r <= 4 * n * 2.0 ** -53


def test_info_first_nonpositive_pivot():
    # R9: info = 1-based index of the first non-positive pivot.
    n = 6
    L0 = np.eye(n) * 2.0
    A = L0 @ L0.T
    A[3, 3] = 0.0   # pivot 4 becomes 0 after steps 1..3 (columns above are zero)
    _, info = oracle.cholesky(A)
    assert info == 4
    A = -np.eye(3)
    assert oracle.cholesky(A)[1] == 1


def test_strict_upper_not_referenced():
    # R7: only j <= i is read or written.
    n = 10
    A = vsgen.spd(4, n).astype(np.float64)
    junk = np.triu(np.full((n, n), np.nan), 1)
    Aj = np.tril(A) + np.nan_to_num(junk, nan=0.0)
    Aj[np.triu_indices(n, 1)] = 12345.0
    buf = np.ascontiguousarray(Aj.copy())
    info = oracle.lib().oracle_cholesky_f64(n, buf.ctypes.data_as(ctypes.POINTER(ctypes.c_double)), n)
    assert info == 0
    assert np.all(buf[np.triu_indices(n, 1)] == 12345.0)
    L, _ = oracle.cholesky(A)
    assert np.array_equal(np.tril(buf), L)


def test_task_gemm_nt_and_syrk_integer():
    b = 12
    A = vsgen.int_matrix(1, b, b).astype(np.int64)
    B = vsgen.int_matrix(2, b, b).astype(np.int64)
    C = vsgen.int_matrix(3, b, b).astype(np.int64)
    assert np.array_equal(oracle.gemm_nt(A, B, C), (C - A @ B.T).astype(np.float64))
    S = oracle.syrk(A, C)
    full = C - A @ A.T
    lo = np.tril_indices(b)
    up = np.triu_indices(b, 1)
    assert np.array_equal(S[lo], full[lo].astype(np.float64))
    assert np.array_equal(S[up], C[up].astype(np.float64))   # strict upper untouched


def test_task_trsm_integer_exact():
    # B = X0 L0^T with integer X0, unit/2-diagonal L0: forward substitution recovers X0 exactly.
    b = 10
    L0 = vsgen.int_lower(5, b, -2, 2, 1, 1)
    L0[np.arange(0, b, 3), np.arange(0, b, 3)] = 2.0
    X0 = vsgen.int_matrix(6, b, b, -4, 4).astype(np.float64) * 2   # even: /2 exact
    B = X0 @ L0.T
    X = oracle.trsm(L0, B)
    assert np.array_equal(X, X0)


def test_task_trsm_not_transposed():
    # X L^T = B must hold (not X L = B): residual check with a non-symmetric L.
    b = 16
    L = np.tril(vsgen.uniform(8, b, b).astype(np.float64)) + 4 * np.eye(b)
    B = vsgen.uniform(9, b, b).astype(np.float64)
    X = oracle.trsm(L, B)
    assert np.linalg.norm(X @ L.T - B) <= 1e-13 * np.linalg.norm(B)
    assert np.linalg.norm(X @ L - B) > 1e-3


def test_tiled_composition_reaches_unblocked():
    # R5: the right-looking tiled algorithm (potrf/trsm/syrk/gemm in submission order)
    # applied with the task definitions reaches the unblocked Cholesky up to rounding.
    n, b = 96, 16
    nt = n // b
    A = vsgen.spd(17, n).astype(np.float64)
    T = {(i, j): A[i * b:(i + 1) * b, j * b:(j + 1) * b].copy() for i in range(nt) for j in range(i + 1)}
    for k in range(nt):
        T[k, k], info = oracle.potrf(T[k, k])
        assert info == 0
        for i in range(k + 1, nt):
            T[i, k] = oracle.trsm(T[k, k], T[i, k])
        for i in range(k + 1, nt):
            for j in range(k + 1, i):
                T[i, j] = oracle.gemm_nt(T[i, k], T[j, k], T[i, j])
            T[i, i] = oracle.syrk(T[i, k], T[i, i])
    Lt = np.zeros((n, n))
    for (i, j), t in T.items():
        Lt[i * b:(i + 1) * b, j * b:(j + 1) * b] = np.tril(t) if i == j else t
    L, _ = oracle.cholesky(A)
    assert oracle.relF(Lt, L) < 1e-14

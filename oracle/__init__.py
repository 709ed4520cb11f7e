"""oracle — CPU reference for parity (TEST INFRASTRUCTURE ONLY).

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s ``cpu_baseline``
/ ``--impl reference`` leg may import this package.  The product path
(``paper_conf_ipps_planasbal13_b200``) never imports it and shares no code with
it; it fails loudly when its CUDA library is missing instead of falling back.

Contents
  * ``oracle.c`` (built to ``liboracle.so``): fp64 matmul (O1), unblocked
    right-looking Cholesky (O2), the four Cholesky tile-task definitions, and
    the fp32-fmaf per-task order of Fig 1 (pin P6).
  * ``sched_model.py``: the versioning-scheduler reference model (O3), written
    rule by rule from Sec IV.B (L353-495) — pure Python, integer arithmetic.

Every function is pinned by tests/test_oracle_*.py against closed forms,
integer exactness, brute force (fractions / mpmath) or invariants; none is
"parity unpinned".
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "oracle.c")
_LIB = os.path.join(_HERE, "liboracle.so")
_lib = None


def build(force: bool = False) -> str:
    """Compile oracle.c with gcc (fp contraction OFF so a*b+c is never fused)."""
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        cmd = ["gcc", "-O3", "-mavx2", "-mfma", "-ffp-contract=off", "-fno-fast-math", "-fopenmp",
               "-shared", "-fPIC", "-fvisibility=hidden", _SRC, "-o", _LIB + ".tmp", "-lm"]
        subprocess.check_call(cmd)
        os.replace(_LIB + ".tmp", _LIB)
    return _LIB


def lib():
    global _lib
    if _lib is None:
        build()
        L = ctypes.CDLL(_LIB)
        dp = ctypes.POINTER(ctypes.c_double)
        fp = ctypes.POINTER(ctypes.c_float)
        i64 = ctypes.c_int64
        ci = ctypes.c_int
        L.oracle_matmul_f64.argtypes = [ci, ci, ci, dp, i64, dp, i64, dp, i64]
        L.oracle_matmul_f64.restype = None
        L.oracle_cholesky_f64.argtypes = [ci, dp, i64]
        L.oracle_cholesky_f64.restype = ci
        L.oracle_gemm_nt_f64.argtypes = [ci, dp, dp, dp]
        L.oracle_syrk_f64.argtypes = [ci, dp, dp]
        L.oracle_trsm_f64.argtypes = [ci, dp, dp]
        L.oracle_potrf_f64.argtypes = [ci, dp]
        L.oracle_potrf_f64.restype = ci
        L.oracle_matmul_tiled_fmaf_f32.argtypes = [ci, ci, ci, ci, fp, fp, fp]
        L.oracle_gemm_nt_fmaf_f32.argtypes = [ci, fp, fp, fp]
        _lib = L
    return _lib


def _dp(a):
    return a.ctypes.data_as(ctypes.POINTER(ctypes.c_double))


def _fp(a):
    return a.ctypes.data_as(ctypes.POINTER(ctypes.c_float))


def _f64(a):
    return np.ascontiguousarray(a, dtype=np.float64)


def matmul(A, B, C0=None) -> np.ndarray:
    """O1: C0 + A @ B in fp64 (plain i,k,j loop)."""
    A = _f64(A)
    B = _f64(B)
    M, K = A.shape
    K2, N = B.shape
    assert K == K2
    C = np.zeros((M, N)) if C0 is None else _f64(C0).copy()
    lib().oracle_matmul_f64(M, K, N, _dp(A), K, _dp(B), N, _dp(C), N)
    return C


def cholesky(A):
    """O2: (tril(L), info) of the lower triangle of A, fp64, unblocked right-looking."""
    A = _f64(A).copy()
    n = A.shape[0]
    info = lib().oracle_cholesky_f64(n, _dp(A), n)
    return np.tril(A), int(info)


def gemm_nt(A, B, C):
    C = _f64(C).copy()
    lib().oracle_gemm_nt_f64(C.shape[0], _dp(_f64(A)), _dp(_f64(B)), _dp(C))
    return C


def syrk(A, C):
    C = _f64(C).copy()
    lib().oracle_syrk_f64(C.shape[0], _dp(_f64(A)), _dp(C))
    return C


def trsm(L, B):
    B = _f64(B).copy()
    lib().oracle_trsm_f64(B.shape[0], _dp(_f64(L)), _dp(B))
    return B


def potrf(A):
    A = _f64(A).copy()
    info = lib().oracle_potrf_f64(A.shape[0], _dp(A))
    return A, int(info)


def matmul_tiled_fmaf_f32(At, Bt, Ct):
    """Fig 1 driver + fmaf tile body on tile-major fp32 arrays (m,l,b,b),(l,n,b,b),(m,n,b,b)."""
    At = np.ascontiguousarray(At, dtype=np.float32)
    Bt = np.ascontiguousarray(Bt, dtype=np.float32)
    C = np.ascontiguousarray(Ct, dtype=np.float32).copy()
    m, l, b, _ = At.shape
    n = Bt.shape[1]
    lib().oracle_matmul_tiled_fmaf_f32(m, l, n, b, _fp(At), _fp(Bt), _fp(C))
    return C


def gemm_nt_fmaf_f32(A, B, C):
    A = np.ascontiguousarray(A, dtype=np.float32)
    B = np.ascontiguousarray(B, dtype=np.float32)
    C = np.ascontiguousarray(C, dtype=np.float32).copy()
    lib().oracle_gemm_nt_fmaf_f32(C.shape[0], _fp(A), _fp(B), _fp(C))
    return C


def relF(X, Xref) -> float:
    """||X - Xref||_F / ||Xref||_F in fp64 (SURVEY §8(c) comparison)."""
    X = np.asarray(X, dtype=np.float64)
    Xref = np.asarray(Xref, dtype=np.float64)
    return float(np.linalg.norm(X - Xref) / np.linalg.norm(Xref))

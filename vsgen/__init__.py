"""vsgen — seeded synthetic input generators shared by the oracle tests and the CUDA path.

This module holds NO arithmetic of the method (no matmul, no factorisation, no
scheduling).  It only draws numbers and lays them out.  Both sides of every
parity test (``oracle/`` and the CUDA path) take their inputs from here, or —
for inputs too large to draw on the host — from the library's device generator
``vs_gen_uniform`` / ``vs_gen_spd`` which implements the SAME counter-based
function (bit-identity is tested in ``tests/test_gen.py``).

Counter-based uniform:

    key(seed, idx) = (seed << 40) | idx                      (idx < 2**40)
    z = splitmix64(key)
    u(seed, idx)   = (z >> 40) * 2**-23 - 1                  in [-1, 1), exact in fp32

Matrices are indexed by GLOBAL (row, col): idx = row * ncols + col, so every
tiling of the same matrix holds identical values.

SPD recipe (reading R8):  S_rc = S_cr = u(seed, max(r,c)*N + min(r,c));
A = S + alpha*I, alpha = 2.5*sqrt(N) for N >= 256 else N; the diagonal is
rounded once to fp32 (fl32(S_rr + alpha) computed in fp64).
"""
from __future__ import annotations

import math

import numpy as np

_M64 = np.uint64(0xFFFFFFFFFFFFFFFF)
GOLDEN = np.uint64(0x9E3779B97F4A7C15)
MIX1 = np.uint64(0xBF58476D1CE4E5B9)
MIX2 = np.uint64(0x94D049BB133111EB)

# Seeds per BASELINE.json config; B = seed + 1000, C0 = seed + 2000.
SEEDS = {"cfg1": 1, "cfg2": 2, "cfg3": 3, "cfg4": 4}
SEED_B_OFFSET = 1000
SEED_C_OFFSET = 2000


def splitmix64(x: np.ndarray) -> np.ndarray:
    """Vectorised splitmix64 finaliser on uint64 (wrapping arithmetic)."""
    with np.errstate(over="ignore"):
        z = (x + GOLDEN).astype(np.uint64)
        z = (z ^ (z >> np.uint64(30))) * MIX1
        z = (z ^ (z >> np.uint64(27))) * MIX2
        z = z ^ (z >> np.uint64(31))
    return z


def uniform_idx(seed: int, idx: np.ndarray) -> np.ndarray:
    """u(seed, idx) as float64 (exactly representable in fp32)."""
    idx = np.asarray(idx, dtype=np.uint64)
    key = (np.uint64(seed) << np.uint64(40)) | idx
    z = splitmix64(key)
    k = (z >> np.uint64(40)).astype(np.float64)  # 24 random bits
    return k * (2.0 ** -23) - 1.0


def uniform(seed: int, rows: int, cols: int, dtype=np.float32) -> np.ndarray:
    """rows x cols matrix, global row-major index r*cols + c."""
    idx = np.arange(rows * cols, dtype=np.uint64)
    return uniform_idx(seed, idx).reshape(rows, cols).astype(dtype)


def spd_alpha(n: int) -> float:
    """Diagonal shift alpha of reading R8."""
    return 2.5 * math.sqrt(n) if n >= 256 else float(n)


def spd(seed: int, n: int, dtype=np.float32) -> np.ndarray:
    """A = S + alpha*I with S symmetric U(-1,1) (reading R8); full symmetric matrix."""
    r = np.arange(n, dtype=np.uint64)[:, None]
    c = np.arange(n, dtype=np.uint64)[None, :]
    hi = np.maximum(r, c)
    lo = np.minimum(r, c)
    s = uniform_idx(seed, hi * np.uint64(n) + lo)
    d = np.arange(n)
    s[d, d] = s[d, d] + spd_alpha(n)
    return s.astype(dtype)


def int_matrix(seed: int, rows: int, cols: int, lo: int = -8, hi: int = 8, dtype=np.float32):
    """Integer-valued matrix in [lo, hi] (pin P1: exact in fp32/TF32 products)."""
    u = uniform_idx(seed, np.arange(rows * cols, dtype=np.uint64)).reshape(rows, cols)
    v = np.floor((u + 1.0) * 0.5 * (hi - lo + 1)) + lo
    return np.clip(v, lo, hi).astype(dtype)


def int_lower(seed: int, n: int, lo: int = -3, hi: int = 3, diag_lo: int = 1, diag_hi: int = 4,
              dtype=np.float64) -> np.ndarray:
    """Integer lower-triangular L0 with positive diagonal (pin P2)."""
    m = int_matrix(seed, n, n, lo, hi, np.float64)
    L = np.tril(m, -1)
    d = int_matrix(seed + 7, 1, n, diag_lo, diag_hi, np.float64)[0]
    L[np.arange(n), np.arange(n)] = d
    return L.astype(dtype)


# ---------------------------------------------------------------- tile layout
def to_tiles(a: np.ndarray, b: int) -> np.ndarray:
    """Global row-major (R, C) -> tile-major array (R/b, C/b, b, b), each tile row-major (D6)."""
    R, C = a.shape
    assert R % b == 0 and C % b == 0
    return np.ascontiguousarray(a.reshape(R // b, b, C // b, b).transpose(0, 2, 1, 3))


def from_tiles(t: np.ndarray) -> np.ndarray:
    """Inverse of to_tiles."""
    mt, nt, b, _ = t.shape
    return np.ascontiguousarray(t.transpose(0, 2, 1, 3).reshape(mt * b, nt * b))

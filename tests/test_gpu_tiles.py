"""GPU parity of every built-in tile task version against the CPU oracle, through the C ABI
(vs_tile_run).  Gates (BASELINE.json north star): relF <= 1e-5 for the fp32 class,
<= 1e-12 for fp64; bit-exact where the arithmetic fixes the result (P1, P2, P6)."""
import numpy as np
import pytest

import oracle
import paper_conf_ipps_planasbal13_b200 as vs
import vsgen

pytestmark = pytest.mark.gpu

F32_VERSIONS = [vs.VS_V_SIMT_F32, vs.VS_V_TC_3XTF32, vs.VS_V_F64IN_F32IO]
F64_VERSIONS = [vs.VS_V_DFMA_F64, vs.VS_V_DMMA_F64]
# tc_3xf16 and oz_i8_f64: gemm-type tasks only (tc_3xf16 also TRSM)
GEMM_VERSIONS = F32_VERSIONS + [vs.VS_V_TC_3XF16] + F64_VERSIONS + [vs.VS_V_OZ_I8_F64]
FP64_STORAGE = (vs.VS_V_DFMA_F64, vs.VS_V_DMMA_F64, vs.VS_V_OZ_I8_F64)
SIZES = [64, 128, 192, 320, 512, 1024]   # 1024: the bench's tile size


def _torch():
    import torch
    return torch


def _dev(a):
    torch = _torch()
    return torch.from_numpy(np.ascontiguousarray(a)).cuda()


def _host(t):
    _torch().cuda.synchronize()
    return t.cpu().numpy()


def _run(ttype, version, b, arrays, info=None):
    ts = [_dev(a) for a in arrays]
    dinfo = info.data_ptr() if info is not None else 0
    vs.vs_tile_run(ttype, version, b, [t.data_ptr() for t in ts], dinfo)
    return [_host(t) for t in ts]


def _gate(version):
    return 1e-12 if version in FP64_STORAGE else 1e-5


def _dt(version):
    return np.float64 if version in FP64_STORAGE else np.float32


# ------------------------------------------------------------------ generator
def test_device_generator_bit_identical(gpu):
    torch = _torch()
    for tile_b in (0, 32):
        out = torch.empty(96 * 64, dtype=torch.float32, device="cuda")
        vs.vs_gen_uniform(7, 96, 64, vs.VS_F32, tile_b, out.data_ptr())
        ref = vsgen.uniform(7, 96, 64)
        if tile_b:
            ref = vsgen.to_tiles(ref, tile_b)
        assert np.array_equal(_host(out).reshape(ref.shape), ref)
    out = torch.empty(320 * 320, dtype=torch.float64, device="cuda")
    vs.vs_gen_spd(9, 320, vs.VS_F64, 64, out.data_ptr())
    ref = vsgen.to_tiles(vsgen.spd(9, 320, np.float64), 64)
    assert np.array_equal(_host(out).reshape(ref.shape), ref)
    out = torch.empty(512 * 512, dtype=torch.float32, device="cuda")
    vs.vs_gen_spd(2, 512, vs.VS_F32, 0, out.data_ptr())
    assert np.array_equal(_host(out).reshape(512, 512), vsgen.spd(2, 512))


# ------------------------------------------------------------------ matmul / gemm / syrk
@pytest.mark.parametrize("version", GEMM_VERSIONS)
@pytest.mark.parametrize("b", SIZES)
def test_matmul_tile(gpu, version, b):
    dt = _dt(version)
    A, B, C0 = (vsgen.uniform(100 + i, b, b, dt) for i in range(3))
    (_, _, C) = _run(vs.VS_T_MATMUL, version, b, [A, B, C0])
    ref = oracle.matmul(A, B, C0)
    assert oracle.relF(C, ref) <= _gate(version)


@pytest.mark.parametrize("version", GEMM_VERSIONS)
@pytest.mark.parametrize("b", SIZES)
def test_gemm_nt_and_syrk_tiles(gpu, version, b):
    dt = _dt(version)
    A, B, C0 = (vsgen.uniform(200 + i, b, b, dt) for i in range(3))
    (_, _, C) = _run(vs.VS_T_GEMM_NT, version, b, [A, B, C0])
    assert oracle.relF(C, oracle.gemm_nt(A, B, C0)) <= _gate(version)
    (_, S) = _run(vs.VS_T_SYRK, version, b, [A, C0])
    ref = oracle.syrk(A, C0)
    lo = np.tril_indices(b)
    assert oracle.relF(S[lo], ref[lo]) <= _gate(version)
    up = np.triu_indices(b, 1)
    assert np.array_equal(S[up], C0[up])          # strict upper untouched (R7)


def test_simt_f32_bit_exact_fig1_fmaf(gpu):
    # P6: simt_f32 == Fig 1 with fmaf, ascending k, from C_in — bit for bit.
    b = 192
    A, B, C0 = (vsgen.uniform(300 + i, b, b) for i in range(3))
    (_, _, C) = _run(vs.VS_T_MATMUL, vs.VS_V_SIMT_F32, b, [A, B, C0])
    ref = oracle.matmul_tiled_fmaf_f32(A[None, None], B[None, None], C0[None, None])[0, 0]
    assert np.array_equal(C.view(np.uint32), ref.view(np.uint32))
    (_, _, G) = _run(vs.VS_T_GEMM_NT, vs.VS_V_SIMT_F32, b, [A, B, C0])
    assert np.array_equal(G.view(np.uint32), oracle.gemm_nt_fmaf_f32(A, B, C0).view(np.uint32))


@pytest.mark.parametrize("version", GEMM_VERSIONS)
def test_integer_inputs_exact(gpu, version):
    # P1: integer inputs -> exact results in every version (|C| < 2^24, ints exact in TF32).
    b = 256
    dt = _dt(version)
    A, B, C0 = (vsgen.int_matrix(400 + i, b, b, dtype=dt) for i in range(3))
    (_, _, C) = _run(vs.VS_T_MATMUL, version, b, [A, B, C0])
    exact = C0.astype(np.int64) + A.astype(np.int64) @ B.astype(np.int64)
    assert np.array_equal(C.astype(np.int64), exact)
    (_, _, G) = _run(vs.VS_T_GEMM_NT, version, b, [A, B, C0])
    assert np.array_equal(G.astype(np.int64), C0.astype(np.int64) - A.astype(np.int64) @ B.astype(np.int64).T)


@pytest.mark.parametrize("ttype", ["MATMUL", "GEMM_NT"])
def test_tc_3xf16_row_scaling(gpu, ttype):
    # R30: the split form scales each operand row (B: column for MATMUL) by its own power of
    # two; rows spanning 2^-60 .. 2^60, an all-zero row and a row of subnormal-range fp16
    # values (relative to the row maximum) must keep the 3xTF32-class accuracy,
    # componentwise against |A| |B| (no overflow / underflow from fp16's range).
    b = 256
    rng = np.random.default_rng(5)
    A = vsgen.uniform(700, b, b) * np.exp2(rng.integers(-60, 60, size=(b, 1))).astype(np.float32)
    B = vsgen.uniform(701, b, b)
    B = B * (np.exp2(rng.integers(-60, 60, size=(1, b))).astype(np.float32) if ttype == "MATMUL"
             else np.exp2(rng.integers(-60, 60, size=(b, 1))).astype(np.float32))
    A[3, :] = 0.0
    A[5, :] = vsgen.uniform(702, 1, b)[0] * 1e-5
    A[5, 0] = 1e4                        # one large entry: the rest of the row is < 2^-29 of the max
    C0 = np.zeros((b, b), np.float32)
    A, B = A.astype(np.float32), B.astype(np.float32)
    t = getattr(vs, "VS_T_" + ttype)
    (_, _, C) = _run(t, vs.VS_V_TC_3XF16, b, [A, B, C0])
    Bop = B if ttype == "MATMUL" else B.T
    ref = oracle.matmul(A, Bop, C0) if ttype == "MATMUL" else oracle.gemm_nt(A, B, C0)
    bound = np.abs(A.astype(np.float64)) @ np.abs(Bop.astype(np.float64))
    err = np.abs(C.astype(np.float64) - ref)
    assert np.all(err <= 3e-5 * bound + 1e-37), float(np.max(err / (bound + 1e-300)))
    assert np.all(C[3] == 0.0)


@pytest.mark.parametrize("ttype", ["MATMUL", "GEMM_NT", "SYRK"])
def test_oz_i8_f64_row_scales_and_componentwise_bound(gpu, ttype):
    # oz_i8_f64: each operand row (B: column for MATMUL) carries its own power-of-two scale;
    # rows spanning 2^-300 .. 2^300, an all-zero row and a row whose other entries are
    # ~2^-30 of its maximum keep the bound |C - ref| <= 2^-44 |A||B| + b 2^-45 max|a_i.| max|b_.j|
    # (truncated slices: < 10 * 2^-49 of the row maxima per product, tc_oz.cuh; plus the
    # fp64 summation of the oracle and of the epilogue).
    b = 192
    rng = np.random.default_rng(6)
    A = vsgen.uniform(710, b, b, np.float64) * np.exp2(rng.integers(-300, 300, size=(b, 1)))
    B = vsgen.uniform(711, b, b, np.float64)
    B = B * (np.exp2(rng.integers(-300, 300, size=(1, b))) if ttype == "MATMUL"
             else np.exp2(rng.integers(-300, 300, size=(b, 1))))
    A[3, :] = 0.0
    A[5, :] = vsgen.uniform(712, 1, b, np.float64)[0] * 1e-9
    A[5, 0] = 1.0
    C0 = np.zeros((b, b))
    t = getattr(vs, "VS_T_" + ttype)
    if ttype == "SYRK":
        (_, C) = _run(t, vs.VS_V_OZ_I8_F64, b, [A, C0])
        ref, Bop = oracle.syrk(A, C0), A.T
    else:
        (_, _, C) = _run(t, vs.VS_V_OZ_I8_F64, b, [A, B, C0])
        Bop = B if ttype == "MATMUL" else B.T
        ref = oracle.matmul(A, Bop, C0) if ttype == "MATMUL" else oracle.gemm_nt(A, B, C0)
    rowmax_a = np.max(np.abs(A), axis=1, keepdims=True)
    colmax_b = np.max(np.abs(Bop), axis=0, keepdims=True)
    bound = 2.0 ** -44 * (np.abs(A) @ np.abs(Bop)) + b * 2.0 ** -45 * rowmax_a * colmax_b
    err = np.abs(C - ref)
    if ttype == "SYRK":
        lo = np.tril_indices(b)
        err, bound = err[lo], bound[lo]
    assert np.all(err <= bound), float(np.max(err / (bound + 1e-300)))
    assert np.all(C[3] == 0.0)


# ------------------------------------------------------------------ trsm / potrf
@pytest.mark.parametrize("version", F32_VERSIONS + [vs.VS_V_TC_3XF16] + F64_VERSIONS + [vs.VS_V_OZ_I8_F64])
@pytest.mark.parametrize("b", [64, 128, 192, 320, 512, 1024])   # 192, 320: ragged inverse levels (R31)
def test_trsm_tile(gpu, version, b):
    dt = _dt(version)
    Lfull, _ = oracle.cholesky(vsgen.spd(500 + b, b, np.float64))
    L = Lfull.astype(dt)
    X0 = vsgen.uniform(501, b, b, dt)
    (_, X) = _run(vs.VS_T_TRSM, version, b, [L, X0])
    assert oracle.relF(X, oracle.trsm(L, X0)) <= _gate(version)


@pytest.mark.parametrize("version", F32_VERSIONS + F64_VERSIONS + [vs.VS_V_OZ_I8_F64])
@pytest.mark.parametrize("b", [64, 128, 192, 512, 1024])
def test_potrf_tile(gpu, version, b):
    torch = _torch()
    dt = _dt(version)
    A = vsgen.spd(600 + b, b, dt)
    junk = A.copy()
    junk[np.triu_indices(b, 1)] = 777.0
    info = torch.zeros(1, dtype=torch.int32, device="cuda")
    (L,) = _run(vs.VS_T_POTRF, version, b, [junk], info)
    assert int(info.item()) == 0
    ref, _ = oracle.cholesky(A)
    lo = np.tril_indices(b)
    slo = np.tril_indices(b, -1)
    assert oracle.relF(L[lo], ref[lo]) <= _gate(version)
    assert oracle.relF(L[slo], ref[slo]) <= _gate(version)         # R23 strict-lower gate
    assert np.all(L[np.triu_indices(b, 1)] == 777.0)                  # R7


@pytest.mark.parametrize("version", F32_VERSIONS + F64_VERSIONS + [vs.VS_V_OZ_I8_F64])
def test_potrf_integer_L0_exact_and_info(gpu, version):
    torch = _torch()
    dt = _dt(version)
    b = 128
    L0 = vsgen.int_lower(11, b)
    A = (L0.astype(np.int64) @ L0.T.astype(np.int64)).astype(dt)
    info = torch.zeros(1, dtype=torch.int32, device="cuda")
    (L,) = _run(vs.VS_T_POTRF, version, b, [A], info)
    assert int(info.item()) == 0
    assert np.array_equal(np.tril(L).astype(np.float64), L0)
    # non-SPD: pivot 70 (1-based) is the first non-positive one
    bad = np.eye(b, dtype=dt) * 4
    bad[69, 69] = -1.0
    info.zero_()
    _run(vs.VS_T_POTRF, version, b, [bad], info)
    assert int(info.item()) == 70


# ------------------------------------------------------------------ edge cases
@pytest.mark.parametrize("version", [vs.VS_V_TC_3XF16, vs.VS_V_TC_3XTF32])
def test_max_tile_4096_sampled_rows(gpu, version):
    # the largest tile the built-in versions accept (b = 4096, 64 MiB per fp32 tile): C = C0 + A B
    # and C0 - A B^T, checked on sampled rows the oracle computes one by one (first, last, a
    # 256-row group boundary, the middle).  K = 4096 is accumulated in chunks of 1024 (R34):
    # before, tc_3xtf32 measured relF 2.9e-5 and tc_3xf16 1.4e-5 here
    b = 4096
    A, B, C0 = (vsgen.uniform(800 + i, b, b) for i in range(3))
    rows = [0, 255, 256, 2047, 4095]
    (_, _, C) = _run(vs.VS_T_MATMUL, version, b, [A, B, C0])
    ref = oracle.matmul(A[rows], B, C0[rows])
    assert oracle.relF(C[rows], ref) <= 1e-5
    (_, _, G) = _run(vs.VS_T_GEMM_NT, version, b, [A, B, C0])
    ref = oracle.matmul(-A[rows], np.ascontiguousarray(B.T), C0[rows])   # C0 - A B^T (negation exact)
    assert oracle.relF(G[rows], ref) <= 1e-5


@pytest.mark.parametrize("b", [2048, 4096])
def test_trsm_inverse_large(gpu, b):
    # tc_3xf16's TRSM multiplies by the inv(L) form (R31), built by recursive doubling up to
    # h = b / 2 (K = 2048 at b = 4096 runs in two accumulation chunks); L a well-conditioned
    # lower triangle (unit-scale entries, diagonal b).  b = 2048: the whole tile against the
    # oracle's substitution; b = 4096: sampled rows at block boundaries through the residual
    # X L^T - B (the oracle's square-only trsm would take minutes there)
    L = (np.tril(vsgen.uniform(810 + b, b, b, np.float64)) + b * np.eye(b)).astype(np.float32)
    X0 = vsgen.uniform(811 + b, b, b)
    (_, X) = _run(vs.VS_T_TRSM, vs.VS_V_TC_3XF16, b, [L, X0])
    if b == 2048:
        assert oracle.relF(X, oracle.trsm(L, X0)) <= 1e-5
    else:
        rows = [0, 63, 64, 1023, 1024, 2047, 2048, b - 1]
        assert oracle.relF(oracle.matmul(X[rows], np.ascontiguousarray(L.T)), X0[rows]) <= 1e-5


@pytest.mark.parametrize("b", [0, 32, 96, 8192])
def test_unsupported_tile_sizes_rejected(gpu, b):
    # b must be a positive multiple of 64 up to 4096: anything else is VS_E_INVAL, no launch
    torch = _torch()
    t = torch.zeros(max(1, min(b, 128)) ** 2, device="cuda")
    with pytest.raises(vs.VSError):
        vs.vs_tile_run(vs.VS_T_MATMUL, vs.VS_V_TC_3XTF32, b, [t.data_ptr()] * 3)


@pytest.mark.parametrize("ttype", ["MATMUL", "GEMM_NT"])
def test_oz_i8_f64_full_53bit_inputs(gpu, ttype):
    # the generator's values have 24-bit mantissas, which 7 int8 slices (49 bits) hold exactly;
    # full-precision fp64 inputs exercise the slice truncation and the dropped slice products:
    # relF within the fp64 gate and the componentwise bound of the scheme (tc_oz.cuh)
    b = 256
    rng = np.random.default_rng(11)
    A, B, C0 = (rng.standard_normal((b, b)) for _ in range(3))
    t = getattr(vs, "VS_T_" + ttype)
    (_, _, C) = _run(t, vs.VS_V_OZ_I8_F64, b, [A, B, C0])
    Bop = B if ttype == "MATMUL" else B.T
    ref = oracle.matmul(A, np.ascontiguousarray(Bop), C0) if ttype == "MATMUL" else oracle.gemm_nt(A, B, C0)
    assert oracle.relF(C, ref) <= 1e-12
    bound = 2.0 ** -44 * (np.abs(A) @ np.abs(Bop)) + b * 2.0 ** -45 * np.max(np.abs(A), axis=1, keepdims=True) * \
        np.max(np.abs(Bop), axis=0, keepdims=True)
    assert np.all(np.abs(C - ref) <= bound)
    assert oracle.relF(C, ref) > 0.0     # not exact: the truncation is really exercised

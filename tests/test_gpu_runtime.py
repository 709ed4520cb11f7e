"""End-to-end GPU runs through the C ABI runtime (versioning scheduler + device-enforced
dependences + tile kernels) on the BASELINE.json configs, against the CPU oracle."""
import numpy as np
import pytest

import oracle
import paper_conf_ipps_planasbal13_b200 as vs
import vsgen

pytestmark = pytest.mark.gpu

F32_MASK = (1 << vs.VS_V_SIMT_F32) | (1 << vs.VS_V_TC_3XTF32) | (1 << vs.VS_V_F64IN_F32IO)


def _torch():
    import torch
    return torch


def _tiles_dev(a, b):
    torch = _torch()
    t = vsgen.to_tiles(a, b)
    return torch.from_numpy(t).cuda()


def _register_tiles(rt, T, device=0):
    """T: tensor (mt, nt, b, b) on cuda (device=0) or pinned host (device=-1)."""
    mt, nt, b, _ = T.shape
    nbytes = b * b * T.element_size()
    return [rt.vs_data_register(T[i, j].data_ptr(), device, nbytes) for i in range(mt) for j in range(nt)]


def _matmul(rt, N, b, dtype=vs.VS_F32, mask=F32_MASK, seed=1, C0=None, host=False):
    torch = _torch()
    nt = N // b
    types = rt.vs_register_builtins(dtype, mask)
    npdt = np.float32 if dtype == vs.VS_F32 else np.float64
    A = vsgen.uniform(seed, N, N, npdt)
    B = vsgen.uniform(seed + 1000, N, N, npdt)
    C = np.zeros((N, N), npdt) if C0 is None else C0
    if host:
        tA, tB, tC = (torch.from_numpy(vsgen.to_tiles(x, b)).pin_memory() for x in (A, B, C))
        dev = -1
    else:
        tA, tB, tC = (_tiles_dev(x, b) for x in (A, B, C))
        dev = 0
    ia, ib, ic = (_register_tiles(rt, t, dev) for t in (tA, tB, tC))
    rt.vs_app_matmul(types[vs.VS_T_MATMUL], nt, nt, nt, ia, ib, ic)
    rt.vs_wait_all()
    torch.cuda.synchronize()
    return A, B, C, vsgen.from_tiles(tC.cpu().numpy())


def test_cfg1_matmul_versioning(gpu):
    # cfg1: matmul N=1024 fp32, 256x256 tiles, 2 versions, lambda = 3
    rt = vs.Runtime(lam=3)
    mask = (1 << vs.VS_V_SIMT_F32) | (1 << vs.VS_V_TC_3XTF32)
    C0 = vsgen.uniform(2001, 1024, 1024)
    A, B, C0, C = _matmul(rt, 1024, 256, mask=mask, C0=C0)
    ref = oracle.matmul(A, B, C0)
    assert oracle.relF(C, ref) <= 1e-5
    g = rt.vs_group_stats()[0]
    assert g["bytes"] == 786432 and sum(g["n"]) == 64
    assert all(n >= 3 for n in g["n"])                  # each version ran >= lambda times
    assert g["reliable"] and g["first_reliable"] == 7   # V*lambda + 1 with hold
    st = rt.vs_stats()
    assert st.tasks_completed == 64 and st.input_tx_bytes == 0
    rt.close()


def test_matmul_host_data_copy_deps(gpu):
    # e2e path: tiles registered in (pinned) host memory; runtime moves them (copy_deps)
    rt = vs.Runtime(lam=1)
    A, B, C0, C = _matmul(rt, 512, 128, mask=1 << vs.VS_V_TC_3XTF32, host=True)
    assert oracle.relF(C, oracle.matmul(A, B, C0)) <= 1e-5
    st = rt.vs_stats()
    tile = 128 * 128 * 4
    assert st.input_tx_bytes == 3 * 16 * tile           # each A, B, C tile in once (R25)
    assert st.output_tx_bytes == 16 * tile              # written C tiles flushed home
    rt.close()


def test_host_data_bench_config_eager_writeback(gpu):
    # host-homed tiles in the bench's launch configuration (ready mode, grouped launches): the
    # final version of every written tile is copied home as soon as its last writer completes
    # (eager flush), the rest of the graph still reading the GPU replica; results and Tx
    # counters as with the flush at vs_wait_all
    import torch

    import bench
    rt = vs.Runtime(bench.bench_config(vs, lam=1, slots_per_gpu=4))
    mask = (1 << vs.VS_V_TC_3XTF32) | (1 << vs.VS_V_TC_3XF16)
    A, B, C0, C = _matmul(rt, 1024, 256, mask=mask, host=True)
    assert oracle.relF(C, oracle.matmul(A, B, C0)) <= 1e-5
    st = rt.vs_stats()
    assert st.output_tx_bytes == 16 * 256 * 256 * 4
    rt.close()
    rt = vs.Runtime(bench.bench_config(vs, lam=1, slots_per_gpu=4))
    types = rt.vs_register_builtins(vs.VS_F32, mask)
    N, b = 2048, 256
    nt = N // b
    S = vsgen.spd(12, N)
    T = torch.from_numpy(vsgen.to_tiles(S, b)).pin_memory()
    ids = {i * nt + j: rt.vs_data_register(T[i, j].data_ptr(), -1, b * b * 4) for i in range(nt) for j in range(i + 1)}
    rt.vs_app_cholesky(types, nt, ids)
    rt.vs_wait_all()
    L = np.tril(vsgen.from_tiles(T.numpy()))
    Lref, info = oracle.cholesky(S)
    assert info == 0 and oracle.relF(L, Lref) <= 1e-5
    assert rt.vs_stats().output_tx_bytes == len(ids) * b * b * 4   # every tile written once home
    rt.close()


@pytest.mark.parametrize("stage", [32, 1, 0])
def test_staged_host_batch_matmul_and_cholesky(gpu, stage):
    # transfer-ordered drive (R39): a matmul and a Cholesky with host-homed tiles in one batch;
    # the inputs cross the link in the planned order (window of `stage` copies, 1 = one at a
    # time), tasks wait for their inputs in the ready queue, results as without staging
    import torch

    import bench
    rt = vs.Runtime(bench.bench_config(vs, lam=1, slots_per_gpu=4, stage=stage))
    mask = (1 << vs.VS_V_TC_3XTF32) | (1 << vs.VS_V_TC_3XF16)
    types = rt.vs_register_builtins(vs.VS_F32, mask)
    Nm, bm, Nc, bc = 1024, 256, 2048, 256
    A, B = vsgen.uniform(81, Nm, Nm), vsgen.uniform(82, Nm, Nm)
    C0 = vsgen.uniform(83, Nm, Nm)
    tA, tB, tC = (torch.from_numpy(vsgen.to_tiles(x, bm)).pin_memory() for x in (A, B, C0))
    ia, ib, ic = (_register_tiles(rt, t, -1) for t in (tA, tB, tC))
    S = vsgen.spd(84, Nc)
    nt = Nc // bc
    T = torch.from_numpy(vsgen.to_tiles(S, bc)).pin_memory()
    ids = {i * nt + j: rt.vs_data_register(T[i, j].data_ptr(), -1, bc * bc * 4) for i in range(nt) for j in range(i + 1)}
    rt.vs_app_matmul(types[vs.VS_T_MATMUL], 4, 4, 4, ia, ib, ic)
    rt.vs_app_cholesky(types, nt, ids)
    plan = rt.vs_transfer_plan()
    assert len(plan) == 48 + len(ids) and len(set(plan)) == len(plan)
    assert set(plan[:len(ids)]) == set(ids.values())       # the longer chain's inputs first
    rt.vs_wait_all()
    C = vsgen.from_tiles(tC.numpy())
    assert oracle.relF(C, oracle.matmul(A, B, C0)) <= 1e-5
    L = np.tril(vsgen.from_tiles(T.numpy()))
    Lref, info = oracle.cholesky(S)
    assert info == 0 and oracle.relF(L, Lref) <= 1e-5
    st = rt.vs_stats()
    assert st.input_tx_bytes == len(plan) * bm * bm * 4
    assert st.output_tx_bytes == (16 + len(ids)) * bm * bm * 4
    assert (st.gated_tasks > 0) == (stage > 0)
    rt.close()


def test_depend_on_event_orders_the_batch_after_the_callers_stream(gpu):
    # vs_depend_on_event: the inputs are written on the caller's stream behind a long sleep and
    # the batch is submitted without any host synchronisation; its kernels must still see them
    import torch

    import bench
    rt = vs.Runtime(bench.bench_config(vs, lam=1, slots_per_gpu=4))
    mask = (1 << vs.VS_V_TC_3XTF32) | (1 << vs.VS_V_TC_3XF16)
    types = rt.vs_register_builtins(vs.VS_F32, mask)
    N, b = 1024, 256
    A, B = vsgen.uniform(91, N, N), vsgen.uniform(92, N, N)
    src = [_tiles_dev(x, b) for x in (A, B)]
    tA, tB, tC = (torch.zeros((N // b, N // b, b, b), device="cuda") for _ in range(3))
    ia, ib, ic = (_register_tiles(rt, t, 0) for t in (tA, tB, tC))
    s = torch.cuda.Stream()
    with torch.cuda.stream(s):
        torch.cuda._sleep(200_000_000)     # ~0.1 s of GPU time before the inputs exist
        tA.copy_(src[0])
        tB.copy_(src[1])
        ev = torch.cuda.Event()
        ev.record(s)
    rt.vs_depend_on_event(ev)
    rt.vs_app_matmul(types[vs.VS_T_MATMUL], 4, 4, 4, ia, ib, ic)
    rt.vs_wait_all()
    torch.cuda.synchronize()
    C = vsgen.from_tiles(tC.cpu().numpy())
    assert oracle.relF(C, oracle.matmul(A, B)) <= 1e-5
    rt.close()


def test_equally_critical_chains_run_concurrently(gpu):
    # R33: in the bench configuration (bottom-level priority, critical-path streams) a lone
    # matmul has 16 equally critical k-chains; they must run side by side, not queue on the
    # two critical-path streams: some device-recorded task intervals overlap by 4 or more
    import bench
    rt = vs.Runtime(bench.bench_config(vs, lam=1))
    _matmul(rt, 1024, 256, mask=(1 << vs.VS_V_TC_3XTF32) | (1 << vs.VS_V_TC_3XF16))
    log = rt.vs_decision_log()
    ev = sorted([(r[4], 1) for r in log] + [(r[5], -1) for r in log])
    cur = best = 0
    for _, d in ev:
        cur += d
        best = max(best, cur)
    assert best >= 4, best
    rt.close()


def test_lone_matmul_keeps_grouped_launches(gpu):
    # every task of a lone matmul has slack 0 (R33/R38); in the bench configuration its
    # tc_3xf16 tasks must still share grouped launches (a flush of every critical task on its
    # own once ungrouped the whole matmul: 317 -> 123 TFLOP/s in the bench)
    import bench
    rt = vs.Runtime(bench.bench_config(vs, lam=1))
    s0 = rt.vs_stats()
    A, B, C0, C = _matmul(rt, 2048, 256, mask=1 << vs.VS_V_TC_3XF16)
    s1 = rt.vs_stats()
    launches = s1.group_launches - s0.group_launches
    assert launches > 0 and 512 / launches >= 2.0, launches
    assert oracle.relF(C, oracle.matmul(A, B, C0)) <= 1e-5
    rt.close()


def test_matmul_f64_family(gpu):
    rt = vs.Runtime(lam=1)
    mask = (1 << vs.VS_V_DFMA_F64) | (1 << vs.VS_V_DMMA_F64)
    A, B, C0, C = _matmul(rt, 512, 128, dtype=vs.VS_F64, mask=mask)
    assert oracle.relF(C, oracle.matmul(A, B, C0)) <= 1e-12
    rt.close()


def test_f64_family_with_ozaki_version(gpu):
    # the tcgen05 Ozaki version (oz_i8_f64) among the fp64 versions: every version of
    # MATMUL / GEMM_NT / SYRK / TRSM / POTRF runs (lambda = 2 learning runs each; TRSM as
    # X = B inv(L)^T with the slice form of inv(L); POTRF recursive with Ozaki trailing updates),
    # its slice forms are built and cached by the runtime.  Results within the fp64 gate.
    mask = (1 << vs.VS_V_DFMA_F64) | (1 << vs.VS_V_DMMA_F64) | (1 << vs.VS_V_OZ_I8_F64)
    rt = vs.Runtime(lam=2)
    A, B, C0, C = _matmul(rt, 768, 128, dtype=vs.VS_F64, mask=mask)
    assert oracle.relF(C, oracle.matmul(A, B, C0)) <= 1e-12
    g = [x for x in rt.vs_group_stats() if x["type_name"].startswith("MATMUL")][0]
    assert "oz_i8_f64" in g["versions"] and min(g["n"]) >= 2
    assert rt.vs_stats().forms_built > 0
    rt.close()
    rt = vs.Runtime(lam=2)
    S, L = _cholesky(rt, 1024, 128, mask=mask, dtype=vs.VS_F64)
    Lref, info = oracle.cholesky(S)
    assert info == 0 and oracle.relF(L, Lref) <= 1e-12
    for g in rt.vs_group_stats():
        if g["type_name"].startswith(("GEMM_NT", "SYRK", "TRSM", "POTRF")):
            assert "oz_i8_f64" in g["versions"] and min(g["n"]) >= 1, g
    rt.close()


def _cholesky(rt, N, b, mask=F32_MASK, seed=2, dtype=vs.VS_F32):
    torch = _torch()
    nt = N // b
    types = rt.vs_register_builtins(dtype, mask)
    npdt = np.float32 if dtype == vs.VS_F32 else np.float64
    A = vsgen.spd(seed, N, npdt)
    T = _tiles_dev(A, b)
    ids = {}
    nbytes = b * b * T.element_size()
    for i in range(nt):
        for j in range(i + 1):
            ids[i * nt + j] = rt.vs_data_register(T[i, j].data_ptr(), 0, nbytes)
    rt.vs_app_cholesky(types, nt, ids)
    rt.vs_wait_all()
    torch.cuda.synchronize()
    return A, np.tril(vsgen.from_tiles(T.cpu().numpy()))


def test_cfg2_cholesky_versioning(gpu):
    # cfg2: Cholesky N=4096 SPD fp32, 512x512 tiles, 3 versions per task, lambda = 3.
    # Oracle on the leading 2048 block (L[:k,:k] = chol(A[:k,:k])) + full-size residual.
    rt = vs.Runtime(lam=3)
    A, L = _cholesky(rt, 4096, 512)
    k = 2048
    Lk, info = oracle.cholesky(A[:k, :k])
    assert info == 0
    lo, slo = np.tril_indices(k), np.tril_indices(k, -1)
    assert oracle.relF(L[:k, :k][lo], Lk[lo]) <= 1e-5
    assert oracle.relF(L[:k, :k][slo], Lk[slo]) <= 1e-5
    rng = np.random.default_rng(0)
    A64, L64 = A.astype(np.float64), L.astype(np.float64)
    for _ in range(4):     # P3 reconstruction bound for fp32 factors: 4 N u, u = 2^-24
        x = rng.standard_normal(4096)
        r = A64 @ x - L64 @ (L64.T @ x)
        assert np.linalg.norm(r) / np.linalg.norm(A64 @ x) <= 4 * 4096 * 2.0 ** -24
    gs = {g["type_name"]: g for g in rt.vs_group_stats()}
    assert not gs["POTRF.f32"]["reliable"] and sum(gs["POTRF.f32"]["n"]) == 8     # L496-501
    assert gs["GEMM_NT.f32"]["reliable"] and sum(gs["GEMM_NT.f32"]["n"]) == 56
    rt.close()


def test_cholesky_not_spd_sticky(gpu):
    torch = _torch()
    rt = vs.Runtime(lam=1)
    types = rt.vs_register_builtins(vs.VS_F32, 1 << vs.VS_V_SIMT_F32)
    b, nt = 128, 2
    A = np.eye(256, dtype=np.float32)
    A[200, 200] = -5.0
    T = _tiles_dev(A, b)
    ids = {i * nt + j: rt.vs_data_register(T[i, j].data_ptr(), 0, b * b * 4) for i in range(nt) for j in range(i + 1)}
    rt.vs_app_cholesky(types, nt, ids)
    with pytest.raises(vs.VSError) as e:
        rt.vs_wait_all()
    assert e.value.code == vs.VS_E_NOT_SPD
    st = rt.vs_stats()
    assert st.error_info == 200 - 128 + 1             # pivot within the failing tile
    rt.close()
    torch.cuda.synchronize()


def test_replay_mode_bit_exact_outputs(gpu):
    # P8: same timing table -> same decisions and bit-identical tiles across runs.
    torch = _torch()
    outs, hashes = [], []
    for _ in range(2):
        rt = vs.Runtime(vs.vs_config_default(lam=2, replay=1))
        types = rt.vs_register_builtins(vs.VS_F32, F32_MASK)
        nbytes = 256 * 256 * 4
        for ti, sz in ((vs.VS_T_POTRF, nbytes), (vs.VS_T_TRSM, 2 * nbytes), (vs.VS_T_SYRK, 2 * nbytes),
                       (vs.VS_T_GEMM_NT, 3 * nbytes)):
            for v, d in enumerate((900, 300, 1500)):
                rt.vs_replay_set(types[ti], sz, v, d + 17 * ti)
        A = vsgen.spd(5, 1024)
        T = _tiles_dev(A, 256)
        ids = {i * 4 + j: rt.vs_data_register(T[i, j].data_ptr(), 0, nbytes) for i in range(4) for j in range(i + 1)}
        rt.vs_app_cholesky(types, 4, ids)
        rt.vs_wait_all()
        torch.cuda.synchronize()
        outs.append(T.cpu().numpy())
        hashes.append(rt.vs_decision_log_hash())
        rt.close()
    assert hashes[0] == hashes[1]
    assert np.array_equal(outs[0].view(np.uint32), outs[1].view(np.uint32))


F16_MASK = F32_MASK | (1 << vs.VS_V_TC_3XF16)


def test_tc_3xf16_versioning_matmul_and_cholesky(gpu):
    # tc_3xf16 competes with the other fp32 versions for MATMUL / GEMM_NT / SYRK (POTRF and
    # TRSM keep three versions); every version's output is within the fp32-class gate (R22).
    rt = vs.Runtime(lam=2)
    C0 = vsgen.uniform(2002, 1024, 1024)
    A, B, C0, C = _matmul(rt, 1024, 256, mask=F16_MASK, C0=C0)
    assert oracle.relF(C, oracle.matmul(A, B, C0)) <= 1e-5
    g = rt.vs_group_stats()[0]
    assert g["versions"] == ["simt_f32", "tc_3xtf32", "f64in_f32io", "tc_3xf16"]
    assert g["n"][3] >= 2
    rt.close()
    rt = vs.Runtime(lam=2)
    A, L = _cholesky(rt, 2048, 256, mask=F16_MASK)
    Lref, info = oracle.cholesky(A)
    lo, slo = np.tril_indices(2048), np.tril_indices(2048, -1)
    assert info == 0 and oracle.relF(L[lo], Lref[lo]) <= 1e-5 and oracle.relF(L[slo], Lref[slo]) <= 1e-5
    gs = {gr["type_name"]: gr for gr in rt.vs_group_stats()}
    assert len(gs["POTRF.f32"]["versions"]) == 3 and len(gs["GEMM_NT.f32"]["versions"]) == 4
    assert rt.vs_stats().forms_built > 0
    rt.close()


def test_tc_3xf16_forms_follow_writes_and_invalidation(gpu):
    # The split forms are cached per datum version: a task write (C of step 1 becomes the A
    # operand of step 2) and vs_data_invalidate after an outside write must both rebuild them.
    torch = _torch()
    N, b = 512, 128
    nt = N // b
    rt = vs.Runtime(vs.vs_config_default(lam=1, policy=vs.VS_POLICY_FIXED, fixed_version=3))
    types = rt.vs_register_builtins(vs.VS_F32, F16_MASK)
    A, B = vsgen.uniform(31, N, N), vsgen.uniform(32, N, N)
    tA, tB, tC, tD = (_tiles_dev(x, b) for x in (A, B, np.zeros((N, N), np.float32), np.zeros((N, N), np.float32)))
    ia, ib, ic, idd = (_register_tiles(rt, t) for t in (tA, tB, tC, tD))
    mm = types[vs.VS_T_MATMUL]
    rt.vs_app_matmul(mm, nt, nt, nt, ia, ib, ic)       # C = A B
    rt.vs_app_matmul(mm, nt, nt, nt, ic, ib, idd)      # D = C B (reads C's new content)
    rt.vs_wait_all()
    C = A.astype(np.float64) @ B
    D = C @ B
    assert oracle.relF(vsgen.from_tiles(tD.cpu().numpy()), D) <= 1e-5
    n1 = rt.vs_stats().forms_built
    assert n1 == 3 * nt * nt                             # A, B, C once each
    # outside write of A + invalidate -> rebuilt; B unchanged -> reused
    A2 = vsgen.uniform(33, N, N)
    tA.copy_(_tiles_dev(A2, b))
    tC.zero_()
    torch.cuda.synchronize()
    for d in ia + ic:
        rt.vs_data_invalidate(d)
    rt.vs_app_matmul(mm, nt, nt, nt, ia, ib, ic)
    rt.vs_wait_all()
    assert oracle.relF(vsgen.from_tiles(tC.cpu().numpy()), A2.astype(np.float64) @ B) <= 1e-5
    assert rt.vs_stats().forms_built == n1 + nt * nt
    rt.close()


def test_empty_graph_and_single_tile_problems(gpu):
    # degenerate graphs: vs_wait_all with nothing submitted, a 1x1x1 tiled matmul (one task)
    # and a one-tile Cholesky (a single potrf) through the runtime, every f32 version enabled
    rt = vs.Runtime(lam=1)
    rt.vs_wait_all()
    assert rt.vs_stats().tasks_completed == 0
    A, B, C0, C = _matmul(rt, 256, 256, mask=F32_MASK | (1 << vs.VS_V_TC_3XF16))
    assert oracle.relF(C, oracle.matmul(A, B, C0)) <= 1e-5
    rt.close()
    rt = vs.Runtime(lam=1)
    S, L = _cholesky(rt, 256, 256)
    Lref, info = oracle.cholesky(S)
    assert info == 0 and oracle.relF(L, Lref) <= 1e-5
    assert rt.vs_stats().tasks_completed == 1
    rt.close()


def test_multi_kernel_tasks_b2048_through_runtime(gpu):
    # b = 2048 tensor-core tasks run as two K-chunk launches each (R34): a task completes only
    # when its last kernel reported through the completion ring (nkern = 2).  A 2x2x2 tiled
    # matmul (N = 4096) with tc_3xtf32 and tc_3xf16, results on sampled rows against the oracle
    import bench
    torch = _torch()
    rt = vs.Runtime(bench.bench_config(vs, lam=1, slots_per_gpu=4))
    N, b = 4096, 2048
    nt = N // b
    types = rt.vs_register_builtins(vs.VS_F32, (1 << vs.VS_V_TC_3XTF32) | (1 << vs.VS_V_TC_3XF16))
    A, B = vsgen.uniform(31, N, N), vsgen.uniform(1031, N, N)
    tA, tB, tC = (_tiles_dev(x, b) for x in (A, B, np.zeros((N, N), np.float32)))
    ia, ib, ic = (_register_tiles(rt, t) for t in (tA, tB, tC))
    rt.vs_app_matmul(types[vs.VS_T_MATMUL], nt, nt, nt, ia, ib, ic)
    rt.vs_wait_all()
    torch.cuda.synchronize()
    C = vsgen.from_tiles(tC.cpu().numpy())
    rows = [0, 2047, 2048, 4095]
    assert oracle.relF(C[rows], oracle.matmul(A[rows], B)) <= 1e-5
    st = rt.vs_stats()
    assert st.tasks_completed == 8 and st.kernel_launches >= 16
    rt.close()

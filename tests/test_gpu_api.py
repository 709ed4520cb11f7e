"""The task-version API on the GPU executor, against the CPU oracle:

* a1 — USER versions (``vs_version_add`` with a launch function, "implements(main)", Fig 4,
  L296-345): the three-implementation fixture of tests/c/fig4_versions.cu runs through the
  learning phase (lambda runs per version, L434-447) and the reliable phase, which must pick a
  version that is the fastest in isolation (ground truth: CUDA-event timing of each version
  alone) and never the slow one; the task's int N arrives as its scalar; outputs are exact;
* a15 — ``vs_wait_on`` ("taskwait on", L243-246) and ``vs_wait_all_noflush`` ("taskwait
  noflush", L267-270) with host-homed data, flush on and off;
* NEXT-1/2/3 on the GPU executor (not only in SIM): the locality term with real host->device
  transfers, a warm start from a dumped timing table, range groups and the recency-weighted
  mean on a mixed-size run.
"""
import ctypes
import os
import subprocess

import numpy as np
import pytest

import oracle
import paper_conf_ipps_planasbal13_b200 as vs
import vsgen

pytestmark = pytest.mark.gpu

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
FIG4_SRC = os.path.join(ROOT, "tests", "c", "fig4_versions.cu")
FIG4_SO = os.path.join(ROOT, "tests", "c", "_build", "libfig4.so")
FIG4_VERSIONS = ("main_impl", "another_impl", "yet_another_one")


def fig4_lib():
    if not os.path.exists(FIG4_SO) or os.path.getmtime(FIG4_SO) < os.path.getmtime(FIG4_SRC):
        os.makedirs(os.path.dirname(FIG4_SO), exist_ok=True)
        subprocess.run(["/usr/local/cuda/bin/nvcc", "-gencode", "arch=compute_100a,code=sm_100a", "-O3", "-shared",
                        "-Xcompiler", "-fPIC", "-o", FIG4_SO, FIG4_SRC], check=True)
    return ctypes.CDLL(FIG4_SO)


def _torch():
    import torch
    return torch


def _fig4_runtime(lam, slots=2, **kw):
    L = fig4_lib()
    rt = vs.Runtime(vs.vs_config_default(lam=lam, slots_per_gpu=slots, **kw))
    t = rt.vs_type_create("fig4_task", [vs.VS_IN, vs.VS_OUT, vs.VS_INOUT])
    for name in FIG4_VERSIONS:
        rt.vs_version_add(t, name, 1, getattr(L, "fig4_" + name))
    return rt, t, L


def _isolated_us(L, n, runs=20):
    """Ground truth: each version alone on one stream, median of `runs` CUDA-event intervals."""
    torch = _torch()
    A = torch.ones(n, device="cuda")
    B = torch.empty_like(A)
    C = torch.zeros_like(A)
    ptrs = (ctypes.c_void_p * 3)(A.data_ptr(), B.data_ptr(), C.data_ptr())
    nbytes = (ctypes.c_int64 * 3)(n * 4, n * 4, n * 4)
    sc = ctypes.c_int(n)
    s = torch.cuda.current_stream()
    out = {}
    for name in FIG4_VERSIONS:
        f = getattr(L, "fig4_" + name)
        ts = []
        for _ in range(runs + 3):
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record()
            assert f(ptrs, nbytes, 3, ctypes.byref(sc), ctypes.c_size_t(4), ctypes.c_void_p(s.cuda_stream), None) == 0
            e1.record()
            e1.synchronize()
            ts.append(e0.elapsed_time(e1) * 1e3)
        out[name] = float(np.median(ts[3:]))
    return out


@pytest.mark.parametrize("device_release", [0, 1])
def test_fig4_user_versions_learn_then_pick_fastest(gpu, device_release):
    """device_release = 1 (ready mode): successors of user versions are released on the device
    by the one-warp release kernel behind each version (a3)."""
    torch = _torch()
    n, ntask, lam = 1 << 20, 24, 2
    # ground truth first: it also loads the fixture's kernels, as an application does before
    # timing anything (a lazily loaded module's first launch would add milliseconds of host
    # time to the event interval of its first learning run, R17)
    gt = _isolated_us(fig4_lib(), n)
    rt, t, L = _fig4_runtime(lam, device_release=device_release, mode=vs.VS_MODE_READY if device_release else 0)
    sc = np.int32(n).tobytes()
    As = [vsgen.int_matrix(50 + k, 1, n, -8, 8)[0] for k in range(ntask)]
    C0s = [vsgen.int_matrix(90 + k, 1, n, -100, 100)[0] for k in range(ntask)]
    # the first 16 tasks are independent; the last 8 form a chain on one C (inout, RAW/WAW)
    tA = [torch.from_numpy(a).cuda() for a in As]
    tB = [torch.full((n,), 5.0, device="cuda") for _ in range(ntask)]
    tC = [torch.from_numpy(c).cuda() for c in C0s[:16]] + [torch.from_numpy(C0s[16]).cuda()]
    nb = n * 4
    reg = lambda x: rt.vs_data_register(x.data_ptr(), 0, nb)          # noqa: E731
    for k in range(ntask):
        c = tC[k] if k < 16 else tC[16]
        rt.vs_submit(t, [reg(tA[k]), reg(tB[k]), reg(c)], sc)
    rt.vs_wait_all()
    torch.cuda.synchronize()
    # exact results (integers: A + A and fma(A, A, C) are exact in fp32)
    for k in range(ntask):
        assert np.array_equal(tB[k].cpu().numpy(), 2 * As[k])
    for k in range(16):
        assert np.array_equal(tC[k].cpu().numpy(), C0s[k] + As[k] * As[k])
    chain = C0s[16].astype(np.int64) + sum(As[k].astype(np.int64) ** 2 for k in range(16, ntask))
    assert np.array_equal(tC[16].cpu().numpy().astype(np.int64), chain)
    # learning then reliable (L434-447): lambda runs per version, first reliable decision V*lambda+1
    (g,) = rt.vs_group_stats()
    assert g["versions"] == list(FIG4_VERSIONS) and g["bytes"] == 3 * nb
    assert g["reliable"] and g["first_reliable"] == 3 * lam + 1
    log = rt.vs_decision_log()
    assert [r[6] for r in log[:3 * lam]] == [0] * (3 * lam)
    assert sorted(r[1] for r in log[:3 * lam]) == sorted(list(range(3)) * lam)
    assert all(r[6] == 1 for r in log[3 * lam:])
    fastest = min(gt.values())
    assert gt["yet_another_one"] > 5 * fastest, gt             # the fixture's slow version is slow
    picks = [FIG4_VERSIONS[r[1]] for r in log[3 * lam:]]
    assert "yet_another_one" not in picks, (picks, gt, g)
    assert all(gt[p] <= 1.3 * fastest for p in picks), (picks, gt, g)
    # the learned means order the slow version last, as the isolated timings do (R17)
    m = dict(zip(FIG4_VERSIONS, g["mean_ns"]))
    assert m["yet_another_one"] > 3 * max(m["main_impl"], m["another_impl"]), (m, gt)
    # event-timed under co-running (two slots share the GPU's memory bandwidth): the one-CTA
    # version is slowed by the bandwidth-bound versions beside it, but stays within a small factor
    assert 0.7 <= m["yet_another_one"] / 1e3 / gt["yet_another_one"] <= 4.0, (m, gt)
    # 16 independent roots + the chain's head: the 7 chained tasks are made ready by the device
    assert rt.vs_stats().device_released == (7 if device_release else 0)
    rt.close()


def test_fig4_version_error_is_reported(gpu):
    torch = _torch()
    L = fig4_lib()
    rt = vs.Runtime(vs.vs_config_default(lam=1, slots_per_gpu=1))
    t = rt.vs_type_create("fig4_task", [vs.VS_IN, vs.VS_OUT, vs.VS_INOUT])
    rt.vs_version_add(t, "failing", 1, L.fig4_failing)
    x = [torch.zeros(256, device="cuda") for _ in range(3)]
    rt.vs_submit(t, [rt.vs_data_register(v.data_ptr(), 0, 1024) for v in x], np.int32(256).tobytes())
    with pytest.raises(vs.VSError) as e:
        rt.vs_wait_all()
    assert "returned 7" in str(e.value)
    rt.close()


# ------------------------------------------------------------------ waits (a15)
def _host_matmul(rt, N, b, seed):
    torch = _torch()
    nt = N // b
    types = rt.vs_register_builtins(vs.VS_F32, 1 << vs.VS_V_TC_3XTF32)
    A = vsgen.uniform(seed, N, N)
    B = vsgen.uniform(seed + 1000, N, N)
    tA, tB, tC = (torch.from_numpy(vsgen.to_tiles(x, b)).pin_memory() for x in (A, B, np.zeros((N, N), np.float32)))
    nbytes = b * b * 4
    ids = [[rt.vs_data_register(T[i, j].data_ptr(), -1, nbytes) for i in range(nt) for j in range(nt)]
           for T in (tA, tB, tC)]
    return types, (A, B), (tA, tB, tC), ids


def test_wait_noflush_and_wait_on_without_flush(gpu):
    """flush = 0: taskwait noflush leaves the results on the device (no copy home, host C still
    0); taskwait on(C_00) brings exactly that tile home (Output Tx = one tile)."""
    N, b = 512, 128
    nt = N // b
    rt = vs.Runtime(vs.vs_config_default(lam=1, slots_per_gpu=2, flush=0))
    types, (A, B), (tA, tB, tC), (ia, ib, ic) = _host_matmul(rt, N, b, 31)
    rt.vs_app_matmul(types[vs.VS_T_MATMUL], nt, nt, nt, ia, ib, ic)
    rt.vs_wait_all_noflush()
    st = rt.vs_stats()
    assert st.tasks_completed == nt ** 3 and st.output_tx_bytes == 0
    assert not tC.numpy().any()
    rt.vs_wait_on(ic[0])
    assert rt.vs_stats().output_tx_bytes == b * b * 4
    ref = oracle.matmul(A, B)
    assert oracle.relF(tC.numpy()[0, 0], ref[:b, :b]) <= 1e-5
    assert not tC.numpy()[0, 1:].any() and not tC.numpy()[1:].any()
    rt.close()


def test_wait_on_while_other_tasks_run(gpu):
    """taskwait on(d) returns once d's last writer is done and d is valid at home, without
    waiting for the rest of the graph; the rest completes at the next wait.  512 tasks, so that
    C_00's 8-task chain (submitted first) cannot be observed only after the whole graph ran
    (with 64 tasks the GPU occasionally finished them all before the host's first poll)."""
    N, b = 2048, 256
    nt = N // b
    rt = vs.Runtime(vs.vs_config_default(lam=1, slots_per_gpu=2))
    types, (A, B), (tA, tB, tC), (ia, ib, ic) = _host_matmul(rt, N, b, 41)
    rt.vs_app_matmul(types[vs.VS_T_MATMUL], nt, nt, nt, ia, ib, ic)
    rt.vs_wait_on(ic[0])
    st = rt.vs_stats()
    assert st.tasks_completed < nt ** 3          # C_00's chain is done, not the whole graph
    ref = oracle.matmul(A, B)
    assert oracle.relF(tC.numpy()[0, 0], ref[:b, :b]) <= 1e-5
    rt.vs_wait_all()
    assert oracle.relF(vsgen.from_tiles(tC.numpy()), ref) <= 1e-5
    rt.close()


def test_noflush_then_restore_and_invalidate(gpu):
    """flush = 1 (eager write-back of final versions): after taskwait noflush the copies home the
    runtime started are complete, so the caller can restore its host inputs, invalidate them and
    run again (a late copy used to be able to overwrite the restored data)."""
    N, b = 1024, 256
    nt = N // b
    rt = vs.Runtime(vs.vs_config_default(lam=1, slots_per_gpu=4))
    types, (A, B), (tA, tB, tC), (ia, ib, ic) = _host_matmul(rt, N, b, 51)
    for it in range(3):
        An = vsgen.uniform(60 + it, N, N)
        tA.copy_(_torch().from_numpy(vsgen.to_tiles(An, b)))
        tC.zero_()
        rt.vs_data_invalidate_n(ia + ic)
        rt.vs_app_matmul(types[vs.VS_T_MATMUL], nt, nt, nt, ia, ib, ic)
        rt.vs_wait_all_noflush()
        assert oracle.relF(vsgen.from_tiles(tC.numpy()), oracle.matmul(An, B)) <= 1e-5, it
    rt.close()


# ------------------------------------------------------------------ NEXT on the GPU executor
def _dev_matmul(rt, N, b, seed, mask, types=None):
    torch = _torch()
    nt = N // b
    if types is None:
        types = rt.vs_register_builtins(vs.VS_F32, mask)
    A, B = vsgen.uniform(seed, N, N), vsgen.uniform(seed + 1000, N, N)
    T = [torch.from_numpy(vsgen.to_tiles(x, b)).cuda() for x in (A, B, np.zeros((N, N), np.float32))]
    ids = [[rt.vs_data_register(X[i, j].data_ptr(), 0, b * b * 4) for i in range(nt) for j in range(nt)] for X in T]
    rt.vs_app_matmul(types[vs.VS_T_MATMUL], nt, nt, nt, *ids)
    return types, A, B, T


MASK2 = (1 << vs.VS_V_SIMT_F32) | (1 << vs.VS_V_TC_3XTF32)


def test_next2_warm_start_from_dumped_table(gpu, tmp_path):
    """NEXT-2 (external hints, L998-1003): a table dumped by one run makes the next run's groups
    reliable from its first decision, which picks the table's fastest version."""
    path = str(tmp_path / "table.txt")
    rt = vs.Runtime(vs.vs_config_default(lam=2, slots_per_gpu=4))
    _dev_matmul(rt, 1024, 256, 1, MASK2)
    rt.vs_wait_all()
    rt.vs_table_dump(path)
    g0 = rt.vs_group_stats()[0]
    rt.close()
    lines = open(path).read().split()
    assert len(lines) == 2 * 5
    rt = vs.Runtime(vs.vs_config_default(lam=2, slots_per_gpu=4))
    types = rt.vs_register_builtins(vs.VS_F32, MASK2)
    rt.vs_table_load(path)
    _, A, B, T = _dev_matmul(rt, 1024, 256, 7, MASK2, types)
    rt.vs_wait_all()
    log = rt.vs_decision_log()
    assert all(r[6] == 1 for r in log)                      # no learning run
    g = rt.vs_group_stats()[0]
    assert g["first_reliable"] == 1
    fastest = int(np.argmin(g0["mean_ns"]))
    assert log[0][1] == fastest
    assert oracle.relF(vsgen.from_tiles(T[2].cpu().numpy()), oracle.matmul(A, B)) <= 1e-5
    rt.close()


def test_next3_range_groups_and_ewma_mixed_sizes(gpu):
    """NEXT-3 (L984-997, fn. 3): tiles of 256 and 320 (DataSetSizes 786432 and 1228800, ratio
    1.5625) share one group under a 600 per-mille band: lambda runs per version in total, not per
    size; the recency-weighted mean is what the group reports."""
    rt = vs.Runtime(vs.vs_config_default(lam=2, slots_per_gpu=4, group_ratio_permille=600, ewma_weight=256))
    types, A1, B1, T1 = _dev_matmul(rt, 1024, 256, 11, MASK2)
    _, A2, B2, T2 = _dev_matmul(rt, 1280, 320, 12, MASK2, types)
    rt.vs_wait_all()
    (g,) = rt.vs_group_stats()
    assert g["bytes"] == 3 * 256 * 256 * 4 and sum(g["n"]) == 64 + 64
    assert g["reliable"] and g["first_reliable"] == 2 * 2 + 1
    assert all(m > 0 for m in g["mean_ns"])
    assert oracle.relF(vsgen.from_tiles(T1[2].cpu().numpy()), oracle.matmul(A1, B1)) <= 1e-5
    assert oracle.relF(vsgen.from_tiles(T2[2].cpu().numpy()), oracle.matmul(A2, B2)) <= 1e-5
    rt.close()


def test_next1_locality_with_host_transfers(gpu):
    """NEXT-1 (L978-984) with real host->device moves: every datum starts in host memory, the
    locality term (bytes not valid on the worker's GPU / 1 GB/s) enters every reliable EFT; on
    one GPU it shifts every worker equally, so decisions keep to the fastest version and every
    tile moves in once (Input Tx = 3 matrices) and home once (Output Tx = C)."""
    N, b = 1024, 256
    nt = N // b
    rt = vs.Runtime(vs.vs_config_default(lam=1, slots_per_gpu=4, locality_gbps=1))
    types, (A, B), (tA, tB, tC), (ia, ib, ic) = _host_matmul(rt, N, b, 71)
    rt.vs_app_matmul(types[vs.VS_T_MATMUL], nt, nt, nt, ia, ib, ic)
    rt.vs_wait_all()
    st = rt.vs_stats()
    assert st.input_tx_bytes == 3 * nt * nt * b * b * 4 and st.output_tx_bytes == nt * nt * b * b * 4
    assert oracle.relF(vsgen.from_tiles(tC.numpy()), oracle.matmul(A, B)) <= 1e-5
    rt.close()


def test_next1_locality_two_gpus_prefers_resident_data(gpu):
    """One process driving two GPUs (n_gpus = 2): with the locality term, a reliable task whose
    inputs live on GPU 1 runs there (skipped on a one-GPU box)."""
    torch = _torch()
    if torch.cuda.device_count() < 2:
        pytest.skip("needs 2 GPUs")
    b = 512
    rt = vs.Runtime(vs.vs_config_default(n_gpus=2, lam=1, slots_per_gpu=1, locality_gbps=1))
    types = rt.vs_register_builtins(vs.VS_F32, 1 << vs.VS_V_TC_3XTF32)
    # learn on GPU 0 data, then submit a task whose operands are all on GPU 1
    X0 = [torch.from_numpy(vsgen.uniform(80 + i, b, b)).to("cuda:0") for i in range(3)]
    ids0 = [rt.vs_data_register(x.data_ptr(), 0, b * b * 4) for x in X0]
    rt.vs_submit(types[vs.VS_T_MATMUL], ids0)
    rt.vs_wait_all()
    X1 = [torch.from_numpy(vsgen.uniform(90 + i, b, b)).to("cuda:1") for i in range(3)]
    ref = oracle.matmul(*[x.cpu().numpy() for x in X1])
    ids1 = [rt.vs_data_register(x.data_ptr(), 1, b * b * 4) for x in X1]
    rt.vs_submit(types[vs.VS_T_MATMUL], ids1)
    rt.vs_wait_all()
    assert rt.vs_decision_log()[-1][2] == 1              # worker 1 = GPU 1
    assert rt.vs_stats().device_tx_bytes == 0
    assert oracle.relF(X1[2].cpu().numpy(), ref) <= 1e-5
    rt.close()


# ------------------------------------------------------------------ a3: device dependence release
def test_device_release_matmul_and_cholesky(gpu):
    """cfg1 matmul + cfg2 Cholesky in one batch, bench launch configuration with the device
    tracker: every non-root task is made ready by its last predecessor's last CTA on the GPU
    (in-degree counters + CSR successors in device memory, ready ring in host memory)."""
    import bench
    torch = _torch()
    rt = vs.Runtime(bench.bench_config(vs, device_release=1))
    types = rt.vs_register_builtins(vs.VS_F32, bench.F32_VERSIONS_MASK)
    N, b = 1024, 256
    nt = N // b
    A, B = vsgen.uniform(1, N, N), vsgen.uniform(1001, N, N)
    T = [torch.from_numpy(vsgen.to_tiles(x, b)).cuda() for x in (A, B, np.zeros((N, N), np.float32))]
    ids = [[rt.vs_data_register(X[i, j].data_ptr(), 0, b * b * 4) for i in range(nt) for j in range(nt)] for X in T]
    rt.vs_app_matmul(types[vs.VS_T_MATMUL], nt, nt, nt, *ids)
    Nc, bc = 4096, 512
    ntc = Nc // bc
    S = vsgen.spd(2, Nc)
    TS = torch.from_numpy(vsgen.to_tiles(S, bc)).cuda()
    cids = {i * ntc + j: rt.vs_data_register(TS[i, j].data_ptr(), 0, bc * bc * 4) for i in range(ntc) for j in range(i + 1)}
    rt.vs_app_cholesky(types, ntc, cids)
    rt.vs_wait_all()
    torch.cuda.synchronize()
    st = rt.vs_stats()
    assert st.tasks_completed == 64 + 120
    assert st.device_released == (64 - 16) + (120 - 1)      # every task but the roots
    assert oracle.relF(vsgen.from_tiles(T[2].cpu().numpy()), oracle.matmul(A, B)) <= 1e-5
    L = np.tril(vsgen.from_tiles(TS.cpu().numpy()))
    Lref, info = oracle.cholesky(S)
    lo, slo = np.tril_indices(Nc), np.tril_indices(Nc, -1)
    assert info == 0
    assert oracle.relF(L[lo], Lref[lo]) <= 1e-5 and oracle.relF(L[slo], Lref[slo]) <= 1e-5
    # a second batch on the same runtime (new epoch): same results, same count
    T[2].zero_()
    rt.vs_data_invalidate_n(ids[2])
    rt.vs_app_matmul(types[vs.VS_T_MATMUL], nt, nt, nt, *ids)
    rt.vs_wait_all()
    assert rt.vs_stats().device_released == st.device_released + 48
    assert oracle.relF(vsgen.from_tiles(T[2].cpu().numpy()), oracle.matmul(A, B)) <= 1e-5
    rt.close()


def test_dev_alloc_hooks_use_the_callers_allocator(gpu):
    """vs_config.dev_alloc / dev_free (§8(b)): replicas and operand forms come from the caller's
    allocator — here torch's caching allocator — and are returned at vs_destroy."""
    torch = _torch()
    calls = {"alloc": 0, "free": 0, "bytes": 0}
    live = {}

    def alloc(dev, nbytes, user):
        calls["alloc"] += 1
        calls["bytes"] += nbytes
        p = torch.cuda.caching_allocator_alloc(nbytes, device=dev)
        live[p] = nbytes
        return p

    def free(dev, ptr, user):
        calls["free"] += 1
        torch.cuda.caching_allocator_delete(ptr)
        live.pop(ptr)

    fa, ff = vs.VS_DEV_ALLOC_FN(alloc), vs.VS_DEV_FREE_FN(free)
    rt = vs.Runtime(vs.vs_config_default(lam=1, slots_per_gpu=2, dev_alloc=fa, dev_free=ff))
    N, b = 512, 128
    nt = N // b
    types = rt.vs_register_builtins(vs.VS_F32, (1 << vs.VS_V_TC_3XTF32) | (1 << vs.VS_V_TC_3XF16))
    A, B = vsgen.uniform(3, N, N), vsgen.uniform(1003, N, N)
    T = [torch.from_numpy(vsgen.to_tiles(x, b)).pin_memory() for x in (A, B, np.zeros((N, N), np.float32))]
    ids = [[rt.vs_data_register(X[i, j].data_ptr(), -1, b * b * 4) for i in range(nt) for j in range(nt)] for X in T]
    rt.vs_app_matmul(types[vs.VS_T_MATMUL], nt, nt, nt, *ids)
    rt.vs_wait_all()
    assert calls["alloc"] >= 1 and calls["bytes"] >= 48 * b * b * 4      # host-homed tiles got device replicas
    assert oracle.relF(vsgen.from_tiles(T[2].numpy()), oracle.matmul(A, B)) <= 1e-5
    rt.close()
    assert calls["free"] == calls["alloc"] and not live

"""C ABI on CPU: symbol exports, and the C++ scheduler/DAG (VS_EXEC_SIM) against the
independent Python reference model (O3) — decision logs must be identical (R22, P8)."""
import os
import re

import pytest

import paper_conf_ipps_planasbal13_b200 as vs
from oracle.sched_model import SchedModel, submit_cholesky, submit_matmul

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
ALL = 0xFFFF


def test_library_exports_every_header_symbol():
    L = vs.lib()
    hdr = open(os.path.join(ROOT, "include", "vsched.h")).read()
    names = set(re.findall(r"^(?:int|void|uint64_t|int64_t|const char \*)\s*(vs_[a-z_0-9]+)\(", hdr, re.M))
    assert len(names) >= 25
    for n in sorted(names):
        assert hasattr(L, n), n
    assert set(vs.EXPORTED) == names
    assert "sm_100a" in vs.vs_build_info()


def _sim(n_gpus=1, slots=4, lam=3, learning=vs.VS_LEARN_HOLD, **kw):
    return vs.Runtime(vs.vs_config_default(exec=vs.VS_EXEC_SIM, n_gpus=n_gpus, slots_per_gpu=slots, lam=lam,
                                           learning=learning, **kw))


def _fake_ptr(i, nbytes):
    return 0x10000000 + i * ((nbytes + 4095) // 4096 * 4096)


def _pair_matmul(nt, b, lam, slots, durations, n_gpus=1):
    """Build the same matmul workload in the C++ runtime and in the Python model."""
    rt = _sim(n_gpus, slots, lam)
    t = rt.vs_type_create("MATMUL", [vs.VS_IN, vs.VS_IN, vs.VS_INOUT])
    for v in range(len(durations)):
        rt.vs_version_add(t, "v%d" % v, ALL)
    nbytes = b * b * 4
    ids = [rt.vs_data_register(_fake_ptr(i, nbytes), 0, nbytes) for i in range(3 * nt * nt)]
    A, B, C = ids[:nt * nt], ids[nt * nt:2 * nt * nt], ids[2 * nt * nt:]
    rt.vs_app_matmul(t, nt, nt, nt, A, B, C)
    for v, d in enumerate(durations):
        rt.vs_replay_set(t, 3 * nbytes, v, d)
    m = SchedModel(n_gpus, slots, lam)
    mt = m.add_type("MATMUL", [("v%d" % v, ALL) for v in range(len(durations))])
    mids = [m.add_data(nbytes) for _ in range(3 * nt * nt)]
    submit_matmul(m, mt, nt, nt, nt, mids[:nt * nt], mids[nt * nt:2 * nt * nt], mids[2 * nt * nt:])
    return rt, m


@pytest.mark.parametrize("lam,slots", [(1, 1), (3, 4), (5, 2)])
def test_matmul_sim_matches_reference_model(lam, slots):
    durs = [7000, 3000]
    rt, m = _pair_matmul(4, 256, lam, slots, durs)
    rt.vs_wait_all()
    ref = m.simulate(lambda ty, nb, v: durs[v])
    got = rt.vs_decision_log()
    assert [r[:4] for r in got] == [r[:4] for r in ref]
    assert [(r[4], r[5]) for r in got] == [(r[4], r[5]) for r in ref]
    assert rt.vs_decision_log_hash() == SchedModel.log_hash(ref)
    st = rt.vs_stats()
    assert st.tasks_completed == 64 and st.decisions == 64
    g = rt.vs_group_stats()[0]
    assert g["bytes"] == 786432 and g["first_reliable"] == 2 * lam + 1
    assert g["n"] == [sum(1 for r in got if r[1] == v) for v in range(2)]


def _pair_cholesky(nt, b, lam, slots, nv, dur, n_gpus=1):
    rt = _sim(n_gpus, slots, lam)
    names = ("POTRF", "TRSM", "SYRK", "GEMM_NT")
    modes = ([vs.VS_INOUT], [vs.VS_IN, vs.VS_INOUT], [vs.VS_IN, vs.VS_INOUT], [vs.VS_IN, vs.VS_IN, vs.VS_INOUT])
    tys = []
    for n, md in zip(names, modes):
        t = rt.vs_type_create(n, md)
        for v in range(nv):
            rt.vs_version_add(t, "v%d" % v, ALL)
        tys.append(t)
    nbytes = b * b * 4
    A = {}
    k = 0
    for i in range(nt):
        for j in range(i + 1):
            A[i * nt + j] = rt.vs_data_register(_fake_ptr(k, nbytes), 0, nbytes)
            k += 1
    # vs_app_cholesky takes the built-in type order [MATMUL, POTRF, TRSM, SYRK, GEMM_NT]
    rt.vs_app_cholesky([-1, tys[0], tys[1], tys[2], tys[3]], nt, A)
    sizes = {0: nbytes, 1: 2 * nbytes, 2: 2 * nbytes, 3: 3 * nbytes}
    for ti, t in enumerate(tys):
        for v in range(nv):
            rt.vs_replay_set(t, sizes[ti], v, dur(ti, sizes[ti], v))
    m = SchedModel(n_gpus, slots, lam)
    mt = tuple(m.add_type(n, [("v%d" % v, ALL) for v in range(nv)]) for n in names)
    mA = {}
    for i in range(nt):
        for j in range(i + 1):
            mA[i * nt + j] = m.add_data(nbytes)
    submit_cholesky(m, mt, nt, mA)
    return rt, m


@pytest.mark.parametrize("nt,lam,slots,n_gpus", [(8, 3, 4, 1), (6, 1, 1, 1), (8, 2, 2, 4), (12, 3, 4, 2)])
def test_cholesky_sim_matches_reference_model(nt, lam, slots, n_gpus):
    dur = lambda ti, nb, v: [500, 900, 700][v] * (ti + 1) + 13 * v + ti   # noqa: E731
    rt, m = _pair_cholesky(nt, 512, lam, slots, 3, dur, n_gpus)
    rt.vs_wait_all()
    ref = m.simulate(dur)
    got = rt.vs_decision_log()
    assert len(got) == len(ref) == nt * (nt + 1) * (nt + 2) // 6
    assert [r[:4] for r in got] == [r[:4] for r in ref]
    assert rt.vs_decision_log_hash() == SchedModel.log_hash(ref)


def test_replay_bit_exact_twice():
    dur = lambda ti, nb, v: [500, 900, 700][v] + 7 * ti   # noqa: E731
    h = []
    for _ in range(2):
        rt, _m = _pair_cholesky(8, 512, 3, 4, 3, dur)
        rt.vs_wait_all()
        h.append(rt.vs_decision_log_hash())
    assert h[0] == h[1]


def test_cfg2_potrf_never_reliable_through_abi():
    dur = lambda ti, nb, v: [500, 900, 700][v] * (ti + 1)   # noqa: E731
    rt, _ = _pair_cholesky(8, 512, 3, 4, 3, dur)
    rt.vs_wait_all()
    gs = {g["type_name"]: g for g in rt.vs_group_stats()}
    assert not gs["POTRF"]["reliable"] and sum(gs["POTRF"]["n"]) == 8
    assert gs["GEMM_NT"]["reliable"] and gs["GEMM_NT"]["first_reliable"] == 10


def test_table_i_and_new_group(tmp_path):
    MB = 1 << 20
    p = tmp_path / "table.txt"
    p.write_text("task1 %d task1-v1 30000000 200\ntask1 %d task1-v2 18000000 350\ntask1 %d task1-v3 25000000 230\n"
                 "task1 %d task1-v1 45000000 80\ntask1 %d task1-v2 25000000 300\ntask1 %d task1-v3 40000000 120\n"
                 "task2 %d task2-v1 15000000 40\ntask2 %d task2-v2 20000000 3\n"
                 % (2 * MB, 2 * MB, 2 * MB, 3 * MB, 3 * MB, 3 * MB, 5 * MB, 5 * MB))
    for lam, expect_v2 in ((3, 0), (4, 1)):
        rt = _sim(2, 1, lam)
        t1 = rt.vs_type_create("task1", [vs.VS_INOUT])
        for v in ("task1-v1", "task1-v2", "task1-v3"):
            rt.vs_version_add(t1, v, ALL)
        t2 = rt.vs_type_create("task2", [vs.VS_INOUT])
        for v in ("task2-v1", "task2-v2"):
            rt.vs_version_add(t2, v, ALL)
        rt.vs_table_load(str(p))
        d2 = rt.vs_data_register(_fake_ptr(0, 2 * MB), 0, 2 * MB)
        d3 = rt.vs_data_register(_fake_ptr(1, 4 * MB), 0, 3 * MB)
        d5 = rt.vs_data_register(_fake_ptr(3, 6 * MB), 0, 5 * MB)
        d4 = rt.vs_data_register(_fake_ptr(5, 6 * MB), 0, 4 * MB)
        for t, d in ((t1, d2), (t1, d3), (t2, d5), (t1, d4)):
            rt.vs_submit(t, [d])
        for t, nb, nv in ((t1, 2 * MB, 3), (t1, 3 * MB, 3), (t2, 5 * MB, 2), (t1, 4 * MB, 3)):
            for v in range(nv):
                rt.vs_replay_set(t, nb, v, 1000)
        rt.vs_wait_all()
        log = rt.vs_decision_log()
        assert log[0][1] == 1 and log[0][6] == 1          # task1 @2MB -> v2, reliable
        assert log[1][1] == 1 and log[1][6] == 1          # task1 @3MB -> v2
        assert log[2][1] == expect_v2                      # task2 @5MB: v1 (lam 3) / v2 learning (lam 4)
        assert log[2][6] == (1 if lam == 3 else 0)
        assert log[3][6] == 0 and log[3][1] == 0           # new size 4MB -> learning, RR from v1
        out = tmp_path / ("dump%d.txt" % lam)
        rt.vs_table_dump(str(out))
        assert "task1 %d task1-v1 45000000 80" % (3 * MB) in out.read_text()   # untouched group entry


def test_weighted_bottom_level_matches_model(tmp_path):
    """R29 / R38 through the C ABI: learned means (warm-start table) weight the bottom levels;
    the same graph as tests/test_sched_fixtures.py::test_weighted_bottom_level_uses_learned_means,
    C++ log = model log."""
    p = tmp_path / "w.txt"
    p.write_text("A 8 v 100 1\nB 8 v 10 1\n")
    rt = _sim(1, 1, 1, priority=2, queue_depth=1)
    ta = rt.vs_type_create("A", [vs.VS_INOUT])
    rt.vs_version_add(ta, "v", ALL)
    tb = rt.vs_type_create("B", [vs.VS_INOUT])
    rt.vs_version_add(tb, "v", ALL)
    rt.vs_table_load(str(p))
    a = rt.vs_data_register(_fake_ptr(0, 8), 0, 8)
    b = rt.vs_data_register(_fake_ptr(1, 8), 0, 8)
    for t, d, n in ((ta, a, 2), (tb, b, 3)):
        for _ in range(n):
            rt.vs_submit(t, [d])
    rt.vs_replay_set(ta, 8, 0, 100)
    rt.vs_replay_set(tb, 8, 0, 10)
    rt.vs_wait_all()
    got = rt.vs_decision_log()
    m = SchedModel(1, 1, 1, priority=2, qdepth=1)
    ma, mb = m.add_type("A", [("v", ALL)]), m.add_type("B", [("v", ALL)])
    da, db = m.add_data(8), m.add_data(8)
    for t, d, n in ((ma, da, 2), (mb, db, 3)):
        for _ in range(n):
            m.submit(t, [(d, "inout")])
    m.load_table([(ma, 8, [(100, 1)]), (mb, 8, [(10, 1)])])
    ref = m.simulate(lambda ty, nb, v: 100 if ty == ma else 10)
    assert [r[:6] for r in got] == [r[:6] for r in ref]
    assert [(r[0], r[3]) for r in got] == [(0, 0), (1, 100), (2, 200), (3, 210), (4, 220)]


def test_fig5_earliest_executor_masks():
    # Fig 5: version "fast" runs only on gpu 3 (worker 3), "slow" only on gpu 2.
    rt = _sim(4, 1, 1)
    t = rt.vs_type_create("task", [vs.VS_INOUT])
    rt.vs_version_add(t, "fast", 1 << 3)
    rt.vs_version_add(t, "slow", 1 << 2)
    ds = [rt.vs_data_register(_fake_ptr(i, 64), 0, 64) for i in range(8)]
    for d in ds:
        rt.vs_submit(t, [d])
    rt.vs_replay_set(t, 64, 0, 10_000)
    rt.vs_replay_set(t, 64, 1, 40_000)
    rt.vs_wait_all()
    log = rt.vs_decision_log()
    m = SchedModel(4, 1, 1)
    mt = m.add_type("task", [("fast", 1 << 3), ("slow", 1 << 2)])
    for _ in range(8):
        m.submit(mt, [(m.add_data(64), "inout")])
    ref = m.simulate(lambda ty, nb, v: [10_000, 40_000][v])
    assert [r[:4] for r in log] == [r[:4] for r in ref]
    # after learning, tasks pile on worker 3 until its backlog exceeds 40 us, then worker 2 helps
    reliable = [r for r in log if r[6] == 1]
    assert any(r[2] == 2 for r in reliable) and any(r[2] == 3 for r in reliable)


def test_overlap_and_errors():
    rt = _sim()
    a = rt.vs_data_register(0x1000, 0, 4096)
    assert rt.vs_data_register(0x1000, 0, 4096) == a
    with pytest.raises(vs.VSError) as e:
        rt.vs_data_register(0x1800, 0, 4096)
    assert e.value.code == vs.VS_E_OVERLAP
    t = rt.vs_type_create("x", [vs.VS_INOUT])
    with pytest.raises(vs.VSError):
        rt.vs_submit(t, [a])        # no version
    rt.vs_version_add(t, "v", ALL)
    with pytest.raises(vs.VSError):
        rt.vs_submit(t, [a, a])     # wrong arity
    rt.vs_submit(t, [a])
    with pytest.raises(vs.VSError) as e:
        rt.vs_wait_all()            # no replay duration
    assert e.value.code == vs.VS_E_STATE


def test_rr_learning_variant_keeps_cycling():
    rt = _sim(1, 4, 2, learning=vs.VS_LEARN_RR)
    t = rt.vs_type_create("x", [vs.VS_INOUT])
    rt.vs_version_add(t, "a", ALL)
    rt.vs_version_add(t, "b", ALL)
    ds = [rt.vs_data_register(_fake_ptr(i, 64), 0, 64) for i in range(12)]
    for d in ds:
        rt.vs_submit(t, [d])
    rt.vs_replay_set(t, 64, 0, 100)
    rt.vs_replay_set(t, 64, 1, 50)
    rt.vs_wait_all()
    log = rt.vs_decision_log()
    # all 12 are ready at t=0, no time has been recorded yet: paper-literal RR alternates
    assert [r[1] for r in log] == [0, 1] * 6


@pytest.mark.parametrize("ratio,ewma", [(0, 0), (300, 0), (300, 256), (0, 512)])
def test_next3_range_groups_and_ewma_match_model(ratio, ewma):
    # NEXT-3: range groups (L984-993) + recency-weighted mean (fn. 3, L458-460), C++ vs O3.
    sizes = [128, 144, 160, 192, 256, 320]
    rt = vs.Runtime(vs.vs_config_default(exec=vs.VS_EXEC_SIM, n_gpus=1, slots_per_gpu=2, lam=2,
                                         group_ratio_permille=ratio, ewma_weight=ewma))
    t = rt.vs_type_create("MATMUL", [vs.VS_IN, vs.VS_IN, vs.VS_INOUT])
    rt.vs_version_add(t, "a", ALL)
    rt.vs_version_add(t, "b", ALL)
    m = SchedModel(1, 2, 2, group_ratio=ratio, ewma=ewma)
    mt = m.add_type("MATMUL", [("a", ALL), ("b", ALL)])
    k = 0
    dur = lambda ty, nb, v: (nb // 1000) * (3 if v == 0 else 2) + 100 * v   # noqa: E731
    for rep in range(6):
        for b in sizes:
            nb = b * b * 4
            ids = [rt.vs_data_register(0x10000000 + k + i * nb, 0, nb) for i in range(3)]
            mids = [m.add_data(nb) for _ in range(3)]
            k += 3 * nb
            rt.vs_submit(t, ids)
            m.submit(mt, [(mids[0], "in"), (mids[1], "in"), (mids[2], "inout")])
    for b in sizes:
        for v in range(2):
            rt.vs_replay_set(t, 3 * b * b * 4, v, dur(t, 3 * b * b * 4, v))
    rt.vs_wait_all()
    ref = m.simulate(dur)
    got = rt.vs_decision_log()
    assert [r[:4] for r in got] == [r[:4] for r in ref]
    ngroups = len(rt.vs_group_stats())
    assert ngroups == (len(sizes) if ratio == 0 else len({id(g) for g in m.groups.values()}))
    if ratio:
        assert ngroups < len(sizes)


def _locality_run(gbps):
    # NEXT-1 (L978-984): EFT + bytes not on the worker's GPU / bandwidth; 2 GPUs x 2 slots.
    nt, b = 4, 256
    nbytes = b * b * 4
    rt = vs.Runtime(vs.vs_config_default(exec=vs.VS_EXEC_SIM, n_gpus=2, slots_per_gpu=2, lam=1,
                                         locality_gbps=gbps))
    t = rt.vs_type_create("MATMUL", [vs.VS_IN, vs.VS_IN, vs.VS_INOUT])
    rt.vs_version_add(t, "a", ALL)
    rt.vs_version_add(t, "b", ALL)
    ids = [rt.vs_data_register(_fake_ptr(i, nbytes), i % 2, nbytes) for i in range(3 * nt * nt)]
    rt.vs_app_matmul(t, nt, nt, nt, ids[:16], ids[16:32], ids[32:])
    rt.vs_replay_set(t, 3 * nbytes, 0, 30000)
    rt.vs_replay_set(t, 3 * nbytes, 1, 20000)
    m = SchedModel(2, 2, 1, locality_gbps=gbps)
    mt = m.add_type("MATMUL", [("a", ALL), ("b", ALL)])
    mids = [m.add_data(nbytes, home=i % 2) for i in range(3 * nt * nt)]
    submit_matmul(m, mt, nt, nt, nt, mids[:16], mids[16:32], mids[32:])
    rt.vs_wait_all()
    ref = m.simulate(lambda ty, nb, v: [30000, 20000][v])
    got = rt.vs_decision_log()
    assert [r[:4] for r in got] == [r[:4] for r in ref]
    # chain migrations: consecutive tasks of one C tile on different GPUs
    gpu_of = {r[0]: r[2] // 2 for r in got}
    return sum(gpu_of[c * nt + k] != gpu_of[c * nt + k - 1] for c in range(nt * nt) for k in range(1, nt))


@pytest.mark.parametrize("gbps", [0, 50])
def test_next1_locality_eft_matches_model(gbps):
    _locality_run(gbps)


def test_next1_locality_reduces_migrations():
    assert _locality_run(50) <= _locality_run(0)


# ---------------------------------------------------------------- NEXT-4 (R29)
def _mixed(nt_mm, nt_ch, lam, slots, dur_us, n_gpus=1, model=True, **kw):
    """Fig 1 matmul and the tiled Cholesky submitted to ONE runtime (the bench workload's
    shape), replayed from a timing table; returns (C++ log, Python model log or None)."""
    rt = _sim(n_gpus, slots, lam, **kw)
    names = ("MATMUL", "POTRF", "TRSM", "SYRK", "GEMM_NT")
    modes = ([vs.VS_IN, vs.VS_IN, vs.VS_INOUT], [vs.VS_INOUT], [vs.VS_IN, vs.VS_INOUT], [vs.VS_IN, vs.VS_INOUT],
             [vs.VS_IN, vs.VS_IN, vs.VS_INOUT])
    nbytes = 1024 * 1024 * 4
    sizes = (3 * nbytes, nbytes, 2 * nbytes, 2 * nbytes, 3 * nbytes)
    tys = []
    for ti, (n, md) in enumerate(zip(names, modes)):
        t = rt.vs_type_create(n, md)
        for v in range(2):
            rt.vs_version_add(t, "v%d" % v, ALL)
            rt.vs_replay_set(t, sizes[ti], v, dur_us[ti] * 1000 * (3 if v == 0 else 1))
        tys.append(t)
    k = [0]

    def reg():
        k[0] += 1
        return rt.vs_data_register(_fake_ptr(k[0], nbytes), 0, nbytes)
    mm = [reg() for _ in range(3 * nt_mm * nt_mm)]
    q = nt_mm * nt_mm
    rt.vs_app_matmul(tys[0], nt_mm, nt_mm, nt_mm, mm[:q], mm[q:2 * q], mm[2 * q:])
    A = {i * nt_ch + j: reg() for i in range(nt_ch) for j in range(i + 1)}
    rt.vs_app_cholesky(tys, nt_ch, A)
    rt.vs_wait_all()
    got = rt.vs_decision_log()
    rt.close()
    if not model:
        return got, None
    m = SchedModel(n_gpus, slots, lam, priority=kw.get("priority", 0), qdepth=kw.get("queue_depth", 0))
    mt = [m.add_type(n, [("v0", ALL), ("v1", ALL)]) for n in names]
    mm_ = [m.add_data(nbytes) for _ in range(3 * q)]
    submit_matmul(m, mt[0], nt_mm, nt_mm, nt_mm, mm_[:q], mm_[q:2 * q], mm_[2 * q:])
    mA = {i * nt_ch + j: m.add_data(nbytes) for i in range(nt_ch) for j in range(i + 1)}
    submit_cholesky(m, tuple(mt[1:]), nt_ch, mA)
    idx = {t: i for i, t in enumerate(mt)}
    ref = m.simulate(lambda ty, nb, v: dur_us[idx[ty]] * 1000 * (3 if v == 0 else 1))
    return got, ref


BENCH_US = (68, 1500, 330, 52, 50)   # measured per-task us at b=1024 (MATMUL POTRF TRSM SYRK GEMM_NT)


@pytest.mark.parametrize("priority,qdepth,slots", [(0, 0, 4), (0, 2, 4), (2, 0, 3), (2, 1, 2), (2, 2, 6),
                                                   (2, 3, 4)])
def test_next4_priority_and_queue_depth_match_model(priority, qdepth, slots):
    got, ref = _mixed(4, 6, 2, slots, BENCH_US, priority=priority, queue_depth=qdepth)
    assert len(got) == len(ref) == 64 + 56
    assert [r[:6] for r in got] == [r[:6] for r in ref]


def test_next4_bottom_level_with_queue_depth_shortens_the_mixed_makespan():
    # the bench workload's shape at 1/4 scale in each dimension; paper rule vs NEXT-4
    span = {}
    for key, kw in (("paper", {}), ("next4", dict(priority=2, queue_depth=2))):
        got, _ = _mixed(8, 16, 3, 6, BENCH_US, model=False, **kw)
        span[key] = max(r[5] for r in got)
    assert span["next4"] < span["paper"]


def test_fixed_policy_version_checked_per_type():
    """VS_POLICY_FIXED indexes each type's own version list: an index that a type does not have
    is rejected at submission instead of reading past its versions."""
    rt = _sim(policy=vs.VS_POLICY_FIXED, fixed_version=2)
    t3 = rt.vs_type_create("T3", [vs.VS_INOUT])
    t2 = rt.vs_type_create("T2", [vs.VS_INOUT])
    for v in range(3):
        rt.vs_version_add(t3, "v%d" % v, ALL)
    for v in range(2):
        rt.vs_version_add(t2, "v%d" % v, ALL)
    d = rt.vs_data_register(_fake_ptr(0, 4096), 0, 4096)
    rt.vs_replay_set(t3, 4096, 2, 1000)
    rt.vs_submit(t3, [d])
    with pytest.raises(vs.VSError) as e:
        rt.vs_submit(t2, [d])
    assert e.value.code == vs.VS_E_INVAL and "fixed version 2" in rt.vs_last_error()
    rt.vs_wait_all()
    assert [r[1] for r in rt.vs_decision_log()] == [2]


def test_version_mask_must_name_a_configured_gpu():
    rt = _sim(n_gpus=2)
    t = rt.vs_type_create("T", [vs.VS_INOUT])
    with pytest.raises(vs.VSError) as e:
        rt.vs_version_add(t, "nowhere", 1 << 2)   # only gpus 0 and 1 exist
    assert e.value.code == vs.VS_E_INVAL
    with pytest.raises(vs.VSError):
        rt.vs_submit(t, [rt.vs_data_register(_fake_ptr(0, 4096), 0, 4096)])   # no version at all
    rt.vs_version_add(t, "gpu1", 1 << 1)
    assert rt.vs_submit(t, [rt.vs_data_register(_fake_ptr(0, 4096), 0, 4096)]) == 0


def test_trace_path_jsonl_matches_decision_log(tmp_path):
    """vs_config.trace_path (§8(b)): each wait appends the decisions completed since the last one
    as JSON lines, identical to vs_decision_log."""
    import json
    path = str(tmp_path / "trace.jsonl")
    rt = _sim(slots=2, lam=1, trace_path=path)
    t = rt.vs_type_create("MATMUL", [vs.VS_IN, vs.VS_IN, vs.VS_INOUT])
    for v in range(2):
        rt.vs_version_add(t, "v%d" % v, ALL)
    nb = 4096
    ids = [rt.vs_data_register(_fake_ptr(i, nb), 0, nb) for i in range(12)]
    rt.vs_app_matmul(t, 2, 2, 2, ids[:4], ids[4:8], ids[8:])
    rt.vs_replay_set(t, 3 * nb, 0, 3000)
    rt.vs_replay_set(t, 3 * nb, 1, 1000)
    rt.vs_wait_all()
    rt.vs_app_matmul(t, 2, 2, 2, ids[:4], ids[4:8], ids[8:])
    rt.vs_wait_all_noflush()
    lines = [json.loads(x) for x in open(path)]
    log = rt.vs_decision_log()
    assert len(lines) == len(log) == 16
    for rec, r in zip(lines, log):
        assert (rec["task"], rec["worker"], rec["phase"], rec["t_decide_ns"], rec["t_start_ns"], rec["t_end_ns"]) == \
            (r[0], r[2], r[6], r[3], r[4], r[5])
        assert rec["type"] == "MATMUL" and rec["version"] == "v%d" % r[1]
    rt.vs_decision_log_clear()
    assert len(open(path).read().splitlines()) == 16    # nothing written twice

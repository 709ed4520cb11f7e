"""Pins for the scheduler reference model (O3): the paper's own fixtures (Table I,
Fig 5), the lambda invariants stated in Sec IV.B, and brute-force DAG checks (P5)."""
import itertools

import pytest

from oracle.sched_model import SchedModel, submit_cholesky, submit_matmul

ALL = 0xFF


def _matmul_model(nt, lam=3, n_gpus=1, slots=4, versions=(("simt", ALL), ("tc", ALL)), b=256):
    m = SchedModel(n_gpus, slots, lam)
    t = m.add_type("MATMUL", versions)
    A = [m.add_data(b * b * 4) for _ in range(nt * nt)]
    B = [m.add_data(b * b * 4) for _ in range(nt * nt)]
    C = [m.add_data(b * b * 4) for _ in range(nt * nt)]
    submit_matmul(m, t, nt, nt, nt, A, B, C)
    return m, t


def _chol_model(nt, lam=3, n_gpus=1, slots=4, nv=3, b=512):
    m = SchedModel(n_gpus, slots, lam)
    vers = [("v%d" % i, ALL) for i in range(nv)]
    types = tuple(m.add_type(n, vers) for n in ("POTRF", "TRSM", "SYRK", "GEMM_NT"))
    A = {}
    for i in range(nt):
        for j in range(i + 1):
            A[i * nt + j] = m.add_data(b * b * 4)
    submit_cholesky(m, types, nt, A)
    return m, types


@pytest.mark.parametrize("nt,edges", [(4, 48), (16, 3840)])
def test_matmul_edge_counts(nt, edges):
    m, _ = _matmul_model(nt)
    assert len(m.tasks) == nt ** 3
    assert m.build_edges() == edges


@pytest.mark.parametrize("nt,tasks,edges", [(8, 120, 252), (16, 816, 2040), (32, 5984, 16368)])
def test_cholesky_counts(nt, tasks, edges):
    m, _ = _chol_model(nt)
    assert len(m.tasks) == tasks
    assert m.build_edges() == edges


@pytest.mark.parametrize("nt", [2, 3, 4, 5])
def test_dag_brute_force(nt):
    # P5: every pair touching a common datum with >= 1 writer is ordered (transitively, in
    # submission order), and every direct edge joins such a conflicting pair.
    m, _ = _chol_model(nt)
    m.build_edges()
    T = len(m.tasks)
    reach = [set() for _ in range(T)]
    for t in range(T):
        for p in m.preds[t]:
            assert p < t
            reach[t] |= reach[p] | {p}

    def conflict(a, b):
        da = {d: mo for d, mo in m.tasks[a]["args"]}
        db = {d: mo for d, mo in m.tasks[b]["args"]}
        return any(d in db and ("in" != da[d] or "in" != db[d]) for d in da)

    for a, b in itertools.combinations(range(T), 2):
        if conflict(a, b):
            assert a in reach[b], (a, b)
    for t in range(T):
        for p in m.preds[t]:
            assert conflict(p, t)


def test_dataset_size_footnote2():
    # fn. 2: each parameter counted once even if inout: matmul fp32 b=256 -> 786432 B.
    m, _ = _matmul_model(1, b=256)
    assert m.dataset_size(m.tasks[0]) == 786432
    m2, _ = _chol_model(3, b=512)
    sizes = sorted({(m2.types[t["type"]][0], m2.dataset_size(t)) for t in m2.tasks})
    assert sizes == [("GEMM_NT", 3 << 20), ("POTRF", 1 << 20), ("SYRK", 2 << 20), ("TRSM", 2 << 20)]


def _table_i_model(lam):
    m = SchedModel(2, 1, lam)
    t1 = m.add_type("task1", [("task1-v1", ALL), ("task1-v2", ALL), ("task1-v3", ALL)])
    t2 = m.add_type("task2", [("task2-v1", ALL), ("task2-v2", ALL)])
    MB = 1 << 20
    m.load_table([(t1, 2 * MB, [(30_000_000, 200), (18_000_000, 350), (25_000_000, 230)]),
                  (t1, 3 * MB, [(45_000_000, 80), (25_000_000, 300), (40_000_000, 120)]),
                  (t2, 5 * MB, [(15_000_000, 40), (20_000_000, 3)])])
    return m, t1, t2, MB


def _decide_one(m, ttype, nbytes):
    d = m.add_data(nbytes)
    t = m.submit(ttype, [(d, "inout")])
    m.queue = [[] for _ in range(m.W)]
    m.running = [None] * m.W
    return m.decide(t, 0)


def test_table_i_fixture():
    # Table I (L371-381): fastest = v2 @2MB, v2 @3MB, v1 @5MB.
    m, t1, t2, MB = _table_i_model(3)
    assert _decide_one(m, t1, 2 * MB)[0] == 1
    assert _decide_one(m, t1, 3 * MB)[0] == 1
    v, w, est, phase = _decide_one(m, t2, 5 * MB)
    assert (v, phase, est) == (0, 1, 15_000_000)
    # lambda = 4: task2-v2 has #Exec 3 < 4, still learning, must run v2 next.
    m, t1, t2, MB = _table_i_model(4)
    v, w, est, phase = _decide_one(m, t2, 5 * MB)
    assert (v, phase) == (1, 0)
    # A new data-set size opens a new group in learning (L484-489).
    v, w, est, phase = _decide_one(m, t1, 4 * MB)
    assert phase == 0 and v == 0


def test_fig5_earliest_executor():
    # Fig 5 / L453-475: the fastest executor (worker 3, 10 ms) has a 50 ms backlog;
    # idle worker 2 runs the slow version (40 ms) and finishes first -> worker 2.
    m = SchedModel(4, 1, 1)
    t = m.add_type("task", [("gpu", 1 << 3), ("smp", 1 << 2)])
    m.load_table([(t, 64, [(10_000_000, 5), (40_000_000, 5)])])
    d = m.add_data(64)
    x = m.submit(t, [(d, "inout")])
    m.queue = [[] for _ in range(4)]
    m.running = [None] * 4
    m.running[3] = (999, 0, 50_000_000)
    v, w, est, phase = m.decide(x, 0)
    assert (v, w, phase) == (1, 2, 1)
    m.running[3] = (999, 0, 20_000_000)      # backlog small: fastest executor wins
    v, w, est, phase = m.decide(x, 0)
    assert (v, w) == (0, 3)


def _dur_two_versions(ttype, nbytes, v):
    return [7000, 3000][v]


@pytest.mark.parametrize("lam", [1, 2, 3, 5])
def test_lambda_invariants_matmul(lam):
    # "each task version at least lambda times" (L438-440); with hold exactly lambda learning
    # runs per version and the first reliable decision is V*lambda+1; afterwards all
    # decisions pick the fastest mean on homogeneous workers (L675-680).
    m, _ = _matmul_model(4, lam=lam)
    log = m.simulate(_dur_two_versions)
    learning = [r for r in log if r[6] == 0]
    assert len(learning) == 2 * lam
    assert sorted(r[1] for r in learning) == [0] * lam + [1] * lam
    g = m.groups[m.group_order[0]]
    assert g["first_reliable"] == 2 * lam + 1
    assert all(r[1] == 1 for r in log if r[6] == 1)


def test_cfg2_potrf_stays_learning():
    # L496-501: potrf has 8 instances < 3 versions x lambda=3 -> never reliable.
    m, types = _chol_model(8, lam=3)
    log = m.simulate(lambda t, b, v: 1000 * (v + 1) + 10 * t)
    g = m.groups[(types[0], 512 * 512 * 4)]
    assert not g["reliable"]
    assert sum(g["n"]) == 8
    gg = m.groups[(types[3], 3 * 512 * 512 * 4)]
    assert gg["reliable"] and gg["first_reliable"] == 10


def test_replay_deterministic():
    m1, _ = _chol_model(6, lam=2)
    m2, _ = _chol_model(6, lam=2)
    dur = lambda t, b, v: 1000 + 37 * v + 5 * t     # noqa: E731
    h1 = SchedModel.log_hash(m1.simulate(dur))
    h2 = SchedModel.log_hash(m2.simulate(dur))
    assert h1 == h2

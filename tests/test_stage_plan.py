"""Transfer plan of a batch whose inputs are homed in host memory (vs_config.stage, DESIGN
reading R39; overlap of moves with computation): the order in which the runtime
copies the inputs to the GPU, from vs_transfer_plan on the SIM executor (the plan is the same
host computation the GPU executor runs at drive start).  Expected orders are worked by hand
from the rule in vsched.h (critical-path component first; then critical tasks, weighted slack,
fewest unplanned input bytes, the datum closest to its final version, weighted bottom level,
id), with every weight the unknown-weight default, so that equal weights reduce the weighted
levels to unit levels."""
import paper_conf_ipps_planasbal13_b200 as vs

NB = 256 * 256 * 4


def _rt():
    return vs.Runtime(vs.vs_config_default(exec=vs.VS_EXEC_SIM, slots_per_gpu=2, lam=1, priority=2,
                                           mode=vs.VS_MODE_READY))


def _reg(rt, names, dev=-1, base=0x10000000):
    return {n: rt.vs_data_register(base + i * NB, dev, NB) for i, n in enumerate(names)}


def _matmul(rt, types, d, nt=2):
    A = [d["A%d%d" % (i, k)] for i in range(nt) for k in range(nt)]
    B = [d["B%d%d" % (k, j)] for k in range(nt) for j in range(nt)]
    C = [d["C%d%d" % (i, j)] for i in range(nt) for j in range(nt)]
    rt.vs_app_matmul(types[vs.VS_T_MATMUL], nt, nt, nt, A, B, C)


def _cholesky(rt, types, d, nt=3):
    rt.vs_app_cholesky(types, nt, {i * nt + j: d["L%d%d" % (i, j)] for i in range(nt) for j in range(i + 1)})


MM = ["%s%d%d" % (m, i, j) for m in "ABC" for i in range(2) for j in range(2)]
CH = ["L%d%d" % (i, j) for i in range(3) for j in range(i + 1)]
# matmul 2x2x2: every C tile's chain (i,j,0) -> (i,j,1) is its own component (equal critical
# paths: taken in id order), so each C tile is finished before the next is opened; A00 B00 C00
# for (0,0,0), A01 B10 for (0,0,1), B01 C01 for (0,1,0), B11 for (0,1,1), A10 C10, A11, C11.
MM_ORDER = ["A00", "B00", "C00", "A01", "B10", "B01", "C01", "B11", "A10", "C10", "A11", "C11"]
# Cholesky 3x3 (task ids: potrf00 0, trsm10 1, trsm20 2, syrk11 3, gemm21 4, syrk22 5,
# potrf11 6, trsm21 7, syrk22' 8, potrf22 9; critical path 0-1-3-6-7-8-9, slack of trsm20 and
# gemm21 = 1, of syrk22 = 2): potrf00 (L00), trsm10 (L10), syrk11 (L11), potrf11, trsm20 (L20),
# gemm21 (L21), trsm21, syrk22 (L22) — the leading blocks first, as the chain needs them.
CH_ORDER = ["L00", "L10", "L11", "L20", "L21", "L22"]


def _plan(build):
    rt = _rt()
    types = rt.vs_register_builtins(vs.VS_F32, 1 << vs.VS_V_SIMT_F32)
    d = build(rt, types)
    inv = {v: k for k, v in d.items()}
    return [inv[x] for x in rt.vs_transfer_plan()]


def test_matmul_plan_finishes_each_output_tile_first():
    def build(rt, types):
        d = _reg(rt, MM)
        _matmul(rt, types, d)
        return d
    assert _plan(build) == MM_ORDER


def test_cholesky_plan_follows_the_critical_path():
    def build(rt, types):
        d = _reg(rt, CH)
        _cholesky(rt, types, d)
        return d
    assert _plan(build) == CH_ORDER


def test_longest_component_first():
    # the matmul is submitted first, but the Cholesky's critical path (7 tasks) is longer than
    # any of the matmul's chains (2 tasks): all of its inputs cross the link first
    def build(rt, types):
        d = _reg(rt, MM + CH)
        _matmul(rt, types, d)
        _cholesky(rt, types, d)
        return d
    assert _plan(build) == CH_ORDER + MM_ORDER


def test_only_host_data_read_at_batch_start():
    def build(rt, types):
        d = _reg(rt, MM)
        d.update(_reg(rt, ["X"], dev=0, base=0x80000000))          # device-homed: never in the plan
        t = rt.vs_type_create("FILL", [vs.VS_IN, vs.VS_OUT])
        rt.vs_version_add(t, "v", 0xFFFF)
        rt.vs_submit(t, [d["X"], d["A00"]])       # A00 written before any read: not an input
        _matmul(rt, types, d)
        return d
    got = _plan(build)
    assert "X" not in got and "A00" not in got
    assert sorted(got) == sorted(x for x in MM if x != "A00")


def test_device_resident_batch_has_no_plan():
    def build(rt, types):
        d = _reg(rt, MM, dev=0)
        _matmul(rt, types, d)
        return d
    assert _plan(build) == []


def test_plan_empty_after_the_batch_retired():
    rt = _rt()
    types = rt.vs_register_builtins(vs.VS_F32, 1 << vs.VS_V_SIMT_F32)
    d = _reg(rt, MM)
    _matmul(rt, types, d)
    rt.vs_replay_set(types[vs.VS_T_MATMUL], 3 * NB, 0, 1000)
    rt.vs_wait_all()
    assert rt.vs_transfer_plan() == []      # batch retired: nothing left to plan

"""Hand-worked fixtures for the scheduler reference model's option branches (O3).

Each fixture is a tiny graph whose expected decisions were derived BY HAND from the passage
the option follows (the derivation is written next to each expectation), and is asserted
against ``SchedModel`` alone — not against the C++ runtime (test_capi_sim.py then checks
C++ = model).  Each one is chosen so that a plausible misreading fails it:

* NEXT-3 range groups (future work L984-997): inclusive ratio band, first group in creation
  order (not the nearest), band measured against the group's creating size;
* NEXT-3 recency-weighted mean (footnote 3, L458-460): m += (x - m) * w / 1024 with the
  correction truncated toward zero, first sample taken as is;
* NEXT-1 locality-aware earliest executor (L978-984): EFT + bytes not valid on the worker's
  GPU / bandwidth (1 GB/s = 1 byte/ns, integer division), validity updated in decision order
  (reads replicate, writes own);
* NEXT-4 bottom-level priority + queue depth (R29), critical path first (R38);
* the paper-literal "rr" learning variant (R12) against the default hold policy.
"""
from oracle.sched_model import SchedModel

ALL = 0xFF


def _reset_queues(m):
    m.queue = [[] for _ in range(m.W)]
    m.running = [None] * m.W


# ----------------------------------------------------------------- NEXT-3 range groups
def test_range_groups_band_is_inclusive_first_created_wins():
    """ratio 100 per mille = sizes within a factor 1.1 of a group's creating size share it."""
    m = SchedModel(1, 1, 1, group_ratio=100)
    t = m.add_type("T", [("v", ALL)])

    def task(nbytes):
        return m.submit(t, [(m.add_data(nbytes), "inout")])

    g1000 = m.group_of(task(1000))
    assert m.group_of(task(1100)) is g1000          # 1100*1000 == 1000*1100: on the band edge, joins
    g1101 = m.group_of(task(1101))                  # 1101*1000 > 1000*1100: a new group
    assert g1101 is not g1000
    # 1080 is within the band of BOTH groups (1101*1000 <= 1080*1100) and nearer to 1101 (21 vs
    # 80 bytes); it joins the first group created, 1000
    assert m.group_of(task(1080)) is g1000
    # the band is measured from the creating size (1101), not from a member (1100): 1190 joins
    # 1101 (1190*1000 <= 1101*1100 = 1211100) and not 1000 (1190*1000 > 1000*1100)
    assert m.group_of(task(1190)) is g1101
    assert len({id(g) for g in m.groups.values()}) == 2
    assert m.group_order == [(t, 1000), (t, 1101)]


def test_range_groups_share_learning():
    """lambda = 1, two versions, one worker, four independent tasks of sizes 1000, 1080, 1000,
    1080 (one range group with ratio 100), durations d(size, v) = (100 if v == 0 else 50) +
    (size - 1000).  Hand derivation (hold policy, R12):
      t=0    t0 -> v0 (rr 0), t1 -> v1 (same group, rr 1); t2, t3 held (both versions assigned).
             t0 runs 0-100, t1 100-230 (50 + 80).
      t=100  record v0 = 100 (n = [1, 0], still learning).
      t=230  record v1 = 130 -> reliable, held t2, t3 released in FIFO order.
             t2: worker idle, v* = argmin mean = v0 (100 < 130): EFT 100 -> (t2, v0), runs 230-330.
             t3: busy = remaining estimate of t2 = 100 -> EFT 200 with v0 -> (t3, v0), 330-510.
    With exact groups the 1080 tasks would learn on their own (t1 -> v0 of a second group)."""
    def dur(ttype, nbytes, v):
        return (100 if v == 0 else 50) + (nbytes - 1000)

    def run(ratio):
        m = SchedModel(1, 1, 1, group_ratio=ratio)
        t = m.add_type("T", [("a", ALL), ("b", ALL)])
        for nb in (1000, 1080, 1000, 1080):
            m.submit(t, [(m.add_data(nb), "inout")])
        return m.simulate(dur)

    assert run(100) == [(0, 0, 0, 0, 0, 100, 0), (1, 1, 0, 0, 100, 230, 0),
                        (2, 0, 0, 230, 230, 330, 1), (3, 0, 0, 230, 330, 510, 1)]
    exact = run(0)
    assert [(r[0], r[1], r[6]) for r in exact[:2]] == [(0, 0, 0), (1, 0, 0)]   # 1080 opens its own group


# --------------------------------------------------- NEXT-3 recency-weighted mean (fn. 3)
def test_ewma_update_truncates_toward_zero():
    m = SchedModel(1, 1, 1, ewma=512)
    t = m.add_type("T", [("v", ALL)])
    m.submit(t, [(m.add_data(8), "inout")])
    g = m.group_of(0)
    m._record(g, 0, 1000)
    assert g["ew"][0] == 1000                      # first sample taken as is
    m._record(g, 0, 2000)
    assert g["ew"][0] == 1500                      # 1000 + 1000 * 512 / 1024
    m._record(g, 0, 500)
    assert g["ew"][0] == 1000                      # 1500 - 1000 * 512 / 1024
    assert g["sum"][0] // g["n"][0] == 1166        # the arithmetic mean is still kept (L408-411)
    # w = 300: the correction |d| * 300 / 1024 is truncated toward zero in both directions
    m2 = SchedModel(1, 1, 1, ewma=300)
    t2 = m2.add_type("T", [("v", ALL)])
    m2.submit(t2, [(m2.add_data(8), "inout")])
    g2 = m2.group_of(0)
    m2._record(g2, 0, 1000)
    m2._record(g2, 0, 2001)
    assert g2["ew"][0] == 1293                     # 1000 + trunc(1001 * 300 / 1024 = 293.26)
    m2._record(g2, 0, 0)
    assert g2["ew"][0] == 915                      # 1293 - trunc(378.8); floor would give 914


def test_ewma_changes_the_earliest_executor():
    """Version a ran 1000, 1000, 1000; version b ran 3000, 200, 200 (getting faster).
    Arithmetic mean: a 1000 < b 1133 -> a.  w = 512: b's weighted mean 3000 -> 1600 -> 900 < 1000
    -> b (footnote 3: more weight to recent executions)."""
    for ewma, want in ((0, 0), (512, 1)):
        m = SchedModel(1, 1, 3, ewma=ewma)
        t = m.add_type("T", [("a", ALL), ("b", ALL)])
        x = m.submit(t, [(m.add_data(64), "inout")])
        g = m.group_of(x)
        for v, xs in ((0, (1000, 1000, 1000)), (1, (3000, 200, 200))):
            for d in xs:
                m._record(g, v, d)
            g["assigned"][v] = 3
        assert m._check_switch(g, t) == [] and g["reliable"]
        _reset_queues(m)
        v, w, est, phase = m.decide(x, 0)
        assert (v, phase) == (want, 1)
        assert est == (1000 if want == 0 else 900)


# --------------------------------------------------- NEXT-1 locality-aware earliest executor
def _locality_model(gbps):
    m = SchedModel(2, 1, 1, locality_gbps=gbps)
    t = m.add_type("T", [("v", ALL)])
    d0 = m.add_data(4000, home=0)     # valid on gpu 0
    d1 = m.add_data(1000, home=1)     # valid on gpu 1
    x = m.submit(t, [(d0, "in"), (d1, "inout")])
    m.load_table([(t, 5000, [(1000, 1)])])
    return m, x


def test_locality_term_in_eft():
    """Worker 0 (gpu 0) has 1500 ns of work; the task needs d0 (4000 B, on gpu 0) and d1
    (1000 B, on gpu 1); mean 1000.
      no locality: EFT w0 = 1500 + 1000 = 2500, w1 = 0 + 1000 = 1000 -> w1
      1 GB/s:      w0 = 2500 + 1000 (d1 missing) = 3500, w1 = 1000 + 4000 (d0) = 5000 -> w0
      4 GB/s:      w0 = 2500 + 250 = 2750, w1 = 1000 + 1000 = 2000 -> w1"""
    for gbps, want in ((0, 1), (1, 0), (4, 1)):
        m, x = _locality_model(gbps)
        _reset_queues(m)
        m.running[0] = (99, 0, 1500)
        v, w, est, phase = m.decide(x, 0)
        assert (w, phase, est) == (want, 1, 1000), gbps


def test_locality_validity_follows_decisions():
    """2 GPUs x 1 slot, 1 GB/s, every task 1000 ns.  t0 (d0 in, d1 inout), t1 (d1 in, d2 inout);
    d0 4000 B on gpu 0, d1 1000 B on gpu 1, d2 500 B on gpu 1.
      t0 at 0:    w0 = 0 + 1000 + 1000 (d1) = 2000, w1 = 1000 + 4000 (d0) = 5000 -> w0, runs 0-1000;
                  the write makes d1 valid on gpu 0 ONLY.
      t1 at 1000: w0 = 1000 + 500 (d2) = 1500, w1 = 1000 + 1000 (d1 now only on gpu 0) = 2000 -> w0.
    (Had the write not invalidated gpu 1's copy of d1, w1 = 1000 would win.)"""
    m = SchedModel(2, 1, 1, locality_gbps=1)
    t = m.add_type("T", [("v", ALL)])
    d0, d1, d2 = m.add_data(4000, home=0), m.add_data(1000, home=1), m.add_data(500, home=1)
    m.submit(t, [(d0, "in"), (d1, "inout")])
    m.submit(t, [(d1, "in"), (d2, "inout")])
    m.load_table([(t, 5000, [(1000, 1)]), (t, 1500, [(1000, 1)])])
    log = m.simulate(lambda ty, nb, v: 1000)
    assert log == [(0, 0, 0, 0, 0, 1000, 1), (1, 0, 0, 1000, 1000, 2000, 1)]
    assert m.vvalid[d1] == {0} and m.vvalid[d0] == {0} and m.vvalid[d2] == {0}


# ------------------------------------------------- NEXT-4 bottom level + queue depth (R29)
def _prio_model(priority, qdepth):
    """t0 alone; chain t1 -> t2 -> t3; chain t4 -> t5; one worker, one version, 10 ns each."""
    m = SchedModel(1, 1, 1, priority=priority, qdepth=qdepth)
    t = m.add_type("T", [("v", ALL)])
    a, b, c = m.add_data(8), m.add_data(8), m.add_data(8)
    m.submit(t, [(a, "inout")])                     # t0
    for _ in range(3):
        m.submit(t, [(b, "inout")])                 # t1, t2, t3
    for _ in range(2):
        m.submit(t, [(c, "inout")])                 # t4, t5
    m.load_table([(t, 8, [(10, 1)])])
    return m


def test_bottom_levels():
    # 1 + max over successors, a task without successors = 1 (off-by-one would shift all)
    assert _prio_model(2, 1).bottom_levels() == [1, 3, 2, 1, 2, 1]


def test_slacks():
    # R38: top levels [1, 1, 2, 3, 1, 2], longest path L = 3 (t1 -> t2 -> t3); slack = L - (tl +
    # bl - 1): t0 3 - 1 = 2, the chain 0, t4 / t5 3 - 2 = 1 (an exclusive "< 1" or a missing -1
    # would change the critical set)
    assert _prio_model(2, 1).slacks() == [2, 0, 0, 0, 1, 1]


def test_bottom_level_order_with_queue_depth_1():
    """Ready at 0: t0 (bl 1, slack 2), t1 (bl 3), t4 (bl 2).  Depth 1: one task per worker at a
    time, the rest stay in the ready heap: slack <= 1 first (R38), then largest bl, then id.
      0: t1.  10: t2 (bl 2) ties t4 (bl 2) -> lower id t2.  20: t4 (bl 2).
      30: t0, t3, t5 all bl 1, t0 off the critical path -> t3 at 30, t5 at 40, t0 at 50
      (bottom level alone would run t0 at 30)."""
    log = _prio_model(2, 1).simulate(lambda ty, nb, v: 10)
    assert [(r[0], r[3], r[4]) for r in log] == [(1, 0, 0), (2, 10, 10), (4, 20, 20), (3, 30, 30),
                                                (5, 40, 40), (0, 50, 50)]


def test_weighted_bottom_level_uses_learned_means():
    """R29: types A (learned mean 100 ns) and B (10 ns); chain a0 -> a1 (t0, t1) and chain
    b0 -> b1 -> b2 (t2, t3, t4); one worker, depth 1.  Weighted bottom levels: a0 = 200, a1 =
    100, b0 = 30, b1 = 20, b2 = 10 (unit levels would be 2, 1, 3, 2, 1).  Slack (unit): L = 3,
    every task <= 1, so all are on the critical path and the weighted level decides:
      0: a0 (200 > 30), runs 0-100.  100: a1 (100) before b0 (30), runs 100-200.  200: b0,
      210: b1, 220: b2.  (By unit levels b0 would go first, at 0.)  A task of an unlearned
    group weighs 1000 ns."""
    m = SchedModel(1, 1, 1, priority=2, qdepth=1)
    ta = m.add_type("A", [("v", ALL)])
    tb = m.add_type("B", [("v", ALL)])
    a, b = m.add_data(8), m.add_data(8)
    for _ in range(2):
        m.submit(ta, [(a, "inout")])
    for _ in range(3):
        m.submit(tb, [(b, "inout")])
    m.load_table([(ta, 8, [(100, 1)]), (tb, 8, [(10, 1)])])
    assert m.weighted_bottom_levels() == [200, 100, 30, 20, 10]
    log = m.simulate(lambda ty, nb, v: 100 if ty == ta else 10)
    assert [(r[0], r[3]) for r in log] == [(0, 0), (1, 100), (2, 200), (3, 210), (4, 220)]
    m2 = SchedModel(1, 1, 1, priority=2, qdepth=1)
    t2 = m2.add_type("A", [("v", ALL)])
    d = m2.add_data(8)
    for _ in range(2):
        m2.submit(t2, [(d, "inout")])
    assert m2.weighted_bottom_levels() == [2000, 1000]


def _crit_model():
    """Chain a0 -> ... -> a5 (the critical path, L = 6); chain b0 -> b1 -> b2 -> b3 (bl 4, slack
    2); one worker, depth 1, 10 ns each."""
    m = SchedModel(1, 1, 1, priority=2, qdepth=1)
    t = m.add_type("T", [("v", ALL)])
    a, b = m.add_data(8), m.add_data(8)
    for _ in range(6):
        m.submit(t, [(a, "inout")])                 # t0 .. t5
    for _ in range(4):
        m.submit(t, [(b, "inout")])                 # t6 .. t9
    m.load_table([(t, 8, [(10, 1)])])
    return m


def test_critical_path_overtakes_larger_bottom_level():
    """R38.  0: t0 (bl 6).  10: t1 (bl 5) vs t6 (bl 4) -> t1.  20: t2 (bl 4) ties t6 (bl 4), t2
    critical -> t2.  30: t3 (bl 3, critical) vs t6 (bl 4, slack 2): critical first -> t3 (by
    bottom level alone t6 would go at 30 and the chain would end at 100, not 60).  40: t4,
    50: t5, then the b chain 60-90."""
    m = _crit_model()
    assert m.slacks() == [0] * 6 + [2] * 4
    log = m.simulate(lambda ty, nb, v: 10)
    assert [(r[0], r[3]) for r in log] == [(0, 0), (1, 10), (2, 20), (3, 30), (4, 40), (5, 50), (6, 60),
                                           (7, 70), (8, 80), (9, 90)]


def test_bottom_level_order_without_queue_cap():
    """No cap: every ready task is decided at once, in bottom-level order t1, t4, t0 (all at 0,
    queued 0-10, 10-20, 20-30); t2 ready at 10 runs 30-40; t5 ready at 20 runs 40-50; t3 ready
    at 40 runs 50-60."""
    log = _prio_model(2, 0).simulate(lambda ty, nb, v: 10)
    assert [(r[0], r[3], r[4]) for r in log] == [(1, 0, 0), (4, 0, 10), (0, 0, 20), (2, 10, 30),
                                                (5, 20, 40), (3, 40, 50)]


def test_fifo_order_paper_literal():
    """priority 0 (R15): ready tasks in ascending id at 0 (t0, t1, t4), successors as released."""
    log = _prio_model(0, 0).simulate(lambda ty, nb, v: 10)
    assert [(r[0], r[3], r[4]) for r in log] == [(0, 0, 0), (1, 0, 10), (4, 0, 20), (2, 20, 30),
                                                (5, 30, 40), (3, 40, 50)]


# ------------------------------------------------------ learning: rr (paper-literal) vs hold
def _learn_log(learning, slots=1):
    m = SchedModel(1, slots, 1, learning=learning)
    t = m.add_type("T", [("a", ALL), ("b", ALL)])
    for _ in range(4):
        m.submit(t, [(m.add_data(8), "inout")])
    return m.simulate(lambda ty, nb, v: [100, 50][v])


def test_learning_rr_keeps_cycling():
    """lambda = 1, versions a (100 ns) / b (50 ns), four independent tasks, one worker.
    rr (R12, paper-literal "Round-Robin ... distributing"): every version reached lambda
    assignments after t0, t1 but nothing completed: keep cycling a, b, a, b, all in learning."""
    assert _learn_log("rr") == [(0, 0, 0, 0, 0, 100, 0), (1, 1, 0, 0, 100, 150, 0),
                                (2, 0, 0, 0, 150, 250, 0), (3, 1, 0, 0, 250, 300, 0)]


def test_learning_hold_waits_for_completions():
    """hold (R12 default): t2, t3 wait until both learning runs completed (150), then the
    earliest executor picks b (mean 50): t2 150-200, t3 (busy 50 + 50) 200-250."""
    assert _learn_log("hold") == [(0, 0, 0, 0, 0, 100, 0), (1, 1, 0, 0, 100, 150, 0),
                                  (2, 1, 0, 150, 150, 200, 1), (3, 1, 0, 150, 200, 250, 1)]


def test_learning_worker_tie_breaks_by_queue_length():
    """Two slots, rr: unmeasured versions are estimated at 0 (R13), so every worker is 0 busy;
    ties go to the shorter queue, then the lower id: t0 -> w0, t1 -> w1, t2 -> w0 (both hold
    one task: lower id), t3 -> w1."""
    log = _learn_log("rr", slots=2)
    assert [(r[0], r[1], r[2]) for r in log] == [(0, 0, 0), (1, 1, 1), (2, 0, 0), (3, 1, 1)]

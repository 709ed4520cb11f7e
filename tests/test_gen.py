"""Input generator sanity (vsgen): exact fp32 values, range, determinism, layout."""
import numpy as np

import vsgen


def test_uniform_exact_fp32_and_range():
    u = vsgen.uniform_idx(3, np.arange(100000, dtype=np.uint64))
    assert np.all(u >= -1.0) and np.all(u < 1.0)
    assert np.array_equal(u.astype(np.float32).astype(np.float64), u)
    assert abs(u.mean()) < 0.01
    assert abs(u.var() - 1 / 3) < 0.01


def test_global_indexing_independent_of_tiling():
    a = vsgen.uniform(5, 64, 48)
    t = vsgen.to_tiles(a, 16)
    assert t.shape == (4, 3, 16, 16)
    assert np.array_equal(t[2, 1], a[32:48, 16:32])
    assert np.array_equal(vsgen.from_tiles(t), a)


def test_spd_symmetric_and_diag():
    n = 300
    A = vsgen.spd(2, n, np.float64)
    assert np.array_equal(A, A.T)
    assert np.all(np.diag(A) > vsgen.spd_alpha(n) - 1)
    assert np.linalg.eigvalsh(A).min() > 0


def test_known_values_stable():
    # Guard against silent generator changes (the device generator must match these bits).
    v = vsgen.uniform_idx(1, np.array([0, 1, 2, 12345], dtype=np.uint64))
    again = vsgen.uniform_idx(1, np.array([0, 1, 2, 12345], dtype=np.uint64))
    assert np.array_equal(v, again)
    assert len(set(v.tolist())) == 4

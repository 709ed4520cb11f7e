"""cfg5: interleaved matmuls of several tile sizes on the live GPU runtime.

Pins what the learning rule fixes whatever the measured times are (L428-447, R12): every
group makes exactly lambda learning runs per version, its first reliable decision is number
V*lambda + 1, and reliable decisions pick the version with the smallest learned mean
(one GPU: homogeneous workers, so the earliest executor's version is the fastest mean at the
time of the decision, L448-475).
Results stay within the fp32-class gate against the oracle.
"""
import os
import sys

import numpy as np
import pytest

import oracle
import paper_conf_ipps_planasbal13_b200 as vs
import vsgen

pytestmark = pytest.mark.gpu
sys.path.insert(0, os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))), "tools"))


@pytest.mark.parametrize("lam", [1, 2])
def test_cfg5_interleaved_convergence(gpu, lam):
    import sweep_cfg5 as sw
    import torch
    sizes = [128, 256, 512]
    log, groups, task_b, keep = sw.run_sweep_once(lam, sizes, sw.VERSIONS, slots=4)
    V = len(sw.VERSIONS)
    assert len(log) == len(sizes) * 64
    for bi, b in enumerate(sizes):
        g = groups[3 * b * b * 4]
        assert g["reliable"] and g["first_reliable"] == V * lam + 1, g
        recs = [r for r in log if task_b[r[0]] == b]
        learn = [r[1] for r in recs[:V * lam]]
        assert sorted(learn) == sorted(list(range(V)) * lam)
        # means keep learning in the reliable phase (a14), so a near-tie may switch the pick
        # mid-run: every pick is a version whose final mean is near the fastest, most are it
        means = np.array(g["mean_ns"], dtype=np.float64)
        fastest = int(np.argmin(means))
        post = [r[1] for r in recs[V * lam:]]
        assert all(means[v] <= 1.5 * means[fastest] for v in post), (b, g)
        second = min(means[v] for v in range(V) if v != fastest)
        if second >= 1.2 * means[fastest]:   # a clear winner (not a near-tie) takes most picks
            assert sum(v == fastest for v in post) >= len(post) // 2, (b, g)
        if b > 256:
            continue
        # parity of the result (C0 = 0, A = u(100+lam), B = u(1100+lam), N = 4b)
        n = 4 * b
        C = vsgen.from_tiles(keep[3 * bi + 2].view(4, 4, b, b).cpu().numpy())
        A = vsgen.uniform(100 + lam, n, n)
        B = vsgen.uniform(1100 + lam, n, n)
        assert oracle.relF(C, oracle.matmul(A, B)) <= 1e-5
    torch.cuda.synchronize()

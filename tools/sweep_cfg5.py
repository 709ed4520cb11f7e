"""cfg5 — version-selection sweep: scheduler convergence on mixed tile sizes.

For every b in {128, 256, 512, 1024, 2048} an independent 4x4x4 tiled matmul (N = 4b, fp32,
Fig 1 driver order i, j, k) is submitted through the C ABI, the five matmuls INTERLEAVED task by
task (task t of every b before task t+1 of any), on 1 GPU, for lambda = 1..5.  Every b is its own
group (DataSetSize = 3 b^2 4 B, L363-370).  Per group and lambda the sweep reports:

  first_reliable     1-based index (within the group) of its first reliable-phase decision;
                     the rule (L428-447, R12 hold) fixes it at V*lambda + 1
  fastest_gt         the ground-truth fastest version: median of 50 isolated runs per version
                     (no co-running work; back-to-back launches on one stream, CUDA events
                     between consecutive launches)
  picks_fastest      the version the reliable phase chose (all its decisions) == fastest_gt
  frac_fastest       fraction of post-learning decisions that chose fastest_gt
  regret_us          learning regret: sum over the group's decisions of (t_gt(chosen) - t_gt(fastest))
  mean_us            the scheduler's learned mean per version (R17 device-recorded) beside t_gt

  python tools/sweep_cfg5.py [--lams 1,2,3,4,5] [--sizes 128,...] [--out gpurun_out/cfg5.json]

Inputs: A = u(100+lambda), B = u(1100+lambda), C0 = 0 (SURVEY §8(d) cfg5 seeds), tile-major.
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import sys

import torch

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")
import paper_conf_ipps_planasbal13_b200 as vs  # noqa: E402

SIZES = [128, 256, 512, 1024, 2048]
VERSIONS = [vs.VS_V_SIMT_F32, vs.VS_V_TC_3XTF32, vs.VS_V_F64IN_F32IO, vs.VS_V_TC_3XF16]
NT = 4


def ground_truth(b, versions, runs=50):
    """Median of `runs` isolated launches per version (operand forms prepared beforehand, as the
    runtime caches them, R30), us."""
    A = torch.empty(b * b, dtype=torch.float32, device="cuda")
    B = torch.empty_like(A)
    C = torch.zeros_like(A)
    vs.vs_gen_uniform(7, b, b, vs.VS_F32, b, A.data_ptr())
    vs.vs_gen_uniform(8, b, b, vs.VS_F32, b, B.data_ptr())
    info = torch.zeros(1, dtype=torch.int32, device="cuda")
    stream = torch.cuda.current_stream()
    out = {}
    for v in versions:
        keep, fp = [], []
        for i, t in enumerate((A, B, C)):
            f = vs.vs_operand_form(vs.VS_T_MATMUL, v, i)
            if f > 0:
                buf = torch.empty(vs.vs_form_bytes(f, b), dtype=torch.uint8, device="cuda")
                vs.vs_form_make(f, b, t.data_ptr(), buf.data_ptr(), stream.cuda_stream)
                keep.append(buf)
                fp.append(buf.data_ptr())
            else:
                fp.append(0)
        ptrs = [A.data_ptr(), B.data_ptr(), C.data_ptr()] + fp
        for _ in range(3):
            vs.vs_tile_run_prepared(vs.VS_T_MATMUL, v, b, ptrs, info.data_ptr(), stream.cuda_stream)
        torch.cuda.synchronize()
        # back-to-back launches on one stream with an event between consecutive ones: each
        # interval is one kernel's device time (+ the inter-kernel gap), without the host's
        # launch latency that an event pair around a lone launch would include
        evs = [torch.cuda.Event(enable_timing=True) for _ in range(runs + 1)]
        evs[0].record()
        for i in range(runs):
            vs.vs_tile_run_prepared(vs.VS_T_MATMUL, v, b, ptrs, info.data_ptr(), stream.cuda_stream)
            evs[i + 1].record()
        torch.cuda.synchronize()
        ts = [evs[i].elapsed_time(evs[i + 1]) * 1e3 for i in range(runs)]
        out[v] = statistics.median(ts)
    return out


def run_sweep_once(lam, sizes, versions, slots=8, mode=None):
    mask = 0
    for v in versions:
        mask |= 1 << v
    kw = dict(lam=lam, slots_per_gpu=slots)
    if mode is not None:
        kw["mode"] = mode
    rt = vs.Runtime(**kw)
    types = rt.vs_register_builtins(vs.VS_F32, mask)
    mm = types[vs.VS_T_MATMUL]
    keep, ids, task_b = [], {}, {}
    for b in sizes:
        n = NT * b
        A = torch.empty(n * n, dtype=torch.float32, device="cuda")
        B = torch.empty_like(A)
        C = torch.zeros_like(A)
        vs.vs_gen_uniform(100 + lam, n, n, vs.VS_F32, b, A.data_ptr())
        vs.vs_gen_uniform(1100 + lam, n, n, vs.VS_F32, b, B.data_ptr())
        keep += [A, B, C]
        reg = lambda T: [rt.vs_data_register(T.data_ptr() + t * b * b * 4, 0, b * b * 4)  # noqa: E731
                         for t in range(NT * NT)]
        ids[b] = (reg(A), reg(B), reg(C))
    torch.cuda.synchronize()
    order = [(i, j, k) for i in range(NT) for j in range(NT) for k in range(NT)]
    for (i, j, k) in order:
        for b in sizes:
            a, bb, c = ids[b]
            t = rt.vs_submit(mm, [a[i * NT + k], bb[k * NT + j], c[i * NT + j]])
            task_b[t] = b
    rt.vs_wait_all()
    log = rt.vs_decision_log()
    groups = {g["bytes"]: g for g in rt.vs_group_stats()}
    rt.close()
    return log, groups, task_b, keep


def analyse(lam, log, groups, task_b, sizes, versions, gt):
    V = len(versions)
    res = []
    for b in sizes:
        g = groups[3 * b * b * 4]
        recs = [r for r in log if task_b.get(r[0]) == b]   # decision order
        chosen = [versions[r[1]] if r[1] < len(versions) else r[1] for r in recs]
        fastest = min(gt[b], key=gt[b].get)
        fr = g["first_reliable"]
        post = chosen[fr - 1:] if fr > 0 else []
        regret = sum(gt[b][v] - gt[b][fastest] for v in chosen)
        reliable_choice = sorted(set(post))
        res.append({
            "lambda": lam, "b": b, "V": V, "decisions": len(chosen),
            "first_reliable": fr, "expected_first_reliable": V * lam + 1,
            "fastest_gt": vs.VERSION_NAMES[fastest],
            "reliable_choice": [vs.VERSION_NAMES[v] for v in reliable_choice],
            "picks_fastest": reliable_choice == [fastest],
            # near-ties: every reliable pick within 5 % of the ground-truth fastest time
            "picks_within_5pct": bool(post) and all(gt[b][v] <= 1.05 * gt[b][fastest] for v in post),
            "frac_fastest": (sum(1 for v in post if v == fastest) / len(post)) if post else 0.0,
            "regret_us": round(regret, 2),
            "gt_us": {vs.VERSION_NAMES[v]: round(t, 2) for v, t in gt[b].items()},
            "mean_us": {g["versions"][i]: round(m / 1e3, 2) for i, m in enumerate(g["mean_ns"])},
            # learned mean (R17, device-recorded under co-running) / isolated ground truth
            "mean_over_gt": {g["versions"][i]: round(m / 1e3 / gt[b][versions[i]], 3)
                             for i, m in enumerate(g["mean_ns"]) if m > 0},
            "n": g["n"]})
    return res


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--lams", default="1,2,3,4,5")
    ap.add_argument("--sizes", default=",".join(map(str, SIZES)))
    ap.add_argument("--slots", type=int, default=8)
    ap.add_argument("--runs", type=int, default=50)
    ap.add_argument("--out", default="")
    a = ap.parse_args()
    sizes = [int(x) for x in a.sizes.split(",")]
    lams = [int(x) for x in a.lams.split(",")]
    torch.cuda.set_device(0)
    gt = {b: ground_truth(b, VERSIONS, a.runs) for b in sizes}
    allres = []
    for lam in lams:
        log, groups, task_b, _ = run_sweep_once(lam, sizes, VERSIONS, a.slots)
        for r in analyse(lam, log, groups, task_b, sizes, VERSIONS, gt):
            print(json.dumps(r))
            allres.append(r)
    summary = {
        "config": "cfg5: 5 interleaved 4x4x4 matmuls b=%s, lambda=%s, %d slots, versions %s" % (
            sizes, lams, a.slots, [vs.VERSION_NAMES[v] for v in VERSIONS]),
        "first_reliable_rule_holds": all(r["first_reliable"] == r["expected_first_reliable"] for r in allres),
        "groups_picking_fastest": sum(r["picks_fastest"] for r in allres), "groups": len(allres),
        "groups_picking_within_5pct": sum(r["picks_within_5pct"] for r in allres),
        "mean_frac_fastest": round(sum(r["frac_fastest"] for r in allres) / len(allres), 4),
        "mean_over_gt_range": [min(x for r in allres for x in r["mean_over_gt"].values()),
                               max(x for r in allres for x in r["mean_over_gt"].values())],
        "total_regret_us": round(sum(r["regret_us"] for r in allres), 1)}
    print(json.dumps(summary))
    if a.out:
        json.dump({"summary": summary, "groups": allres}, open(a.out, "w"), indent=1)


if __name__ == "__main__":
    main()

"""Measured critical path of a tiled-Cholesky step from a bench decision log (bench.py
--only ch --dump-log LOG, or a combined log): starting from the task that ends last, walk back
through the predecessor that ended last (the one the task actually waited for) and print each
link's device interval and the gap before it (decision / launch / queueing / form builds), with
totals per task type: python tools/crit_path.py LOG [nt]"""
import json
import sys

sys.path.insert(0, __import__("os").path.dirname(__file__))
from chol_cp import ids  # noqa: E402


def preds(key):
    kind, i, j, k = key
    if kind == "potrf":
        return [("syrk", k, k, k - 1)] if k > 0 else []
    if kind == "trsm":
        return [("potrf", k, k, k)] + ([("gemm", i, k, k - 1)] if k > 0 else [])
    if kind == "syrk":
        return [("trsm", i, k, k)] + ([("syrk", i, i, k - 1)] if k > 0 else [])
    return [("trsm", i, k, k), ("trsm", j, k, k)] + ([("gemm", i, j, k - 1)] if k > 0 else [])


def main(path, nt=32):
    d = json.load(open(path))
    log = sorted((r for r in d["log"] if r[7] != 0), key=lambda r: r[0])
    n = len(ids(nt))
    st = log[-n:]
    idx = dict(zip(ids(nt), st))
    t0 = min(r[4] for r in st)
    cur = max(idx, key=lambda k: idx[k][5])
    path = []
    while cur is not None:
        path.append(cur)
        ps = [p for p in preds(cur) if p in idx]
        cur = max(ps, key=lambda p: idx[p][5]) if ps else None
    path.reverse()
    tot, gaps = {}, {}
    prev_end = None
    for key in path:
        r = idx[key]
        dur = (r[5] - r[4]) / 1e3
        gap = (r[4] - prev_end) / 1e3 if prev_end is not None else 0.0
        tot[key[0]] = tot.get(key[0], 0.0) + dur
        gaps[key[0]] = gaps.get(key[0], 0.0) + max(gap, 0.0)
        print("%-22s start %8.0f  gap %6.0f  dur %5.0f  v%d" % (key, (r[4] - t0) / 1e3, gap, dur, r[1]))
        prev_end = r[5]
    span = (max(r[5] for r in st) - t0) / 1e3
    print("step %.0f us; path of %d links: kernels %s; gaps before %s" % (
        span, len(path), {k: round(v) for k, v in tot.items()}, {k: round(v) for k, v in gaps.items()}))


if __name__ == "__main__":
    main(sys.argv[1], *(int(x) for x in sys.argv[2:3]))

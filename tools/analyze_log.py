"""Summarise a bench decision log (bench.py --dump-log): per (type, version) task counts,
mean GPU time, union busy time, and whole-GPU busy fraction of the timed region."""
import json
import sys


def union(iv):
    tot, cs, ce = 0, None, None
    for s, e in sorted(iv):
        if ce is None or s > ce:
            if ce is not None:
                tot += ce - cs
            cs, ce = s, e
        else:
            ce = max(ce, e)
    if ce is not None:
        tot += ce - cs
    return tot


def main(path):
    d = json.load(open(path))
    log, groups = d["log"], d["groups"]
    tn = {g["type"]: g["type_name"] for g in groups}
    vn = {g["type"]: g["versions"] for g in groups}
    per = {}
    allv = []
    for (task, v, w, td, ts, te, ph, ty) in log:
        k = (tn[ty], vn[ty][v])
        x = per.setdefault(k, {"n": 0, "dur": 0, "iv": []})
        x["n"] += 1
        x["dur"] += te - ts
        x["iv"].append((ts, te))
        allv.append((ts, te))
    t0 = min(s for s, _ in allv)
    t1 = max(e for _, e in allv)
    print("timed span %.2f ms, GPU busy (union of task intervals) %.2f ms (%.1f%%)" % (
        (t1 - t0) / 1e6, union(allv) / 1e6, 100 * union(allv) / (t1 - t0)))
    for k, x in sorted(per.items()):
        print("%-16s %-12s n=%6d mean=%8.1f us  union=%8.2f ms" % (k[0], k[1], x["n"], x["dur"] / x["n"] / 1e3,
                                                                   union(x["iv"]) / 1e6))
    for g in groups:
        print(g["type_name"], g["bytes"], "reliable" if g["reliable"] else "learning", "n=", g["n"],
              "mean_us=", [round(m / 1e3, 1) for m in g["mean_ns"]])


if __name__ == "__main__":
    main(sys.argv[1])

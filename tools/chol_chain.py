"""Critical chain of the tiled Cholesky in a bench decision log (bench.py --only ch):
per step k the device interval of potrf(k), trsm(k+1,k), syrk(k+1,k) and the gap between
consecutive links (waiting time on the chain)."""
import json
import sys


def cholesky_ids(nt):
    """(kind, i, j, k) in submission order (R5)."""
    out = []
    for k in range(nt):
        out.append(("potrf", k, k, k))
        for i in range(k + 1, nt):
            out.append(("trsm", i, k, k))
        for i in range(k + 1, nt):
            for j in range(k + 1, i):
                out.append(("gemm", i, j, k))
            out.append(("syrk", i, i, k))
    return out


def main(path, nt=32, offset=0, per_step=None):
    """offset: tasks submitted before the Cholesky in each step (4096 matmul tasks in the
    default bench step); per_step: tasks per step (default: the Cholesky's alone)."""
    d = json.load(open(path))
    log = d["log"]
    iss = d.get("issue") or [0] * len(log)
    log = [list(r) + [iss[n]] for n, r in enumerate(log)]
    ids = cholesky_ids(nt)
    per = per_step or (len(ids) + offset)
    tmin = min(r[0] for r in log)
    by = {}
    for r in log:
        step, pos = (r[0] - tmin) // per, (r[0] - tmin) % per - offset
        if pos >= 0:
            by.setdefault(step, {})[pos] = r
    rs = by[max(by)]
    t0 = min(r[4] for r in rs.values())
    idx = {x: n for n, x in enumerate(ids)}
    tot_wait = 0
    prev_end = None
    for k in range(nt):
        p = rs[idx[("potrf", k, k, k)]]
        line = "k=%2d potrf %7.2f-%7.2f (%5.0f us)" % (k, (p[4] - t0) / 1e6, (p[5] - t0) / 1e6, (p[5] - p[4]) / 1e3)
        if prev_end is not None:
            line += " wait %4.0f us (issued %+5.0f)" % ((p[4] - prev_end) / 1e3, (p[8] - prev_end) / 1e3)
            tot_wait += p[4] - prev_end
        if k + 1 < nt:
            t = rs[idx[("trsm", k + 1, k, k)]]
            s = rs[idx[("syrk", k + 1, k + 1, k)]]
            line += " | trsm +%4.0f %4.0f us (issued %+5.0f) | syrk +%4.0f %4.0f us (issued %+5.0f)" % (
                (t[4] - p[5]) / 1e3, (t[5] - t[4]) / 1e3, (t[8] - p[5]) / 1e3,
                (s[4] - t[5]) / 1e3, (s[5] - s[4]) / 1e3, (s[8] - t[5]) / 1e3)
            prev_end = s[5]
        print(line)
    print("total wait before potrf: %.2f ms" % (tot_wait / 1e6))


if __name__ == "__main__":
    main(sys.argv[1], offset=int(sys.argv[2]) if len(sys.argv) > 2 else 0)

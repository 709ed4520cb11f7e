"""Critical chain of a Cholesky-only bench log (bench.py --only ch --dump-log): per step k the
potrf(k) -> trsm(k+1,k) -> syrk(k+1,k) -> potrf(k+1) links, their device intervals and the
waits between them (us)."""
import json
import sys


def ids(nt):
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


def main(path, nt=32, step=-1):
    d = json.load(open(path))
    # a combined bench log also holds the matmul's tasks (type 0 = MATMUL): the chain is the
    # Cholesky's tasks in submission order
    log = sorted((r for r in d["log"] if r[7] != 0), key=lambda r: r[0])
    n = len(ids(nt))
    steps = [log[i:i + n] for i in range(0, len(log), n)]
    rs = steps[step]
    idx = {key: r for key, r in zip(ids(nt), rs)}
    t0 = min(r[4] for r in rs)
    tot = {"potrf": 0, "trsm": 0, "syrk": 0, "wait": 0}
    prev_end = None
    for k in range(nt):
        p = idx[("potrf", k, k, k)]
        line = "k=%2d potrf %7.0f-%7.0f (%4.0f)" % (k, (p[4] - t0) / 1e3, (p[5] - t0) / 1e3, (p[5] - p[4]) / 1e3)
        tot["potrf"] += p[5] - p[4]
        if prev_end is not None:
            tot["wait"] += max(0, p[4] - prev_end)
        if k + 1 < nt:
            t = idx[("trsm", k + 1, k, k)]
            s = idx[("syrk", k + 1, k + 1, k)]
            line += " | trsm +%5.0f (%3.0f) | syrk +%5.0f (%3.0f)" % ((t[4] - p[5]) / 1e3, (t[5] - t[4]) / 1e3,
                                                                     (s[4] - t[5]) / 1e3, (s[5] - s[4]) / 1e3)
            tot["trsm"] += t[5] - t[4]
            tot["syrk"] += s[5] - s[4]
            tot["wait"] += max(0, t[4] - p[5]) + max(0, s[4] - t[5])
            prev_end = s[5]
        print(line)
    span = max(r[5] for r in rs) - t0
    print("step %.2f ms; chain: potrf %.2f ms, trsm %.2f, syrk %.2f, waits %.2f" % (
        span / 1e6, tot["potrf"] / 1e6, tot["trsm"] / 1e6, tot["syrk"] / 1e6, tot["wait"] / 1e6))


if __name__ == "__main__":
    main(sys.argv[1])

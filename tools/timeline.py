"""Per-step timeline of a bench decision log: for each step (tasks grouped by id ranges),
the span of each task type and the busy fraction in 10 ms bins (mean CTAs in flight)."""
import json
import sys

CTAS = {"GEMM": 16, "MATM": 16, "SYRK": 10, "TRSM": 8, "POTR": 8}


def main(path, per_step=10080):
    d = json.load(open(path))
    log, groups = d["log"], d["groups"]
    tn = {g["type"]: g["type_name"][:4] for g in groups}
    tmin = min(r[0] for r in log)
    steps = {}
    for r in log:
        steps.setdefault((r[0] - tmin) // per_step, []).append(r)
    for si, rs in sorted(steps.items()):
        t0 = min(r[4] for r in rs)
        t1 = max(r[5] for r in rs)
        print("step %d: %.2f ms" % (si, (t1 - t0) / 1e6))
        for ty in sorted(set(tn[r[7]] for r in rs)):
            x = [r for r in rs if tn[r[7]] == ty]
            print("   %s n=%5d first start %7.2f  last end %7.2f ms" % (ty, len(x), (min(r[4] for r in x) - t0) / 1e6,
                                                                      (max(r[5] for r in x) - t0) / 1e6))
        nb = int((t1 - t0) / 5e6) + 1
        occ = [0.0] * nb
        for r in rs:
            c = CTAS.get(tn[r[7]], 16)
            s, e = r[4] - t0, r[5] - t0
            b = int(s / 5e6)
            while s < e and b < nb:
                be = (b + 1) * 5e6
                occ[b] += c * (min(e, be) - s) / 5e6
                s = be
                b += 1
        print("   mean CTAs per 5 ms:", " ".join("%.0f" % o for o in occ))


if __name__ == "__main__":
    main(sys.argv[1])

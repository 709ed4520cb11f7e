"""Task concurrency histogram of a bench decision log (bench.py --dump-log): share of the
timed span during which k tasks were executing on the device, and mean CTAs in flight."""
import collections
import json
import sys

CTAS = {"GEMM": 16, "MATM": 16, "SYRK": 10, "TRSM": 8, "POTR": 8}


def main(path):
    d = json.load(open(path))
    log, groups = d["log"], d["groups"]
    tn = {g["type"]: g["type_name"] for g in groups}
    ev = []
    for r in log:
        k = tn[r[7]][:4]
        ev.append((r[4], 1, CTAS.get(k, 16)))
        ev.append((r[5], -1, CTAS.get(k, 16)))
    ev.sort()
    cur = ctas = 0
    last = ev[0][0]
    hist = collections.Counter()
    cta_t = 0
    for t, dl, c in ev:
        hist[cur] += t - last
        cta_t += ctas * (t - last)
        cur += dl
        ctas += dl * c
        last = t
    tot = sum(hist.values())
    print(" ".join("%d:%.0f%%" % (k, 100 * hist[k] / tot) for k in sorted(hist)), " mean CTAs %.1f" % (cta_t / tot))


if __name__ == "__main__":
    for p in sys.argv[1:]:
        print(p)
        main(p)

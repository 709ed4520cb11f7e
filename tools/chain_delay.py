"""Per link of the Cholesky chain in a bench decision log (bench.py --dump-log): when the
host decided it, when its device interval started and ended (us from the step's first start;
decide times shifted onto the device clock by potrf(0)'s decide -> start offset), its worker
and version: python tools/chain_delay.py LOG [k0 k1]"""
import json
import sys

sys.path.insert(0, __import__("os").path.dirname(__file__))
from chol_cp import ids  # noqa: E402


def main(path, k0=20, k1=31, nt=32):
    d = json.load(open(path))
    log = sorted((r for r in d["log"] if r[7] != 0), key=lambda r: r[0])
    n = len(ids(nt))
    st = log[-n:]
    idx = dict(zip(ids(nt), st))
    t0 = min(r[4] for r in st)
    p0 = idx[("potrf", 0, 0, 0)]
    off = p0[3] - p0[4]
    for k in range(k0, k1):
        for key in [("potrf", k, k, k), ("trsm", k + 1, k, k), ("syrk", k + 1, k + 1, k)]:
            r = idx[key]
            print("%-22s decide %8.0f start %8.0f end %8.0f worker %2d ver %d" % (
                key, (r[3] - off - t0) / 1e3, (r[4] - t0) / 1e3, (r[5] - t0) / 1e3, r[2], r[1]))


if __name__ == "__main__":
    a = sys.argv[1:]
    main(a[0], *(int(x) for x in a[1:3]))

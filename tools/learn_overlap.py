"""Learning-phase runs of a decision log (bench.py --dump-cold-log): per learning task, its
version, device interval and the versions of the tasks overlapping it (co-running slots)."""
import json
import sys


def main(path, type_prefix="MATMUL"):
    d = json.load(open(path))
    log, groups = d["log"], d["groups"]
    tn = {g["type"]: g["type_name"] for g in groups}
    vn = {g["type"]: g["versions"] for g in groups}
    t0 = min(r[4] for r in log)
    for (task, v, w, td, ts, te, ph, ty) in log:
        if ph != 0 or not tn[ty].startswith(type_prefix):
            continue
        ov = [("%s/%s" % (tn[r[7]].split(".")[0], vn[r[7]][r[1]])) for r in log
              if r[0] != task and r[4] < te and r[5] > ts]
        print("task %5d %-12s w=%2d start=%8.1f us dur=%7.1f us  overlaps: %s" % (
            task, vn[ty][v], w, (ts - t0) / 1e3, (te - ts) / 1e3, ", ".join(sorted(set(ov)))))


if __name__ == "__main__":
    main(sys.argv[1], sys.argv[2] if len(sys.argv) > 2 else "MATMUL")

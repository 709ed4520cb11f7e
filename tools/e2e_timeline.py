"""Timeline of one end-to-end step (host-homed tiles: the runtime moves every input H2D and
writes every output back) from the decision log: when the tasks of each kind ran on the device,
against the step's wall time and the bytes moved: python tools/e2e_timeline.py [mm|ch|both]"""
import os
import sys
import time

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import bench  # noqa: E402
import paper_conf_ipps_planasbal13_b200 as vs  # noqa: E402

import torch  # noqa: E402


def main(only="both"):
    rt = vs.Runtime(bench.bench_config(vs))
    wl = bench.Workload(rt, host=True, with_mm=only in ("mm", "both"), with_ch=only in ("ch", "both"))
    wl.step()
    wl.step()
    wl.reset()
    rt.vs_decision_log_clear()
    s0 = rt.vs_stats()
    torch.cuda.synchronize()
    t0 = time.perf_counter()
    wl.submit()
    sub = (time.perf_counter() - t0) * 1e3
    rt.vs_wait_all()
    torch.cuda.synchronize()
    wall = (time.perf_counter() - t0) * 1e3
    s1 = rt.vs_stats()
    log = rt.vs_decision_log()
    d0 = min(r[4] for r in log)
    ends = max(r[5] for r in log)
    print("wall %.1f ms (submit %.1f ms, drive setup %.1f ms); device span of the tasks %.1f ms; H2D %.2f GB, D2H %.2f GB;"
          " %d tasks gated on inputs" % (
              wall, sub, (s1.host_ns_drive_setup - s0.host_ns_drive_setup) / 1e6, (ends - d0) / 1e6,
              (s1.input_tx_bytes - s0.input_tx_bytes) / 1e9, (s1.output_tx_bytes - s0.output_tx_bytes) / 1e9,
              s1.gated_tasks - s0.gated_tasks))
    for _ in range(2):
        wl.reset()
        torch.cuda.synchronize()
        t0 = time.perf_counter()
        wl.submit()
        rt.vs_wait_all()
        torch.cuda.synchronize()
        print("  again: wall %.1f ms" % ((time.perf_counter() - t0) * 1e3))
    names = {0: "mm"}
    bins = {}
    for r in log:
        k = names.get(r[7], "ch")
        b = int((r[4] - d0) / 5e6)
        bins.setdefault(k, {}).setdefault(b, 0)
        bins[k][b] += 1
    for k, h in bins.items():
        print(k, "tasks started per 5 ms:", " ".join("%d" % h.get(i, 0) for i in range(max(h) + 1)))
    ct = os.environ.get("VS_COPY_TRACE")
    if ct and os.path.exists(ct):   # copy completions of the timed step (first block after warm-up)
        blocks, cur = [], []
        for line in open(ct):
            if line.startswith("#"):
                blocks.append(cur)
                cur = []
            else:
                k, t, b = line.split()
                cur.append((int(k), float(t), int(b)))
        if len(blocks) >= 3:
            blk = blocks[2]
            for kind, name in ((0, "H2D"), (1, "D2H")):
                h = {}
                for k, t, b in blk:
                    if k == kind:
                        h[int(t / 5000)] = h.get(int(t / 5000), 0) + b
                if h:
                    print(name, "GB/s per 5 ms:", " ".join("%.0f" % (h.get(i, 0) / 5e-3 / 1e9) for i in range(max(h) + 1)),
                          "| last %.1f ms" % (max(t for k, t, b in blk if k == kind) / 1e3))
    busy = sum(r[5] - r[4] for r in log) / 1e6
    print("summed task time %.1f ms (concurrent tasks overlap)" % busy)
    rt.close()


if __name__ == "__main__":
    main(*sys.argv[1:2])

"""Host time of each phase of a bench step (reset / invalidate / submit / sync / wait_all) and
the runtime's own counters, to see where the gap between two steps goes.

python tools/step_phases.py [--steps 4]
"""
import argparse
import os
import sys
import time

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--steps", type=int, default=4)
    a = ap.parse_args()
    import torch

    import bench
    import paper_conf_ipps_planasbal13_b200 as vs
    torch.cuda.set_device(0)
    rt = vs.Runtime(bench.bench_config(vs))
    wl = bench.Workload(rt)
    wl.step()
    wl.step()
    for _ in range(a.steps):
        t0 = time.perf_counter()
        if wl.with_mm:
            wl.C.zero_()
        if wl.with_ch:
            wl.S.copy_(wl.S0)
        t1 = time.perf_counter()
        rt.vs_data_invalidate_n(wl.ids)
        t2 = time.perf_counter()
        wl.submit()
        t3 = time.perf_counter()
        torch.cuda.current_stream().synchronize()
        t4 = time.perf_counter()
        s0 = rt.vs_stats()
        rt.vs_wait_all()
        t5 = time.perf_counter()
        s1 = rt.vs_stats()
        print("restore-enqueue %.2f ms  invalidate %.2f  submit %.2f  sync %.2f  wait_all %.2f  (drive setup %.2f ms;"
              " decide+issue+poll+flush %.1f ms)"
              % ((t1 - t0) * 1e3, (t2 - t1) * 1e3, (t3 - t2) * 1e3, (t4 - t3) * 1e3, (t5 - t4) * 1e3,
                 (s1.host_ns_drive_setup - s0.host_ns_drive_setup) / 1e6,
                 (s1.host_ns_poll - s0.host_ns_poll + s1.host_ns_flush - s0.host_ns_flush) / 1e6))
    rt.close()


if __name__ == "__main__":
    main()

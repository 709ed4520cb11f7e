"""Per-CTA phase timeline of the tc_3xf16 GEMM (tcf_gemm_kernel) inside a bench step.

Needs a measurement build of the library with -DVS_TCF_TRACE installed as the package's
libvsched.so (scratch build; never the product library).  Runs the bench workload (device
tiles, warm), records every tcf CTA of one timed step and prints, over those CTAs, the median /
mean of each phase and how much of the SMs' time the CTAs covered:

    python tools/tcf_trace.py [mm|ch|both]
"""
import ctypes
import os
import sys

import numpy as np

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import bench  # noqa: E402
import paper_conf_ipps_planasbal13_b200 as vs  # noqa: E402

import torch  # noqa: E402

CAP = 1 << 17


def read(L):
    buf = (ctypes.c_ulonglong * (CAP * 12))()
    n = L.vs_debug_tcf_trace(buf, CAP)
    return np.frombuffer(buf, dtype=np.uint64, count=n * 12).reshape(n, 12).astype(np.int64)


def main(only="both"):
    L = vs.lib()
    if not hasattr(L, "vs_debug_tcf_trace"):
        sys.exit("library built without -DVS_TCF_TRACE")
    L.vs_debug_tcf_trace.restype = ctypes.c_int
    L.vs_debug_tcf_trace.argtypes = [ctypes.c_void_p, ctypes.c_int]
    rt = vs.Runtime(bench.bench_config(vs))
    wl = bench.Workload(rt, with_mm=only in ("mm", "both"), with_ch=only in ("ch", "both"))
    for _ in range(3):
        wl.step()
    torch.cuda.synchronize()
    read(L)
    wl.step()
    torch.cuda.synchronize()
    R = read(L)
    rt.close()
    if len(R) == 0:
        sys.exit("no records")
    t0 = R[:, 0].min()
    span = (R[:, 10].max() - t0) / 1e3
    ph = {"prologue (start -> first stage full)": R[:, 2] - R[:, 0],
          "main loop (first full -> last MMA issued)": R[:, 4] - R[:, 2],
          "  of which waiting for operands": R[:, 9],
          "drain (last MMA issued -> accumulator full)": R[:, 6] - R[:, 4],
          "epilogue (accumulator full -> stores done)": R[:, 8] - R[:, 6],
          "exit (stores done -> CTA end)": R[:, 10] - R[:, 8],
          "CTA total": R[:, 10] - R[:, 0]}
    print("%d tcf CTAs in one step (%s), span %.1f ms" % (len(R), only, span / 1e3))
    for k, v in ph.items():
        print("  %-46s median %7.2f us  mean %7.2f us  p90 %7.2f us" % (k, np.median(v) / 1e3, v.mean() / 1e3,
                                                                      np.percentile(v, 90) / 1e3))
    # SM coverage: per SM, the union of its tcf CTAs' intervals over the step span
    busy = 0
    gaps = []
    for sm in np.unique(R[:, 11]):
        r = R[R[:, 11] == sm]
        r = r[np.argsort(r[:, 0])]
        busy += (r[:, 10] - r[:, 0]).sum()
        gaps.extend((r[1:, 0] - r[:-1, 10]).tolist())
    nsm = len(np.unique(R[:, 11]))
    print("  SMs used %d; tcf CTA time covers %.1f%% of (SMs x span); gap between consecutive tcf CTAs on an SM:"
          " median %.2f us, mean %.2f us" % (nsm, 100 * busy / 1e3 / (nsm * span), np.median(gaps) / 1e3,
                                            np.mean(gaps) / 1e3))
    main_us = (R[:, 4] - R[:, 2]) / 1e3
    mma_frac = ((R[:, 4] - R[:, 2]).sum()) / (R[:, 10] - R[:, 0]).sum()
    print("  main-loop share of CTA time %.3f" % mma_frac)
    np.save(os.environ.get("TCF_TRACE_OUT", "/tmp/tcf_trace.npy"), R)
    del main_us


if __name__ == "__main__":
    main(*sys.argv[1:2])

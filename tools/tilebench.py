"""Per-version tile-kernel timing (CUDA events on the launching stream, after warm-up).

python tools/tilebench.py [b ...]   -> one line per (type, version, b): us/task, GFLOP/s
Concurrent mode (--streams S) runs S independent tasks at once on S streams (the
runtime's slots) and reports aggregate GFLOP/s.
"""
import argparse
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import paper_conf_ipps_planasbal13_b200 as vs  # noqa: E402

FLOPS = {vs.VS_T_MATMUL: lambda b: 2 * b ** 3, vs.VS_T_GEMM_NT: lambda b: 2 * b ** 3,
         vs.VS_T_SYRK: lambda b: b ** 3, vs.VS_T_TRSM: lambda b: b ** 3, vs.VS_T_POTRF: lambda b: b ** 3 / 3}
NARGS = {vs.VS_T_MATMUL: 3, vs.VS_T_GEMM_NT: 3, vs.VS_T_SYRK: 2, vs.VS_T_TRSM: 2, vs.VS_T_POTRF: 1}


def bench(ttype, version, b, streams=1, iters=20):
    dt = torch.float64 if version in (vs.VS_V_DFMA_F64, vs.VS_V_DMMA_F64, vs.VS_V_OZ_I8_F64) else torch.float32
    sets = []
    for s in range(streams):
        args = [torch.randn(b, b, dtype=dt, device="cuda") * 0.1 for _ in range(NARGS[ttype])]
        if ttype in (vs.VS_T_POTRF,):
            args[0] = torch.eye(b, dtype=dt, device="cuda") * b
        if ttype == vs.VS_T_TRSM:
            args[0] = torch.eye(b, dtype=dt, device="cuda") * 2 + torch.tril(args[0], -1) * 0.01
        sets.append(args)
    strs = [torch.cuda.Stream() for _ in range(streams)]
    info = torch.zeros(1, dtype=torch.int32, device="cuda")
    # operands in the version's derived forms, built once (as the runtime caches them)
    ptrs = []
    keep = []
    for s in range(streams):
        p = [t.data_ptr() for t in sets[s]]
        fp = []
        for i, t in enumerate(sets[s]):
            f = vs.vs_operand_form(ttype, version, i)
            if f > 0:
                buf = torch.empty(vs.vs_form_bytes(f, b), dtype=torch.uint8, device="cuda")
                vs.vs_form_make(f, b, t.data_ptr(), buf.data_ptr(), torch.cuda.current_stream().cuda_stream)
                keep.append(buf)
                fp.append(buf.data_ptr())
            else:
                fp.append(0)
        ptrs.append(p + fp)
    torch.cuda.synchronize()

    def run():
        for s in range(streams):
            vs.vs_tile_run_prepared(ttype, version, b, ptrs[s], info.data_ptr(), strs[s].cuda_stream)

    for _ in range(3):
        run()
    torch.cuda.synchronize()
    ev0, ev1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    ev0.record()
    for s in strs:
        s.wait_event(ev0)
    for _ in range(iters):
        run()
    for s in strs:
        e = torch.cuda.Event()
        e.record(s)
        torch.cuda.current_stream().wait_event(e)
    ev1.record()
    torch.cuda.synchronize()
    ms = ev0.elapsed_time(ev1)
    per_task_us = ms * 1e3 / (iters * streams)
    gflops = FLOPS[ttype](b) * iters * streams / (ms * 1e-3) / 1e9
    return per_task_us, gflops


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("sizes", nargs="*", type=int, default=[256, 512, 1024])
    ap.add_argument("--streams", type=int, default=1)
    ap.add_argument("--types", default="0,1,2,3,4")
    ap.add_argument("--versions", default="0,1,2,3")
    ap.add_argument("--iters", type=int, default=20)
    a = ap.parse_args()
    for ttype in map(int, a.types.split(",")):
        for version in map(int, a.versions.split(",")):
            for b in a.sizes:
                us, gf = bench(ttype, version, b, a.streams, a.iters)
                print(json.dumps({"type": vs.TYPE_NAMES[ttype], "version": vs.VERSION_NAMES[version], "b": b,
                                  "streams": a.streams, "us_per_task": round(us, 2), "gflops": round(gf, 1)}))
                sys.stdout.flush()


if __name__ == "__main__":
    main()

"""bench.py — tiled matmul + tiled Cholesky GFLOP/s under the versioning scheduler (B200).

One STEP = one pass of the whole hot path over one batch of synthetic input: the tiled
matmul of cfg3 (N=16384 fp32, 1024x1024 tiles, 4096 MATMUL tasks) and the tiled
Cholesky of cfg4 (N=32768 SPD fp32, 1024x1024 tiles, 5984 potrf/trsm/syrk/gemm tasks),
submitted together through the C ABI (vs_app_matmul + vs_app_cholesky) and run to
completion by vs_wait_all: registration -> dependence analysis -> versioning decisions
(learning, then earliest executor) -> device-enforced dependences -> sm_100a tile kernels.

  python bench.py [--gpus N] [--steps K] [--warmup W] [--impl ours|reference]

value = (2*16384^3 + 32768^3/3) algorithmic flops per step x steps / max-over-ranks time.
N > 1 (torchrun, one process per GPU): the SAME problem is sharded (strong scaling):
every tile has an owner rank (2D block-cyclic), every task runs on the owner of the tile
it writes, and tiles owned by another rank are pulled over NVLink from the owner's memory
(CUDA IPC) after the producer's completion tag is visible (vs_dist_init).
--impl reference: the CPU oracle (oracle/) timed on this host's cores on a bounded sample
of the same workload (this tier's reference arm).
"""
from __future__ import annotations

import argparse
import ctypes
import json
import math
import os
import subprocess
import sys
import threading
import time

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)
# the runtime drives ~2 x slots + 3 streams per GPU; with the default 8 hardware work
# queues several streams share one and a critical-path launch waits behind another
# stream's queued work (must be set before the CUDA context exists)
os.environ.setdefault("CUDA_DEVICE_MAX_CONNECTIONS", "32")

MM_N, MM_B = 16384, 1024
CH_N, CH_B = 32768, 1024
SEED_MM, SEED_CH = 3, 4
# runtime configuration the bench times (env VS_SLOTS / VS_PRIORITY / VS_QDEPTH override):
# lambda 3, 12 workers (streams) per GPU, decisions when predecessors completed (ready mode:
# no cross-stream waits, so no stream is blocked at its head), NEXT-4 bottom-level priority
# with a real queue cap of 1 grouped launch (8 tasks) per worker, grouped launches of up to 8
# tc_3xf16 tasks held up to 200 us while their stream still runs a kernel (group_hold),
# critical-path tasks on their own greatest-priority streams, dependences released on the device
# (a3: in-degree counters + CSR successors on the GPU, ready ring; measured within 0.5 % of the
# host release; VS_BENCH_DEVICE_RELEASE=0 switches back)
RT_DEFAULTS = dict(lam=3, slots=12, priority=2, qdepth=1, group=8, mode="ready", hold=1, group_us=200,
                   device_release=int(os.environ.get("VS_BENCH_DEVICE_RELEASE", "1")))
F32_VERSIONS_MASK = 0b100111  # simt_f32 | tc_3xtf32 | f64in_f32io | tc_3xf16 (gemm-type tasks)
MM_FLOPS = lambda n: 2.0 * n ** 3            # noqa: E731  (reading R6)
CH_FLOPS = lambda n: n ** 3 / 3.0            # noqa: E731


def bench_config(vs, **over):
    """vs_config of the timed launch configuration (RT_DEFAULTS), keyword overrides on top."""
    d = RT_DEFAULTS
    kw = dict(lam=d["lam"], slots_per_gpu=d["slots"], priority=d["priority"], queue_depth=d["qdepth"],
              group_tasks=d["group"], mode=1 if d["mode"] == "ready" else 0, group_hold=d["hold"],
              group_wait_us=d["group_us"], device_release=d["device_release"])
    kw.update(over)
    return vs.vs_config_default(**kw)


def ncu_traffic(path=os.path.join(ROOT, "profiles", "r02s4_ncu_full_tcf_bench.csv")):
    """dram__bytes_read.sum + dram__bytes_write.sum of the committed ncu --set full capture of
    one steady-state tcf_gemm_kernel<24,0> launch inside the bench (8 tasks, 128 CTAs; bytes per
    launch), or None."""
    import csv
    scale = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9}
    try:
        tot = 0.0
        for m, unit, v in [r for r in csv.reader(open(path)) if len(r) == 3][1:]:
            if m in ("dram__bytes_read.sum", "dram__bytes_write.sum"):
                tot += float(v) * scale.get(unit, 1)
        return int(tot)
    except (OSError, ValueError):
        return None


def peaks():
    p = os.path.join(ROOT, "MEASURED_PEAKS.json")
    if os.path.exists(p):
        d = json.load(open(p))
        return d, "measured"
    return {"hbm_gbs": 6650.0, "bf16_tflops": 1590.0, "bf16_tflops_sustained": 1400.0, "sm_max_mhz": 1965.0}, "fallback"


def rank_grid(nranks):
    """P_r x P_c process grid for the 2D block-cyclic tile ownership (§8(e))."""
    return {1: (1, 1), 2: (1, 2), 4: (2, 2), 8: (2, 4)}.get(nranks, (1, nranks))


def rank_device(local_rank, ndev):
    """CUDA ordinal of this rank (one process per GPU): LOCAL_RANK; ranks beyond the visible
    devices time-share them round-robin (only used to test multi-rank runs on one GPU).  The
    runtime's gpu 0 is this device (vs_config.device_base), so its streams, replicas and
    kernels live on the rank's own GPU."""
    return local_rank % max(1, ndev)


def tile_owner(i, j, nranks):
    pr, pc = rank_grid(nranks)
    return (i % pr) * pc + (j % pc)


# ----------------------------------------------------------------------------- workload
class Workload:
    """Tiles of cfg3 + cfg4 and their data ids.  Each rank allocates and generates only the
    tiles it owns (vs_gen_tile, bit-identical to vsgen); with nranks > 1 the other ranks'
    tiles are opened through CUDA IPC and registered as owned by them.  host=True (e2e,
    one rank) keeps the tiles in pinned host memory and lets the runtime move them."""

    def __init__(self, rt, mm_n=MM_N, mm_b=MM_B, ch_n=CH_N, ch_b=CH_B, host=False, rank=0, nranks=1, gather=None,
                 mask=F32_VERSIONS_MASK, with_mm=True, with_ch=True, f64=False, seeds=(SEED_MM, SEED_CH)):
        import torch
        import paper_conf_ipps_planasbal13_b200 as vs
        self.torch, self.vs, self.rt = torch, vs, rt
        self.mm_n, self.mm_b, self.ch_n, self.ch_b, self.host = mm_n, mm_b, ch_n, ch_b, host
        self.rank, self.nranks = rank, nranks
        self.with_mm, self.with_ch = with_mm, with_ch
        self.vdt = vs.VS_F64 if f64 else vs.VS_F32
        self.tdt = torch.float64 if f64 else torch.float32
        self.esize = 8 if f64 else 4
        seed_mm, seed_ch = seeds
        self.types = rt.vs_register_builtins(self.vdt, mask)
        self.flops = 0.0
        self.ids = []            # every registered datum (for invalidation)
        self.opened = []         # IPC bases to close
        if with_mm:
            nt = mm_n // mm_b
            self.mm_nt = nt
            all_t = [(i, j) for i in range(nt) for j in range(nt)]
            self.A, self.ia = self._matrix("A", all_t, mm_b, mm_n, lambda T, k, i, j: vs.vs_gen_tile(
                seed_mm, mm_n, mm_n, self.vdt, mm_b, i, j, 0, T[k].data_ptr()), gather)
            self.B, self.ib = self._matrix("B", all_t, mm_b, mm_n, lambda T, k, i, j: vs.vs_gen_tile(
                seed_mm + 1000, mm_n, mm_n, self.vdt, mm_b, i, j, 0, T[k].data_ptr()), gather)
            self.C, self.ic = self._matrix("C", all_t, mm_b, mm_n, None, gather)
            self.flops += MM_FLOPS(mm_n)
        if with_ch:
            nt = ch_n // ch_b
            self.ch_nt = nt
            low = [(i, j) for i in range(nt) for j in range(i + 1)]
            self.S, idl = self._matrix("S", low, ch_b, ch_n, lambda T, k, i, j: vs.vs_gen_tile(
                seed_ch, ch_n, ch_n, self.vdt, ch_b, i, j, 1, T[k].data_ptr()), gather)
            self.S0 = self.S.clone()
            self.iS = {i * nt + j: d for (i, j), d in zip(low, idl)}
            self.flops += CH_FLOPS(ch_n)
        torch.cuda.synchronize()

    def _matrix(self, name, tiles, b, n, gen, gather):
        """Allocate this rank's tiles of one matrix (one buffer), register every tile."""
        torch, vs, rt = self.torch, self.vs, self.rt
        own = [t for t in tiles if tile_owner(t[0], t[1], self.nranks) == self.rank]
        T = torch.zeros((max(1, len(own)), b, b), dtype=self.tdt, device="cuda")
        if gen is not None:
            for k, (i, j) in enumerate(own):
                gen(T, k, i, j)
        if self.host:
            T = T.cpu().pin_memory()
        nbytes = b * b * self.esize
        dev = -1 if self.host else 0
        ids = {}
        for k, t in enumerate(own):
            ids[t] = rt.vs_data_register(T[k].data_ptr(), dev, nbytes)
        if self.nranks > 1:
            h, off = vs.vs_ipc_export(T.data_ptr())
            peers = gather((self.rank, h, off, own))
            for (r, hr, offr, ownr) in peers:
                if r == self.rank:
                    continue
                base = vs.vs_ipc_open(hr, offr)
                self.opened.append(base - offr)
                for k, t in enumerate(ownr):
                    d = rt.vs_data_register(base + k * nbytes, 0, nbytes)
                    rt.vs_data_set_owner(d, r)
                    ids[t] = d
        self.ids.extend(ids.values())
        return T, [ids[t] for t in tiles]

    def reset(self, sync=True):
        """Restore this rank's inputs (C = 0, A_chol = pristine) and declare EVERY datum
        modified (vs_data_invalidate), as if a new batch of inputs had been written: no
        replica, cached remote tile or derived operand form (tc_3xf16 split halves) of the
        previous step is reused, so each step re-does all moves and conversions.  Device:
        async on torch's stream + sync.  Host (e2e): memcpy; the runtime re-transfers every
        tile (the e2e timed region includes those copies)."""
        if self.with_mm:
            self.C.zero_()
        if self.with_ch:
            self.S.copy_(self.S0)
        if not self.host and sync:
            self.torch.cuda.current_stream().synchronize()
        if getattr(self, "_ids_arr", None) is None:
            self._ids_arr = (ctypes.c_int64 * len(self.ids))(*self.ids)
        self.rt.vs_data_invalidate_n(self._ids_arr)

    def submit(self):
        vs, rt = self.vs, self.rt
        if self.with_mm:
            nt = self.mm_nt
            rt.vs_app_matmul(self.types[vs.VS_T_MATMUL], nt, nt, nt, self.ia, self.ib, self.ic)
        if self.with_ch:
            rt.vs_app_cholesky(self.types, self.ch_nt, self.iS)

    def step(self, barrier=None):
        if barrier:
            barrier()      # every rank finished the previous step: none still pulls a tile we restore
        # the restores run on the GPU while the host builds the step's task graph (vs_submit
        # only records tasks and dependences; nothing is issued before vs_wait_all)
        self.reset(sync=False)
        if not self.host and barrier is None and not os.environ.get("VS_BENCH_SYNC"):
            # one process: the runtime's streams wait for the restore on the device
            # (vs_depend_on_event), so the drive's host-side setup overlaps it
            self._ev = self.torch.cuda.Event()
            self._ev.record()
            self.rt.vs_depend_on_event(self._ev)
        self.submit()
        if not self.host and (barrier is not None or os.environ.get("VS_BENCH_SYNC")):
            self.torch.cuda.current_stream().synchronize()
        if barrier:
            barrier()      # owners' resets done before any rank reads their tiles
        self.rt.vs_wait_all()


# ----------------------------------------------------------------------------- clocks
class ClockSampler:
    Q = ("index,clocks.sm,clocks.max.sm,power.draw,clocks_event_reasons.active,clocks_event_reasons.hw_slowdown,"
         "clocks_event_reasons.hw_thermal_slowdown,clocks_event_reasons.sw_thermal_slowdown,"
         "clocks_event_reasons.sw_power_cap")

    def __init__(self, index):
        self.index = index
        self.rows = []
        self.proc = None

    def start(self):
        try:
            self.proc = subprocess.Popen(["nvidia-smi", "-i", str(self.index), "--query-gpu=" + self.Q,
                                          "--format=csv,noheader,nounits", "-lms", "200"],
                                         stdout=subprocess.PIPE, stderr=subprocess.DEVNULL, text=True)
            self.th = threading.Thread(target=self._read, daemon=True)
            self.th.start()
        except Exception:
            self.proc = None

    def _read(self):
        for line in self.proc.stdout:
            self.rows.append([x.strip() for x in line.split(",")])

    def stop(self):
        if self.proc:
            self.proc.terminate()
            try:
                self.proc.wait(timeout=5)
            except Exception:
                self.proc.kill()
        rows = [r for r in self.rows if len(r) >= 9]
        if not rows:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["unavailable"], "samples": 0}
        sm = sorted(float(r[1]) for r in rows if r[1].replace(".", "").isdigit())
        mx = max(float(r[2]) for r in rows if r[2].replace(".", "").isdigit())
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = sorted({names[i] for r in rows for i in range(4) if r[5 + i].lower().startswith("active")})
        return {"sm_mhz": sm[len(sm) // 2] if sm else None, "sm_max_mhz": mx, "reasons": reasons, "samples": len(rows)}


# ----------------------------------------------------------------------------- roofline
def union_ns(intervals):
    tot, cur_s, cur_e = 0, None, None
    for s, e in sorted(intervals):
        if cur_e is None or s > cur_e:
            if cur_e is not None:
                tot += cur_e - cur_s
            cur_s, cur_e = s, e
        else:
            cur_e = max(cur_e, e)
    if cur_e is not None:
        tot += cur_e - cur_s
    return tot


def task_flops(type_name, b):
    t = type_name.split(".")[0]
    return {"MATMUL": 2.0 * b ** 3, "GEMM_NT": 2.0 * b ** 3, "SYRK": 1.0 * b ** 3, "TRSM": 1.0 * b ** 3,
            "POTRF": b ** 3 / 3.0}[t]


def roofline(log, groups, ms, world, launch_of=None):
    pk, pk_kind = peaks()
    tf32_peak = pk.get("bf16_tflops_sustained", pk["bf16_tflops"]) * 0.5   # TF32 = 1/2 BF16 (nominal ratio)
    tnames = {g["type"]: g["type_name"] for g in groups}
    vnames = {g["type"]: g["versions"] for g in groups}
    tile_b = {}
    for g in groups:
        npar = {"MATMUL": 3, "GEMM_NT": 3, "SYRK": 2, "TRSM": 2, "POTRF": 1}[g["type_name"].split(".")[0]]
        tile_b[g["type"]] = int(round(math.sqrt(g["bytes"] / 4 / npar)))
    # per KERNEL class: every tc_3xf16 task but potrf (MATMUL, GEMM_NT, SYRK and TRSM-by-inverse,
    # R30/R31) runs the same kernel, tcf_gemm_kernel (grouped launches mix them); other
    # versions are keyed by (type, version)
    per, per_tv = {}, {}
    for (task, v, w, td, ts, te, ph, ty) in log:
        tname, vname, b = tnames[ty], vnames[ty][v], tile_b[ty]
        fl = task_flops(tname, b)
        kname = "tcf_gemm_kernel" if vname == "tc_3xf16" and not tname.startswith("POTRF") else "%s/%s" % (tname, vname)
        d = per.setdefault(kname, {"n": 0, "flops": 0.0, "iv": [], "version": vname})
        d["n"] += 1
        d["flops"] += fl
        d["iv"].append((ts, te))
        e = per_tv.setdefault((tname, vname, b), {"n": 0, "flops": 0.0})
        e["n"] += 1
        e["flops"] += fl
    dom = max(per, key=lambda k: per[k]["flops"])
    d = per[dom]
    union = union_ns(d["iv"])
    # per launch (the contract's definition): each launch's hardware flops / its own duration
    # (first task start -> last task end of the tasks it ran), averaged over the launches
    per_launch = None
    if launch_of is not None:
        ln = {}
        for rec, lno in zip(log, launch_of):
            (task, v, w, td, ts, te, ph, ty) = rec
            tname, vname = tnames[ty], vnames[ty][v]
            kname = "tcf_gemm_kernel" if vname == "tc_3xf16" and not tname.startswith("POTRF") else "%s/%s" % (tname, vname)
            if kname != dom or lno < 0:
                continue
            e = ln.setdefault(lno, [0.0, ts, te, 0])
            e[0] += task_flops(tname, tile_b[ty])
            e[1], e[2], e[3] = min(e[1], ts), max(e[2], te), e[3] + 1
        if ln:
            hw_l = 3.0 if d["version"] in ("tc_3xtf32", "tc_3xf16") else 1.0
            fl = sum(x[0] for x in ln.values()) * hw_l
            dur = sum(x[2] - x[1] for x in ln.values())
            per_launch = {"launches": len(ln), "tasks_per_launch": round(sum(x[3] for x in ln.values()) / len(ln), 2),
                          "avg_launch_us": round(dur / len(ln) / 1e3, 2),
                          "achieved": round(fl / (dur * 1e-9) / 1e12, 2)}
    f16_peak = pk.get("bf16_tflops_sustained", pk["bf16_tflops"])            # fp16 dense = bf16 dense rate
    tc_peak = {"tc_3xtf32": (tf32_peak, "%s bf16_tflops_sustained x 0.5 (TF32/BF16 nominal ratio)" % pk_kind),
               "tc_3xf16": (f16_peak, "%s bf16_tflops_sustained (fp16 = bf16 dense rate)" % pk_kind)}
    hw = 3.0 if d["version"] in tc_peak else 1.0
    achieved = hw * d["flops"] / (union * 1e-9) / 1e12
    if d["version"] in tc_peak:
        (peak, src), bound = tc_peak[d["version"]], "tensor"
    else:
        peak, bound, src = 148 * 128 * 2 * pk["sm_max_mhz"] * 1e6 / 1e12, "alu", "148 SM x 128 FMA x 2 x sm_max_mhz"
    # tensor-pipe busy fraction of the whole step: hardware MMA flops of every tensor-core
    # task / (step time x that version's peak), summed over versions
    frac_step = sum(3.0 * v["flops"] / tc_peak[k[1]][0] for k, v in per_tv.items() if k[1] in tc_peak) / (ms * 1e-3) / 1e12
    traffic = ncu_traffic() if dom == "tcf_gemm_kernel" else None
    if per_launch:
        per_launch["frac"] = round(per_launch["achieved"] / peak, 4)
    roof = {"bound": bound, "kernel": dom, "tasks": d["n"], "achieved": round(achieved, 2), "peak": round(peak, 1),
            "unit": "TFLOP/s", "frac": round(achieved / peak, 4), "traffic": traffic,
            "traffic_note": ("DRAM bytes of one captured steady-state launch (ncu --set full, "
                             "profiles/r02s4_ncu_full_tcf_bench.csv: tcf_gemm_kernel<24,0>, 8 MATMUL/GEMM_NT tasks, "
                             "128 CTAs; algorithmic reads 8 x (A form 4 MiB + B form 4 MiB + C 4 MiB) = 100.7 MB, "
                             "writes 33.6 MB: operand forms shared with earlier launches hit L2, the C writes leave "
                             "L2 after the kernel)") if traffic else None,
            "per_launch": per_launch,
            "peak_source": src,
            "how": "hardware MMA flops (3x the algorithmic flops of its tasks: 2b^3 matmul/gemm, b^3 syrk/trsm) of "
                   "every task this kernel ran in the timed steps / union of their device-recorded execution "
                   "intervals (%globaltimer, task_ctx.cuh); per_launch: the same flops / the sum of each launch's "
                   "own duration (first task start to last task end), i.e. the average launch rate, which "
                   "counts the time concurrent launches on other streams share the SMs against each launch"}
    counts = {"%s/%s" % k[:2]: v["n"] for k, v in sorted(per_tv.items())}
    return roof, frac_step, counts


def config_json(args, world, mm_n=MM_N, mm_b=MM_B, ch_n=CH_N, ch_b=CH_B, with_mm=True, with_ch=True):
    """The `config` of the JSON line (both arms print the same one)."""
    return {"workload": ("cfg3+cfg4: tiled matmul N=%d b=%d + tiled Cholesky N=%d b=%d, fp32, versions "
                         "simt_f32/tc_3xtf32/f64in_f32io/tc_3xf16, lambda=%d, %d slots/GPU" % (
                             mm_n, mm_b, ch_n, ch_b, args.lam, args.slots)) if with_mm and with_ch else args.only,
            "matmul_N": mm_n if with_mm else None, "cholesky_N": ch_n if with_ch else None,
            "tile": mm_b, "lambda": args.lam, "slots_per_gpu": args.slots,
            "parallelism": ("owner-computes 2D block-cyclic %dx%d, NVLink tile pulls" % rank_grid(world))
            if world > 1 else "1 GPU",
            "l2": "inputs larger than L2 (4 GiB + 4 GiB)", "regime": "warm (tables learned in warm-up)"}


# ----------------------------------------------------------------------------- per-config record
# (name, matmul (N, b) or None, Cholesky (N, b) or None, fp64?, version mask, what it is)
V = lambda *vv: sum(1 << v for v in vv)   # noqa: E731
CONFIGS = [
    ("cfg1_matmul_1024_b256", (1024, 256), None, False, V(0, 1),
     "BASELINE cfg1: tiled matmul N=1024 fp32, 256x256 tiles, versions simt_f32/tc_3xtf32"),
    ("cfg2_cholesky_4096_b512", None, (4096, 512), False, V(0, 1, 2),
     "BASELINE cfg2: tiled Cholesky N=4096 SPD fp32, 512x512 tiles, versions simt_f32/tc_3xtf32/f64in_f32io"),
    ("cfg3_matmul_16384_b1024", (16384, 1024), None, False, F32_VERSIONS_MASK,
     "BASELINE cfg3 alone: tiled matmul N=16384 fp32, 1024x1024 tiles, all f32 versions"),
    ("cfg4_cholesky_32768_b1024", None, (32768, 1024), False, F32_VERSIONS_MASK,
     "BASELINE cfg4 alone: tiled Cholesky N=32768 SPD fp32, 1024x1024 tiles, all f32 versions"),
    ("paper_fp64_matmul_16384_b1024", (16384, 1024), None, True, V(3, 4, 6),
     "paper-shaped matmul (L611-612, reading R3): fp64 N=16384, 1024x1024 tiles, versions dfma_f64/dmma_f64/"
     "oz_i8_f64 (the tcgen05 kind::i8 Ozaki version)"),
    ("paper_cholesky_32768_b2048", None, (32768, 2048), False, F32_VERSIONS_MASK,
     "paper-shaped Cholesky (L700-703, reading R4): fp32 N=32768, 2048x2048 tiles (816 tasks)"),
]


def measure_config(args, vs, torch, name, mm, ch, f64, mask, what, steps=3, warmup=2):
    """One config on its own runtime (the bench's launch configuration), warm: `warmup` untimed
    steps (learning happens in the first), then `steps` steps timed with CUDA events."""
    cfg = bench_config(vs, lam=args.lam, slots_per_gpu=args.slots, priority=args.priority, queue_depth=args.qdepth,
                       group_tasks=args.group, group_hold=args.hold, group_wait_us=args.group_us)
    rt = vs.Runtime(cfg)
    kw = dict(with_mm=mm is not None, with_ch=ch is not None, mask=mask, f64=f64)
    wl = Workload(rt, mm[0] if mm else MM_N, mm[1] if mm else MM_B, ch[0] if ch else CH_N, ch[1] if ch else CH_B, **kw)
    for _ in range(warmup):
        wl.step()
    st0 = rt.vs_stats()
    rt.vs_decision_log_clear()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    for _ in range(steps):
        wl.step()
    e1.record()
    torch.cuda.synchronize()
    ms = e0.elapsed_time(e1) / steps
    st1 = rt.vs_stats()
    groups = rt.vs_group_stats()
    picks = {}
    for r in rt.vs_decision_log():
        g = next(x for x in groups if x["type"] == r[7])
        k = "%s/%s" % (g["type_name"], g["versions"][r[1]])
        picks[k] = picks.get(k, 0) + 1
    tasks = (st1.tasks_completed - st0.tasks_completed) // steps
    out = {"what": what, "value": round(wl.flops / (ms * 1e-3) / 1e9, 1), "unit": "GFLOP/s",
           "ms_per_step": round(ms, 3), "steps": steps, "warmup": warmup, "tasks_per_step": int(tasks),
           "us_per_task_step": round(1e3 * ms / max(1, tasks), 2), "dtype": "f64" if f64 else "f32",
           "decisions_per_step": {k: v // steps for k, v in sorted(picks.items())},
           "learned_mean_us": {"%s/%s" % (g["type_name"], v): round(m / 1e3, 1) for g in groups
                               for v, m in zip(g["versions"], g["mean_ns"]) if m}}
    rt.close()
    del wl
    torch.cuda.empty_cache()
    return out


# ----------------------------------------------------------------------------- reference arm
_CPU = {}


def cpu_sample(target_s=12.0):
    """The oracle as it stands, on a bounded sample of the same workload:
    matmul rows 0..R-1 of C = A*B at N=16384 (fp64, plain i,k,j loop) and the Cholesky of
    the leading k x k block of the cfg4 SPD matrix (L[:k,:k] = chol(A[:k,:k]))."""
    import numpy as np

    import oracle
    import vsgen
    cores = len(os.sched_getaffinity(0))
    os.environ.setdefault("OMP_NUM_THREADS", str(cores))
    if "B" not in _CPU:    # input generation is not part of the timed oracle work
        _CPU["A"] = vsgen.uniform(SEED_MM, 64, MM_N).astype(np.float64)
        _CPU["B"] = vsgen.uniform_idx(SEED_MM + 1000, np.arange(MM_N * MM_N, dtype=np.uint64)).reshape(MM_N, MM_N)
        k = 2048
        r = np.arange(k, dtype=np.uint64)[:, None]
        c = np.arange(k, dtype=np.uint64)[None, :]
        S = vsgen.uniform_idx(SEED_CH, np.maximum(r, c) * np.uint64(CH_N) + np.minimum(r, c))
        S[np.arange(k), np.arange(k)] += vsgen.spd_alpha(CH_N)
        _CPU["S"] = S.astype(np.float32).astype(np.float64)
        t0 = time.perf_counter()
        oracle.matmul(_CPU["A"][:4], _CPU["B"])
        _CPU["dt_row"] = (time.perf_counter() - t0) / 4
    rows = int(max(4, min(64, (target_s / 2) / max(_CPU["dt_row"], 1e-4))))
    t0 = time.perf_counter()
    oracle.matmul(_CPU["A"][:rows], _CPU["B"])
    t_mm = time.perf_counter() - t0
    k = _CPU["S"].shape[0]
    t0 = time.perf_counter()
    _, info = oracle.cholesky(_CPU["S"])
    t_ch = time.perf_counter() - t0
    return {"t_mm": t_mm, "f_mm": 2.0 * rows * MM_N * MM_N, "rows": rows, "t_ch": t_ch, "f_ch": k ** 3 / 3.0,
            "k": k, "cores": cores, "info": info}


def run_reference(args, rank, world):
    if rank != 0:
        return 0
    samples = []
    for i in range(args.warmup + args.steps):
        s = cpu_sample(target_s=4.0)
        if i >= args.warmup:
            samples.append(s)
    t = sum(s["t_mm"] + s["t_ch"] for s in samples)
    f = sum(s["f_mm"] + s["f_ch"] for s in samples)
    gf = f / t / 1e9
    s0 = samples[0]
    sample = ("per step: oracle fp64 matmul rows 0..%d of C=A*B at N=16384 + oracle unblocked Cholesky of the "
              "leading %dx%d block of the cfg4 SPD matrix; value = the sample's flops / its time, not extrapolated "
              "(an upper bound for the full workload: the %dx%d factor is cache-resident)" % (
                  s0["rows"] - 1, s0["k"], s0["k"], s0["k"], s0["k"]))
    out = {"metric": "tiled matmul & Cholesky GFLOP/s", "value": round(gf, 3), "unit": "GFLOP/s", "impl": "reference",
           "n_gpus": args.gpus, "steps": args.steps, "warmup": args.warmup,
           "ms_per_step": round(1e3 * t / len(samples), 2), "higher_is_better": True,
           "scaling": "strong" if world > 1 else "weak", "vs_baseline": None, "dtype": "f64",
           "data": "synthetic (vsgen counter-based generator)",
           "config": config_json(args, world),
           "cpu_baseline": {"value": round(gf, 3), "unit": "GFLOP/s", "cores": s0["cores"], "kind": "oracle",
                            "sample": sample},
           "e2e": {"value": round(gf, 3), "unit": "GFLOP/s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}}
    print(json.dumps(out))
    return 0


# ----------------------------------------------------------------------------- our arm
def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=5)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--impl", default="ours", choices=["ours", "reference"])
    ap.add_argument("--slots", type=int, default=int(os.environ.get("VS_SLOTS", RT_DEFAULTS["slots"])))
    ap.add_argument("--priority", type=int, default=int(os.environ.get("VS_PRIORITY", RT_DEFAULTS["priority"])))
    ap.add_argument("--qdepth", type=int, default=int(os.environ.get("VS_QDEPTH", RT_DEFAULTS["qdepth"])))
    ap.add_argument("--lam", type=int, default=RT_DEFAULTS["lam"])
    ap.add_argument("--mode", choices=["ready", "runahead"], default=os.environ.get("VS_MODE", RT_DEFAULTS["mode"]),
                    help="decide when predecessors completed (ready) or on the virtual clock (runahead)")
    ap.add_argument("--group", type=int, default=int(os.environ.get("VS_GROUP", RT_DEFAULTS["group"])),
                    help="tasks per grouped launch (vs_config.group_tasks)")
    ap.add_argument("--hold", type=int, default=int(os.environ.get("VS_GROUP_HOLD", RT_DEFAULTS["hold"])),
                    help="vs_config.group_hold: idle flush spares groups whose stream still runs a kernel")
    ap.add_argument("--group-us", type=int, default=int(os.environ.get("VS_GROUP_US", RT_DEFAULTS["group_us"])),
                    help="vs_config.group_wait_us")
    ap.add_argument("--no-e2e", action="store_true")
    ap.add_argument("--no-cpu", action="store_true")
    ap.add_argument("--small", action="store_true", help="cfg1/cfg2-sized smoke of the bench itself")
    ap.add_argument("--only", choices=["mm", "ch", "both"], default="both")
    ap.add_argument("--dump-log", default="")
    ap.add_argument("--dump-cold-log", default="", help="decision log of the first (learning) step")
    ap.add_argument("--table-dump", default="", help="write the learned TaskVersionSets after warm-up")
    ap.add_argument("--table-load", default="", help="warm start from a table (NEXT-2 hints)")
    ap.add_argument("--replay", action="store_true", help="decisions from the loaded table (profiling runs)")
    ap.add_argument("--no-configs", action="store_true", help="skip the per-config record (cfg1..cfg4 alone, "
                    "paper-shaped fp64 matmul and b=2048 Cholesky) measured after the timed region")
    args = ap.parse_args()
    rank = int(os.environ.get("RANK", "0"))
    world = int(os.environ.get("WORLD_SIZE", "1"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    if args.impl == "reference":
        return run_reference(args, rank, world)

    import torch
    import paper_conf_ipps_planasbal13_b200 as vs
    ndev = torch.cuda.device_count()
    torch.cuda.set_device(rank_device(local, ndev))
    dist = None
    if world > 1:
        import torch.distributed as dist
        dist.init_process_group("gloo")   # host-side plumbing only (IPC handles, barriers, max)

    def barrier():
        if dist is not None:
            dist.barrier()

    def gather(obj):
        out = [None] * world
        dist.all_gather_object(out, obj)
        return out

    mm_n, mm_b, ch_n, ch_b = (MM_N, MM_B, CH_N, CH_B) if not args.small else (1024, 256, 4096, 512)
    with_mm, with_ch = args.only in ("mm", "both"), args.only in ("ch", "both")
    # critical-path scheduling (NEXT-4: vs_config.priority / queue_depth) is on by default
    # in the bench; --priority 0 --qdepth 0 reproduces the paper-literal rule (R15)
    prio, qdepth = args.priority, args.qdepth
    look = int(os.environ.get("VS_LOOKAHEAD", "0"))
    mode = 1 if args.mode == "ready" else 0          # VS_MODE_READY / VS_MODE_RUNAHEAD
    cfg = vs.vs_config_default(lam=args.lam, slots_per_gpu=args.slots, device_base=rank_device(local, ndev),
                               replay=1 if args.replay else 0, priority=prio, lookahead=look, queue_depth=qdepth,
                               group_tasks=args.group, mode=mode, group_hold=args.hold, group_wait_us=args.group_us,
                               device_release=RT_DEFAULTS["device_release"])
    rt = vs.Runtime(cfg)
    if world > 1:
        shm = gather("/vsched_%d_%d" % (os.getpid(), int(time.time())) if rank == 0 else None)[0]
        if rank == 0:
            rt.vs_dist_init(rank, world, shm)
        barrier()
        if rank != 0:
            rt.vs_dist_init(rank, world, shm)
        barrier()
    wl = Workload(rt, mm_n, mm_b, ch_n, ch_b, host=False, rank=rank, nranks=world, gather=gather if world > 1 else None,
                  with_mm=with_mm, with_ch=with_ch)
    if args.table_load:
        rt.vs_table_load(args.table_load)
        if args.replay:          # replay durations = the loaded means
            for line in open(args.table_load):
                tn, nb, vn, mean, n = line.split()
                for ti in wl.types:
                    if vs.lib().vs_type_name(rt.h, ti).decode() == tn:
                        vi = [vs.lib().vs_version_name(rt.h, ti, v).decode() for v in range(8)
                              if vs.lib().vs_version_name(rt.h, ti, v)].index(vn)
                        rt.vs_replay_set(ti, int(nb), vi, int(mean))
    step_barrier = barrier if world > 1 else None

    # warm-up (the first step includes the learning phase: "cold")
    barrier()
    t0 = time.perf_counter()
    wl.step(step_barrier)
    barrier()
    cold_ms = (time.perf_counter() - t0) * 1e3
    if args.dump_cold_log and rank == 0:
        json.dump({"log": rt.vs_decision_log(), "groups": rt.vs_group_stats()}, open(args.dump_cold_log, "w"))
    for _ in range(args.warmup - 1):
        wl.step(step_barrier)
    if args.table_dump:
        rt.vs_table_dump(args.table_dump)
    barrier()
    rt.vs_decision_log_clear()
    st0 = rt.vs_stats()

    sampler = ClockSampler(torch.cuda.current_device())
    sampler.start()
    time.sleep(0.3)
    barrier()
    torch.cuda.synchronize()
    ev0, ev1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    ev0.record()
    for _ in range(args.steps):
        wl.step(step_barrier)
    barrier()
    ev1.record()
    torch.cuda.synchronize()
    ms = ev0.elapsed_time(ev1)
    clocks = sampler.stop()
    if dist is not None:
        ms = max(gather(ms))
    st1 = rt.vs_stats()
    log = rt.vs_decision_log()
    launch_of = rt.vs_decision_launches()
    groups = rt.vs_group_stats()
    ms_step = ms / args.steps
    gflops = wl.flops * args.steps / (ms * 1e-3) / 1e9       # one problem, sharded over the ranks
    roof, frac_step, version_counts = roofline(log, groups, ms, 1, launch_of)
    launches = st1.kernel_launches - st0.kernel_launches
    if dist is not None:
        launches = sum(gather(int(launches)))

    # ---- e2e: same step through the C ABI with HOST (pinned) buffers, copies inside the timed region
    e2e = None
    if not args.no_e2e and world == 1:
        rt2 = vs.Runtime(vs.vs_config_default(lam=args.lam, slots_per_gpu=args.slots, priority=prio, lookahead=look,
                                              queue_depth=qdepth, group_tasks=args.group, mode=mode,
                                              group_hold=args.hold, group_wait_us=args.group_us,
                                              device_release=RT_DEFAULTS["device_release"]))
        wl2 = Workload(rt2, mm_n, mm_b, ch_n, ch_b, host=True, with_mm=with_mm, with_ch=with_ch)
        wl2.step()     # warm-up incl. learning
        tsum, h2d, d2h = 0.0, 0, 0
        n_e2e = 5   # timed e2e steps (a PCIe hiccup in one of 2 steps moved the number by up to 20 %)
        for _ in range(n_e2e):
            wl2.reset()                      # host restore + invalidate (outside the timing)
            s0 = rt2.vs_stats()
            torch.cuda.synchronize()
            t0 = time.perf_counter()
            wl2.submit()
            rt2.vs_wait_all()                # includes the flush of written tiles to host (Output Tx)
            torch.cuda.synchronize()
            tsum += time.perf_counter() - t0
            s1 = rt2.vs_stats()
            h2d += s1.input_tx_bytes - s0.input_tx_bytes
            d2h += s1.output_tx_bytes - s0.output_tx_bytes
        e2e = {"value": round(wl2.flops * n_e2e / tsum / 1e9, 1), "unit": "GFLOP/s",
               "h2d_bytes_per_step": int(h2d // n_e2e), "d2h_bytes_per_step": int(d2h // n_e2e)}
        rt2.close()
        del wl2

    # ---- per-config record (after the timed region and the e2e leg; one GPU)
    configs = None
    if world == 1 and not args.no_configs and not args.small and args.only == "both":
        configs = {}
        for (name, mm, ch, f64, mask, what) in CONFIGS:
            try:
                configs[name] = measure_config(args, vs, torch, name, mm, ch, f64, mask, what)
            except Exception as ex:   # a failing extra record must not lose the main line
                configs[name] = {"what": what, "error": repr(ex)[:300]}

    cpu = None
    if rank == 0 and world == 1 and not args.no_cpu:
        s = cpu_sample()
        cpu = {"value": round((s["f_mm"] + s["f_ch"]) / (s["t_mm"] + s["t_ch"]) / 1e9, 3), "unit": "GFLOP/s",
               "cores": s["cores"], "kind": "oracle",
               "sample": "oracle fp64 matmul rows 0..%d of C=A*B at N=%d (%.1f s) + oracle unblocked Cholesky of the "
                         "leading %dx%d block of the cfg4 SPD matrix (%.1f s); value = the sample's flops / its time, "
                         "not extrapolated; an upper bound for the full workload (the %dx%d factor is cache-resident, "
                         "the N=%d one is not)" % (
                             s["rows"] - 1, MM_N, s["t_mm"], s["k"], s["k"], s["t_ch"], s["k"], s["k"], CH_N)}

    if rank == 0:
        out = {
            "metric": "tiled matmul & Cholesky GFLOP/s", "value": round(gflops, 1), "unit": "GFLOP/s",
            "n_gpus": world, "steps": args.steps, "warmup": args.warmup, "ms_per_step": round(ms_step, 3),
            "higher_is_better": True, "scaling": "strong" if world > 1 else "weak", "vs_baseline": None, "dtype": "f32",
            "data": "synthetic (counter-based generator; U(-1,1) matmul operands, SPD A = S + 2.5 sqrt(N) I)",
            "config": config_json(args, world, mm_n, mm_b, ch_n, ch_b, with_mm, with_ch),
            "parts_gflop": {"matmul": MM_FLOPS(mm_n) / 1e9 if with_mm else 0,
                            "cholesky": CH_FLOPS(ch_n) / 1e9 if with_ch else 0},
            "cold_first_step_ms": round(cold_ms, 1),
            "tensor_pipe_fraction_step": round(frac_step, 4) if world == 1 else None,
            "roofline": roof,
            "cpu_baseline": cpu, "e2e": e2e, "gpu_launches": int(launches), "clocks": clocks,
            "configs": configs,
            "dependence_tracker": ("device in-degree counters + CSR successors, ready ring (a3): %d of %d tasks released "
                                   "on the GPU" % (st1.device_released - st0.device_released,
                                                   st1.tasks_completed - st0.tasks_completed))
            if st1.device_released > st0.device_released else
            "device completion words (stream memops)" if st1.tracker == 1 else "host (completion ring + cuda events)",
            "runtime_options": {"lookahead": look, "priority": prio, "queue_depth": qdepth, "group_tasks": args.group,
                                "group_hold": args.hold, "group_wait_us": args.group_us,
                                "mode": args.mode, "device_release": RT_DEFAULTS["device_release"],
                                "cuda_device_max_connections": os.environ.get("CUDA_DEVICE_MAX_CONNECTIONS")},
            "tasks_per_step": int((st1.tasks_completed - st0.tasks_completed) / args.steps),
            "version_counts": version_counts,
            "operand_forms_per_step": int((st1.forms_built - st0.forms_built) / args.steps),
            "device_tx_bytes_per_step": int((st1.device_tx_bytes - st0.device_tx_bytes) / args.steps),
            "host_us_per_task": {k: round((getattr(st1, "host_ns_" + k) - getattr(st0, "host_ns_" + k)) / 1e3 / max(1, len(log)), 3)
                                 for k in ("decide", "issue", "launch", "deps", "poll", "poll_idle", "vevent", "flush")},
            # host time per task spent doing work: polls that found completions (they include the
            # decisions and issues those completions trigger; launch and deps are parts of issue)
            # + grouped launches from the loop; the rest of the drive loop waits on the GPU
            "host_busy_us_per_task": round(sum(getattr(st1, "host_ns_" + k) - getattr(st0, "host_ns_" + k)
                                               for k in ("poll", "vevent", "flush"))
                                           / 1e3 / max(1, len(log)) -
                                           (st1.host_ns_poll_idle - st0.host_ns_poll_idle) / 1e3 / max(1, len(log)), 3),
            "host_idle_loops_per_task": round((st1.host_idle_loops - st0.host_idle_loops) / max(1, len(log)), 2),
            "host_us_per_group_launch": round((st1.host_ns_group_launch - st0.host_ns_group_launch) / 1e3 /
                                              max(1, st1.group_launches - st0.group_launches), 2),
            "group_launches_per_step": int((st1.group_launches - st0.group_launches) / args.steps),
            "host_loops_per_task": round((st1.host_loops - st0.host_loops) / max(1, len(log)), 2),
        }
        print(json.dumps(out))
        if args.dump_log:
            json.dump({"log": log, "groups": groups, "issue": rt.vs_decision_issue_ns()}, open(args.dump_log, "w"))
    barrier()
    rt.close()
    if dist is not None:
        dist.destroy_process_group()
    return 0


if __name__ == "__main__":
    sys.exit(main() or 0)

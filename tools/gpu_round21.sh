#!/bin/bash
# ncu full captures of the tc_panel kernel (trsm, potrf) at b=1024
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
timeout 600 ncu --set full --import-source on --clock-control none -k regex:tc_panel -c 1 -f -o gpurun_out/panel_trsm python tools/tilebench.py 1024 --streams 1 --types 2 --versions 1 --iters 1 > gpurun_out/ncu_panel_trsm.log 2>&1
timeout 600 ncu --set full --import-source on --clock-control none -k regex:tc_panel -c 1 -f -o gpurun_out/panel_potrf python tools/tilebench.py 1024 --streams 1 --types 1 --versions 1 --iters 1 > gpurun_out/ncu_panel_potrf.log 2>&1

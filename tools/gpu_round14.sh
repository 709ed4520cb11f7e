#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
VS_DEBUG=1 timeout 150 python tools/dist_debug.py mm 120 > gpurun_out/dist_mm.log 2>&1
echo "exit $?" >> gpurun_out/dist_mm.log
VS_DEBUG=1 timeout 150 python tools/dist_debug.py ch 120 > gpurun_out/dist_ch.log 2>&1
echo "exit $?" >> gpurun_out/dist_ch.log
timeout 200 ./tools/probe_tc2 > gpurun_out/probe_tc2.log 2>&1
echo "exit $?" >> gpurun_out/probe_tc2.log

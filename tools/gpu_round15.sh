#!/bin/bash
cd "${GRAFT_REPO_ROOT:-/root/repo}"
mkdir -p gpurun_out
DBG_PRIO=0 DBG_SIZES=1024,256,2048,256 VS_DEBUG=1 timeout 100 python tools/dist_debug.py both 80 > gpurun_out/dist_a.log 2>&1; echo "exit $?" >> gpurun_out/dist_a.log
DBG_PRIO=1 DBG_SIZES=512,256,1024,256 VS_DEBUG=1 timeout 100 python tools/dist_debug.py both 80 > gpurun_out/dist_b.log 2>&1; echo "exit $?" >> gpurun_out/dist_b.log
DBG_PRIO=1 DBG_SIZES=1024,256,2048,256 VS_DEBUG=1 timeout 100 python tools/dist_debug.py both 80 > gpurun_out/dist_c.log 2>&1; echo "exit $?" >> gpurun_out/dist_c.log

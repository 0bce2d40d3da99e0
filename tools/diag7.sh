cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
O=gpurun_out/diag7.log; : > $O
run() { echo "== $*" >> $O; timeout 100 env "$@" >> $O 2>&1 || echo "rc=$?" >> $O; }
run DIAG_TIMEOUT=60 python tools/split_diag.py C2 0 5
run DIAG_TIMEOUT=60 DIAG_N=2000 python tools/split_diag.py C5 1 10
run DIAG_TIMEOUT=60 DIAG_N=5000 python tools/split_diag.py C5 1 10
run DIAG_TIMEOUT=60 python tools/split_diag.py C5 0 5
run DIAG_TIMEOUT=60 python tools/split_diag.py C4 0 5
run DIAG_TIMEOUT=60 python tools/split_diag.py C1 0 5
grep -v "Exception ignored\|culi.py\", line 28\|NoneType\|^Traceback" $O
echo "== hang probe"
timeout 900 bash tools/hang_probe.sh 3 2>&1 | grep -v "Exception ignored\|culi.py\|NoneType\|^Traceback" | tail -20

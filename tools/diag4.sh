cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
O=gpurun_out/diag4.log; : > $O
run() { echo "== $*" >> $O; timeout 100 env "$@" >> $O 2>&1 || echo "rc=$?" >> $O; }
run CULI_LIB=scratch/libculi_wd.so DIAG_TIMEOUT=60 DIAG_N=500 python tools/split_diag.py C5 1 5
run DIAG_TIMEOUT=60 DIAG_N=2000 python tools/split_diag.py C5 1 10
run DIAG_TIMEOUT=60 DIAG_N=5000 python tools/split_diag.py C5 1 10
run DIAG_TIMEOUT=60 python tools/split_diag.py C2 0 5
grep -v "Exception ignored\|culi.py\", line 28\|NoneType" $O | head -60
echo "== hang probe"
timeout 600 bash tools/hang_probe.sh 2 2>&1 | grep -v "Exception ignored\|culi.py\|NoneType" | tail -20

cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
O=gpurun_out/diag3.log; : > $O
echo "== sanitizer wd lib" >> $O
CULI_LIB=scratch/libculi_wd.so DIAG_TIMEOUT=200 DIAG_N=500 timeout 300 /usr/local/cuda/bin/compute-sanitizer --tool memcheck --show-backtrace device --print-limit 5 python tools/split_diag.py C5 1 1 >> $O 2>&1; echo "rc=$?" >> $O
echo "== sanitizer main lib" >> $O
DIAG_TIMEOUT=200 DIAG_N=500 CULI_WAIT_MS=3000 timeout 300 /usr/local/cuda/bin/compute-sanitizer --tool memcheck --show-backtrace device --print-limit 5 python tools/split_diag.py C5 1 1 >> $O 2>&1; echo "rc=$?" >> $O
grep -v "Exception ignored\|culi.py\", line 28\|NoneType" $O | head -150
